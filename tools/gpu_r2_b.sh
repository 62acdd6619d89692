#!/bin/bash
# round 2: tiler + boundary GPU tests, ncu --set full of every tiler / filter kernel, u8->i16 consumer capture
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "tiler or failed_launch or misaligned or packed_rgb_width or unaligned or launch_options or two_reps" > gpurun_out/r2b_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2b_tests.log
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler|filter" -c 40 \
    -o gpurun_out/r2b_tiler -f python tools/tiler_probe_all.py > gpurun_out/r2b_ncu_tiler.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o gpurun_out/r2b_u8i16 -f python bench.py --dtype u8 --out-dtype i16 --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/r2b_ncu_u8i16.log 2>&1
timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2b_bench_d3.json 2>> gpurun_out/r2b.err
