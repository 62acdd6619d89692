#!/bin/bash
# round 2: box tiler kernels, plans, C example; d1 + d3 records
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py tests/test_gpu_plan.py tests/test_gpu_example.py -x -q > gpurun_out/r2c_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2c_tests.log
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "tiler or failed_launch or misaligned or packed_rgb_width or fused_launch or host_streamed" >> gpurun_out/r2c_tests.log 2>&1
echo "tests2 rc=$?" >> gpurun_out/r2c_tests.log
timeout 300 python bench.py --extras d1,d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2c_bench.json 2> gpurun_out/r2c.err
AOL_TILER_BOX=0 timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2c_bench_nobox.json 2>> gpurun_out/r2c.err
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler_box" -c 12 \
    -o gpurun_out/r2c_box -f python tools/tiler_probe_all.py tilers > gpurun_out/r2c_ncu_box.log 2>&1
