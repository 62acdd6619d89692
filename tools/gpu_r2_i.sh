#!/bin/bash
# round 2: box tilers with 16-byte async row copies
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q -x > gpurun_out/r2i_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2i_tests.log
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k tiler >> gpurun_out/r2i_tests.log 2>&1
echo "tests2 rc=$?" >> gpurun_out/r2i_tests.log
timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2i_bench.json 2> gpurun_out/r2i.err
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler_box" -c 12 \
    -o gpurun_out/r2i_box -f python tools/tiler_probe_all.py tilers > gpurun_out/r2i_ncu_box.log 2>&1
