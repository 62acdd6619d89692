#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q -x > gpurun_out/r2r_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2r_tests.log
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k tiler >> gpurun_out/r2r_tests.log 2>&1
echo "tests2 rc=$?" >> gpurun_out/r2r_tests.log
timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2r_bench.json 2>> gpurun_out/r2r.err
mkdir -p /tmp/ncu
timeout 900 ncu --set full --clock-control none -k regex:"tiler_box" -c 6 -o /tmp/ncu/box -f python tools/tiler_probe_all.py tilers > gpurun_out/r2r_ncu.log 2>&1
ncu -i /tmp/ncu/box.ncu-rep --page raw --csv > gpurun_out/r2r_box_raw.csv 2>/dev/null
