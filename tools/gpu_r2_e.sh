#!/bin/bash
# round 2: box tilers with the smem attribute, plans; d1/d3 records; ncu of the box kernels
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py tests/test_gpu_plan.py tests/test_gpu_example.py -q > gpurun_out/r2e_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2e_tests.log
timeout 300 python bench.py --extras d1,d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2e_bench.json 2> gpurun_out/r2e.err
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler_box" -c 12 \
    -o gpurun_out/r2e_box -f python tools/tiler_probe_all.py tilers > gpurun_out/r2e_ncu_box.log 2>&1
