#!/bin/bash
# round 2: double-buffered async box loads; memcheck of the box kernels
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q > gpurun_out/r2f_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2f_tests.log
timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2f_bench.json 2> gpurun_out/r2f.err
timeout 600 compute-sanitizer --tool memcheck python tools/tiler_probe_all.py tilers > gpurun_out/r2f_memcheck.log 2>&1
echo "memcheck rc=$?" >> gpurun_out/r2f_memcheck.log
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler_box" -c 12 \
    -o gpurun_out/r2f_box -f python tools/tiler_probe_all.py tilers > gpurun_out/r2f_ncu_box.log 2>&1
