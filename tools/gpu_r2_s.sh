#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q > gpurun_out/r2s_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2s_tests.log
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k tiler >> gpurun_out/r2s_tests.log 2>&1
echo "tests2 rc=$?" >> gpurun_out/r2s_tests.log
timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2s_bench.json 2>> gpurun_out/r2s.err
AOL_TILER_PIECES=0 timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2s_bench_nopieces.json 2>> gpurun_out/r2s.err
