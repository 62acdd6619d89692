#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_plan.py tests/test_gpu_example.py -q -x > gpurun_out/r2o_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2o_tests.log
timeout 300 python bench.py --extras d1 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2o_bench_d1.json 2>> gpurun_out/r2o.err
