#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_plan.py tests/test_gpu_chain.py tests/test_gpu_example.py tests/test_gpu_bench.py -q -x -k "not full_default" > gpurun_out/r2n_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2n_tests.log
for cfg in "--dtype rgb8" "--dtype u8 --out-dtype i16" "--dtype u8" ""; do
  timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --extras none $cfg >> gpurun_out/r2n_bench.jsonl 2>> gpurun_out/r2n.err
done
timeout 300 python bench.py --extras d1 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2n_bench_d1.json 2>> gpurun_out/r2n.err
