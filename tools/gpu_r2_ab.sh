#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
for i in 1 2; do
timeout 300 python bench.py --dtype rgb8 --extras none --no-cpu-baseline --no-e2e --steps 50 > gpurun_out/r2ab_rgb_$i.json 2>> gpurun_out/r2ab.err
timeout 300 python bench.py --dtype rgb8 --out-dtype i16 --extras none --no-cpu-baseline --no-e2e --steps 50 > gpurun_out/r2ab_rgbh_$i.json 2>> gpurun_out/r2ab.err
done
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_plan.py -q -x -k "packed or rgb or Packed" > gpurun_out/r2ab_tests.log 2>&1
