#!/bin/bash
# A/B launch-option sweep on one box: each config run twice, interleaved.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 300 python tools/bw_probe.py > gpurun_out/bw_probe.json 2>&1
rm -f gpurun_out/ab.jsonl
for rep in 1 2; do
  for o in ${AB_OPTS}; do
    timeout 300 python bench.py --steps 100 --no-e2e --no-cpu-baseline --opts "$o" >> gpurun_out/ab.jsonl 2>> gpurun_out/ab.err
  done
done
