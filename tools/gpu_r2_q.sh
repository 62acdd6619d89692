#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q -x > gpurun_out/r2q_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2q_tests.log
AOL_TILER_BOX_NBUF=1 timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q -x >> gpurun_out/r2q_tests.log 2>&1
echo "tests nbuf1 rc=$?" >> gpurun_out/r2q_tests.log
for nb in "" 1 2; do
  AOL_TILER_BOX_NBUF=$nb timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline >> gpurun_out/r2q_bench.jsonl 2>> gpurun_out/r2q.err
done
