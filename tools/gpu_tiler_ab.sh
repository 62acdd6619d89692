#!/bin/bash
# Tiler A/B: blocked table kernel for wrapping gathers / FAST scatters (default) vs element-by-element.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "tiler or filter" > gpurun_out/pytest_tiler.log 2>&1
echo "pytest rc=$?" >> gpurun_out/pytest_tiler.log
rm -f gpurun_out/tiler_ab.jsonl
for rep in 1 2; do
  AOL_TILER_WRAPTAB=0 timeout 300 python tools/tiler_probe2.py >> gpurun_out/tiler_ab.jsonl 2>&1
  timeout 300 python tools/tiler_probe2.py >> gpurun_out/tiler_ab.jsonl 2>&1
done
