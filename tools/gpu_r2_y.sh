#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_chain.py -q > gpurun_out/r2y_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2y_tests.log
timeout 300 python tools/chain_probe.py > gpurun_out/r2y_probe.jsonl 2> gpurun_out/r2y.err
AOL_CHAIN_SEP=0 timeout 300 python tools/chain_probe.py >> gpurun_out/r2y_probe.jsonl 2>> gpurun_out/r2y.err
