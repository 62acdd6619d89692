#!/bin/bash
# round 2: fused chain v2
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_chain.py -q -x > gpurun_out/r2h_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2h_tests.log
timeout 600 python tools/chain_probe.py > gpurun_out/r2h_chain.jsonl 2>> gpurun_out/r2h.err
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"chain" -c 1 \
    -o gpurun_out/r2h_prof -f python tools/chain_probe.py --ncu > gpurun_out/r2h_ncu.log 2>&1
