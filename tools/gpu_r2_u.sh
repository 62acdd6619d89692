#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py -q > gpurun_out/r2u_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2u_tests.log
timeout 300 python tools/pieces_probe.py > gpurun_out/r2u_probe.jsonl 2> gpurun_out/r2u.err
