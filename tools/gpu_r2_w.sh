#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_strips.py -q > gpurun_out/r2w_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2w_tests.log
timeout 300 python tools/strip_probe.py > gpurun_out/r2w_probe.jsonl 2> gpurun_out/r2w.err
for n in 256 320 352 512; do AOL_STRIP_REPS=$n timeout 300 python tools/strip_probe.py 2>>gpurun_out/r2w.err | head -1 >> gpurun_out/r2w_probe.jsonl; done
