#!/bin/bash
# round 2, first check: new bench sub-records + full-stream parity tests
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
nproc > gpurun_out/r2a_nproc.txt; free -g >> gpurun_out/r2a_nproc.txt
timeout 600 python bench.py > gpurun_out/r2a_bench.json 2> gpurun_out/r2a_bench.err
timeout 1200 python -m pytest tests/test_gpu_bench.py tests/test_gpu_parity.py -k "bench or 4k or d5" -x -q > gpurun_out/r2a_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2a_tests.log
