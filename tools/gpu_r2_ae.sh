#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
: > gpurun_out/r2ae_summary.txt
timeout 300 python tools/sanitize_workload.py > gpurun_out/r2ae_plain.log 2>&1; echo "plain rc=$?" >> gpurun_out/r2ae_summary.txt
timeout 600 compute-sanitizer --tool racecheck --error-exitcode 3 python tools/sanitize_workload.py --chain-only > gpurun_out/r2ae_race.log 2>&1; echo "racecheck chain rc=$?" >> gpurun_out/r2ae_summary.txt
timeout 900 compute-sanitizer --tool memcheck --error-exitcode 3 python tools/sanitize_workload.py > gpurun_out/r2ae_memcheck.log 2>&1; echo "memcheck rc=$?" >> gpurun_out/r2ae_summary.txt
