#!/bin/bash
# Which kernel do racecheck / initcheck complain about?  One sanitizer run per (tool, dtype, kernel).
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/sanitize2_summary.txt
for tool in racecheck initcheck; do
  for dt in i32 u8; do
    for k in 1 2; do
      timeout 600 compute-sanitizer --tool $tool --error-exitcode 3 python tools/sanitize_workload.py --fused-only --dtypes $dt --kernels $k > gpurun_out/san_${tool}_${dt}_k${k}.log 2>&1
      echo "$tool $dt kernel=$k rc=$? $(grep -E 'SUMMARY' gpurun_out/san_${tool}_${dt}_k${k}.log | head -1)" >> gpurun_out/sanitize2_summary.txt
    done
  done
done
timeout 600 compute-sanitizer --tool memcheck --error-exitcode 3 python tools/sanitize_workload.py > gpurun_out/san_memcheck_all.log 2>&1
echo "memcheck all rc=$? $(grep -E 'SUMMARY' gpurun_out/san_memcheck_all.log | head -1)" >> gpurun_out/sanitize2_summary.txt
timeout 600 compute-sanitizer --tool synccheck --error-exitcode 3 python tools/sanitize_workload.py > gpurun_out/san_synccheck_all.log 2>&1
echo "synccheck all rc=$? $(grep -E 'SUMMARY' gpurun_out/san_synccheck_all.log | head -1)" >> gpurun_out/sanitize2_summary.txt
