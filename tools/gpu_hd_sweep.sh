#!/bin/bash
# HD int32 ring depth x unit size around the planner's choice (5 stages, 10 bands), interleaved twice.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/hd_sweep.jsonl
for rep in 1 2; do
  for st in 4 5 6; do for nb in 8 10 12; do
    echo -n "{\"stages\": $st, \"nb\": $nb, \"line\": " >> gpurun_out/hd_sweep.jsonl
    timeout 300 python bench.py --steps 100 --no-e2e --no-cpu-baseline --opts "{\"stages\":$st,\"bands_per_unit\":$nb}" | tr -d '\n' >> gpurun_out/hd_sweep.jsonl
    echo "}" >> gpurun_out/hd_sweep.jsonl
  done; done
done
