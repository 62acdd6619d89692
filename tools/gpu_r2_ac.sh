#!/bin/bash
# A/B: previous build (ab/libaol_prev.so) vs the working tree, alternating on one box
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
: > gpurun_out/r2ac.jsonl
for i in 1 2 3; do
  for lib in ab/libaol_prev.so paper_conf_ipps_guortgbs11_b200/libaol.so; do
    for dt in "rgb8" "rgb8 --out-dtype i16"; do
      AOL_LIB_PATH=$PWD/$lib timeout 300 python bench.py --dtype $dt --extras none --no-cpu-baseline --no-e2e --steps 50 2>>gpurun_out/r2ac.err | python -c "
import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print(json.dumps({'lib':'$lib','dtype':'$dt','ms':d['ms_per_step'],'fps':d['value']}))" >> gpurun_out/r2ac.jsonl
    done
  done
done
