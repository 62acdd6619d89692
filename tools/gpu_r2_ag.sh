#!/bin/bash
# A/B: previous build (ab/libaol_prev.so) vs the working tree on uint8 -> int16, alternating on one box
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
: > gpurun_out/r2ag.jsonl
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_plan.py -q -x -k "u8 or int16 or packed" > gpurun_out/r2ag_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2ag_tests.log
for i in 1 2 3; do
  for lib in ab/libaol_prev.so paper_conf_ipps_guortgbs11_b200/libaol.so; do
    for dt in "u8 --out-dtype i16" "u8"; do
      AOL_LIB_PATH=$PWD/$lib timeout 300 python bench.py --dtype $dt --extras none --no-cpu-baseline --no-e2e --steps 50 2>>gpurun_out/r2ag.err | python -c "
import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print(json.dumps({'lib':'$lib','dtype':'$dt','ms':d['ms_per_step'],'fps':d['value']}))" >> gpurun_out/r2ag.jsonl
    done
  done
done
