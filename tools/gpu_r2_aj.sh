#!/bin/bash
# A/B: ab/libaol_prev.so (staged bulk-store outputs) vs the working tree (direct stores for 8-bit samples)
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
: > gpurun_out/r2aj.jsonl
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_plan.py tests/test_gpu_strips.py -q -x > gpurun_out/r2aj_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2aj_tests.log
for i in 1 2; do
  for lib in ab/libaol_prev.so paper_conf_ipps_guortgbs11_b200/libaol.so; do
    for dt in "u8 --out-dtype i16" "u8" "rgb8" "rgb8 --out-dtype i16" "u8 --out-dtype i16 --H 288 --W 352 --frames 2000" "u8 --H 2160 --W 3840 --frames 64"; do
      AOL_LIB_PATH=$PWD/$lib timeout 300 python bench.py --dtype $dt --extras none --no-cpu-baseline --no-e2e --steps 50 2>>gpurun_out/r2aj.err | python -c "
import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print(json.dumps({'lib':'$lib','dtype':'$dt','ms':d['ms_per_step'],'fps':d['value']}))" >> gpurun_out/r2aj.jsonl
    done
  done
done
