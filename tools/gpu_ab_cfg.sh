#!/bin/bash
# A/B experiment builds on one box over several bench configurations, interleaved REPS times.
# VARS="base x y" (build/var_<x>/libaol.so prepared locally, see tools/ab_vars.sh); CFGS = ';'-separated
# bench.py argument lists.  PARITY=1 first runs the fused parity tests against every variant.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
lib() { if [ "$1" = base ]; then echo "$PWD/paper_conf_ipps_guortgbs11_b200/libaol.so"; else echo "$PWD/build/var_$1/libaol.so"; fi; }
OUT=gpurun_out/${TAG:-ab}_cfg.jsonl
if [ "${PARITY:-0}" = "1" ]; then
  for v in ${VARS}; do
    AOL_LIB_PATH=$(lib $v) timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "${PARITY_K:-fused}" > gpurun_out/${TAG:-ab}_parity_$v.log 2>&1
    echo "$v rc=$?" >> gpurun_out/${TAG:-ab}_parity_summary.txt
  done
fi
IFS=';' read -ra CF <<< "${CFGS:---dtype u8}"
for rep in $(seq ${REPS:-3}); do
  for c in "${CF[@]}"; do
    for v in ${VARS}; do
      AOL_LIB_PATH=$(lib $v) timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --extras none $c \
        | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print(json.dumps({'var': '$v', 'cfg': '$c', 'ms': d['ms_per_step'], 'value': d['value'], 'plan': d['launch']['plan']}))" >> $OUT
    done
  done
done
