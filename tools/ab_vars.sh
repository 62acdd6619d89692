#!/bin/bash
# A/B experiment builds on one box: VARS="base x y" (build/var_<x>/libaol.so, built locally with
# `make BUILD=build/var_x LIB=build/var_x/libaol.so EXTRA=-D... build/var_x/libaol.so`), interleaved REPS times.
# PARITY=1 first runs the GPU parity tests against every variant.  BENCH_ARGS are passed to bench.py.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
lib() { if [ "$1" = base ]; then echo "$PWD/paper_conf_ipps_guortgbs11_b200/libaol.so"; else echo "$PWD/build/var_$1/libaol.so"; fi; }
if [ "${PARITY:-0}" = "1" ]; then
  for v in ${VARS}; do
    AOL_LIB_PATH=$(lib $v) timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "${PARITY_K:-fused}" > gpurun_out/parity_$v.log 2>&1
    echo "$v rc=$?" >> gpurun_out/parity_summary.txt
  done
fi
for rep in $(seq ${REPS:-3}); do
  for d in ${DTYPES:-u8}; do
    for v in ${VARS}; do
      AOL_LIB_PATH=$(lib $v) timeout 300 python bench.py --dtype $d --steps 50 --no-e2e --no-cpu-baseline ${BENCH_ARGS} \
        | sed "s/^{/{\"var\": \"$v\", \"in\": \"$d\", /" >> gpurun_out/ab_vars.jsonl
    done
  done
done
