#!/bin/bash
# ncu --set full of one fused launch for the bench workload given in BENCH_ARGS (+ NCU_TAG name)
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o gpurun_out/prof_${NCU_TAG} -f python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline ${BENCH_ARGS} > gpurun_out/ncu_${NCU_TAG}.log 2>&1
for o in ${AB_OPTS}; do
  timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline ${BENCH_ARGS} --opts "$o" >> gpurun_out/ab_${NCU_TAG}.jsonl 2>> gpurun_out/ab.err
done
