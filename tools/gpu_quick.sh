#!/bin/bash
# Quick GPU check: parity tests + bench (+ optional ncu full capture when NCU=1).
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 600 python bench.py ${BENCH_ARGS} > gpurun_out/bench.json 2> gpurun_out/bench.err
for o in ${EXTRA_OPTS}; do
  timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --opts "$o" >> gpurun_out/bench_opts.jsonl 2>> gpurun_out/bench.err
done
if [ "${NCU:-0}" = "1" ]; then
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
      python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
      -o gpurun_out/prof_fused -f python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/ncu_full.log 2>&1
fi
