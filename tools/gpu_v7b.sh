#!/bin/bash
# Second pass of the round's full measurement: GPU tests (incl. sanitizers), uint8->int16 bench, all configs.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/pytest_gpu_b.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu_b.log
for i in 1 2 3; do timeout 600 python bench.py --dtype u8 --out-dtype i16 --no-cpu-baseline --no-e2e >> gpurun_out/bench_u8i16_b.jsonl 2>> gpurun_out/bench_b.err; done
for i in 1 2; do timeout 600 python bench.py --dtype u8 --no-cpu-baseline --no-e2e >> gpurun_out/bench_u8_b.jsonl 2>> gpurun_out/bench_b.err; done
timeout 1500 python tools/bench_configs.py > gpurun_out/configs_b.jsonl 2> gpurun_out/configs_b.err
