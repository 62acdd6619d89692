#!/bin/bash
# Full round measurement: parity tests, smoke, bench (+ncu launch list and full capture), all configs.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/gpu.txt 2>&1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
timeout 600 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err
timeout 600 python bench.py --dtype u8 --no-cpu-baseline > gpurun_out/bench_u8.json 2>> gpurun_out/bench.err
timeout 600 python bench.py --dtype u8 --out-dtype i16 --no-cpu-baseline > gpurun_out/bench_u8i16.json 2>> gpurun_out/bench.err
timeout 600 python bench.py --dtype rgb8 --no-cpu-baseline > gpurun_out/bench_rgb8.json 2>> gpurun_out/bench.err
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/bench_reference.json 2>> gpurun_out/bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
    python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o gpurun_out/prof_full -f python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/ncu_full.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o gpurun_out/prof_full_u8 -f python bench.py --dtype u8 --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/ncu_full_u8.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o gpurun_out/prof_full_u8i16 -f python bench.py --dtype u8 --out-dtype i16 --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/ncu_full_u8i16.log 2>&1
timeout 900 ncu --set full --clock-control none -k regex:tiler -s 1 -c 2 \
    -o gpurun_out/prof_tiler -f python tools/tiler_probe.py > gpurun_out/ncu_tiler.log 2>&1
timeout 1500 python tools/bench_configs.py > gpurun_out/configs.jsonl 2> gpurun_out/configs.err
for f in 1 2; do timeout 600 python bench.py --dtype u8 --W 3840 --H 2160 --frames 64 --no-cpu-baseline --no-e2e >> gpurun_out/bench_u8_4k.jsonl 2>> gpurun_out/bench.err; done
