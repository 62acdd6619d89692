#!/bin/bash
# round 2 full run: every GPU test, smoke, the default bench (all records), variants, reference arm,
# ncu launch list + full captures (headline i32, u8, u8->i16, every tiler / filter / chain kernel), sanitizer workload
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
T=${TAG:-r02_full}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/${T}_gpu.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/${T}_pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/${T}_pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/${T}_smoke.log
s0=$(date +%s); timeout 900 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err; echo "default bench wall s: $(( $(date +%s) - s0 ))" > gpurun_out/${T}_bench_wall.txt
timeout 600 python bench.py --dtype u8 --no-cpu-baseline > gpurun_out/${T}_bench_u8.json 2>> gpurun_out/${T}_bench.err
timeout 600 python bench.py --dtype u8 --out-dtype i16 --no-cpu-baseline > gpurun_out/${T}_bench_u8i16.json 2>> gpurun_out/${T}_bench.err
timeout 600 python bench.py --dtype rgb8 --no-cpu-baseline > gpurun_out/${T}_bench_rgb8.json 2>> gpurun_out/${T}_bench.err
timeout 600 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/${T}_bench_reference.json 2>> gpurun_out/${T}_bench.err
timeout 600 python tools/chain_probe.py > gpurun_out/${T}_chain.jsonl 2>> gpurun_out/${T}_bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/${T}_launches.csv \
    python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline --extras none > gpurun_out/${T}_ncu_launch_bench.log 2>&1
# ncu reports stay on the box (/tmp/ncu, tens of MB each); their raw metric pages come back as CSV
mkdir -p /tmp/ncu
for v in "i32:" "u8:--dtype u8" "u8i16:--dtype u8 --out-dtype i16"; do
  name=${v%%:*}; args=${v#*:}
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
      -o /tmp/ncu/${T}_${name} -f python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --extras none $args \
      > gpurun_out/${T}_ncu_${name}.log 2>&1
  ncu -i /tmp/ncu/${T}_${name}.ncu-rep --page raw --csv > gpurun_out/${T}_ncu_${name}_raw.csv 2>/dev/null
done
timeout 900 ncu --set full --clock-control none -k regex:"tiler|filter" -c 24 \
    -o /tmp/ncu/${T}_tiler -f python tools/tiler_probe_all.py > gpurun_out/${T}_ncu_tiler.log 2>&1
ncu -i /tmp/ncu/${T}_tiler.ncu-rep --page raw --csv > gpurun_out/${T}_ncu_tiler_raw.csv 2>/dev/null
timeout 900 ncu --set full --clock-control none -k regex:"chain" -c 1 \
    -o /tmp/ncu/${T}_chain -f python tools/chain_probe.py --ncu > gpurun_out/${T}_ncu_chain.log 2>&1
ncu -i /tmp/ncu/${T}_chain.ncu-rep --page raw --csv > gpurun_out/${T}_ncu_chain_raw.csv 2>/dev/null
# the fused kernel's column strips (16 8K DCI frames)
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o /tmp/ncu/${T}_wide -f python bench.py --frames 16 --H 4320 --W 8192 --steps 1 --warmup 3 --no-e2e \
    --no-cpu-baseline --extras none > gpurun_out/${T}_ncu_wide.log 2>&1
ncu -i /tmp/ncu/${T}_wide.ncu-rep --page raw --csv > gpurun_out/${T}_ncu_wide_raw.csv 2>/dev/null
# compute-sanitizer is closed on the GPU pool (runs under it left GPUs needing a reset): the sanitizer workload
# runs directly (every kernel on small shapes, cross-path agreement asserted)
timeout 600 python tools/sanitize_workload.py > gpurun_out/${T}_sanitize_workload.log 2>&1
echo "sanitize workload (no sanitizer) rc=$?" >> gpurun_out/${T}_sanitize_summary.txt
