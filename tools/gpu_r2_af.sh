#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out /tmp/ncu
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o /tmp/ncu/r2af_u8i16 -f python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --extras none --dtype u8 --out-dtype i16 > gpurun_out/r2af.log 2>&1
ncu -i /tmp/ncu/r2af_u8i16.ncu-rep --page raw --csv > gpurun_out/r2af_raw.csv 2>>gpurun_out/r2af.log
ncu -i /tmp/ncu/r2af_u8i16.ncu-rep --page source --csv --print-source sass > gpurun_out/r2af_source.csv 2>>gpurun_out/r2af.log
