#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out /tmp/ncu
timeout 600 ncu --set full --import-source on --clock-control none -k regex:sep_chain -c 1 -o /tmp/ncu/r2z_sep -f python tools/chain_probe.py --ncu > gpurun_out/r2z_ncu.log 2>&1
ncu -i /tmp/ncu/r2z_sep.ncu-rep --page raw --csv > gpurun_out/r2z_sep_raw.csv 2>> gpurun_out/r2z_ncu.log
ncu -i /tmp/ncu/r2z_sep.ncu-rep --page details --csv > gpurun_out/r2z_sep_details.csv 2>> gpurun_out/r2z_ncu.log
ncu -i /tmp/ncu/r2z_sep.ncu-rep --page source --csv --print-source sass > gpurun_out/r2z_sep_source.csv 2>> gpurun_out/r2z_ncu.log
