#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out /tmp/ncu
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"chain" -c 1 \
    -o /tmp/ncu/chain -f python tools/chain_probe.py --ncu > gpurun_out/r2p_ncu.log 2>&1
ncu -i /tmp/ncu/chain.ncu-rep --page raw --csv > gpurun_out/r2p_chain_raw.csv 2>/dev/null
ncu -i /tmp/ncu/chain.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/r2p_chain_src.csv 2>/dev/null
gzip -f gpurun_out/r2p_chain_src.csv
