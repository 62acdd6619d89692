#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out /tmp/ncu
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tiler_pieces -o /tmp/ncu/r2v_pieces -f python tools/pieces_probe.py --once > gpurun_out/r2v_ncu.log 2>&1
ncu -i /tmp/ncu/r2v_pieces.ncu-rep --page raw --csv > gpurun_out/r2v_pieces_raw.csv 2>> gpurun_out/r2v_ncu.log
ncu -i /tmp/ncu/r2v_pieces.ncu-rep --page details --csv > gpurun_out/r2v_pieces_details.csv 2>> gpurun_out/r2v_ncu.log
