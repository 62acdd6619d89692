#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 300 python tools/pieces_probe.py > gpurun_out/r2t_probe.jsonl 2> gpurun_out/r2t.err
AOL_TILER_PIECES=0 timeout 300 python tools/pieces_probe.py >> gpurun_out/r2t_probe.jsonl 2>> gpurun_out/r2t.err
