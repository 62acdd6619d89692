#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python bench.py > gpurun_out/r2aa_bench.json 2> gpurun_out/r2aa_bench.err
