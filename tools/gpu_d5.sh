#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 600 python tools/bench_configs.py --only d5 > gpurun_out/configs_d5.jsonl 2> gpurun_out/configs_d5.err
AOL_DIST_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29541 \
   bench.py --gpus 2 --stream-frames 2000 --pool 256 --steps 3 --warmup 1 > gpurun_out/bench_d5_2rank.json 2> gpurun_out/bench_d5_2rank.err
echo "rc=$?" >> gpurun_out/bench_d5_2rank.err
