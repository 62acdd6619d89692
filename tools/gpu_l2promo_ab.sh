#!/bin/bash
# TMA L2 promotion A/B (int32 HD, 4K; uint8 HD tensor path), interleaved twice.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/l2promo_ab.jsonl
for rep in 1 2; do for p in 3 0 1 2; do
  for cfg in "" "--W 3840 --H 2160 --frames 64" "--dtype u8"; do
    echo -n "{\"promo\": $p, \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/l2promo_ab.jsonl
    AOL_TMA_L2_PROMO=$p timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/l2promo_ab.jsonl
    echo "}" >> gpurun_out/l2promo_ab.jsonl
  done
done; done
