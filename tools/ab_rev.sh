#!/bin/bash
# A/B a previous git revision against the working tree on the same box.
# usage (inside gpurun): REV=<sha> DTYPES="i32 u8" bash tools/ab_rev.sh   (needs build/rev_<sha>/libaol.so prepared locally)
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
for rep in 1 2 3; do
  for d in ${DTYPES:-i32}; do
    AOL_LIB_PATH=$PWD/build/rev_${REV}/libaol.so timeout 300 python bench.py --dtype $d --steps 50 --no-e2e --no-cpu-baseline | sed "s/^{/{\"rev\": \"${REV}\", /" >> gpurun_out/ab_rev.jsonl
    timeout 300 python bench.py --dtype $d --steps 50 --no-e2e --no-cpu-baseline | sed 's/^{/{"rev": "HEAD", /' >> gpurun_out/ab_rev.jsonl
  done
done
