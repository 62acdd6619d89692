#!/bin/bash
# A/B a previous revision's libaol.so (build/rev_$REV/libaol.so) against the working tree on several configs.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/ab_rev_cfgs.jsonl
for rep in 1 2; do
  for cfg in "" "--dtype u8" "--dtype u8 --out-dtype i16" "--W 352 --H 288 --frames 2000" "--W 3840 --H 2160 --frames 64"; do
    for lib in "$PWD/build/rev_${REV}/libaol.so" ""; do
      echo -n "{\"lib\": \"${lib:-HEAD}\", \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/ab_rev_cfgs.jsonl
      AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/ab_rev_cfgs.jsonl
      echo "}" >> gpurun_out/ab_rev_cfgs.jsonl
    done
  done
done
