#!/bin/bash
# round 2: packed-RGB regression bisection (round-1 lib vs HEAD vs HEAD without the plan epilogue / PDL waits)
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
for rep in 1 2; do
  for lib in "$PWD/build/rev_d5be606/libaol.so" "$PWD/build/ab_noplan/libaol.so" "$PWD/build/ab_noplan_nopdl/libaol.so" ""; do
    for cfg in "--dtype rgb8" "--dtype rgb8 --out-dtype i16" "--dtype u8 --out-dtype i16"; do
      echo -n "{\"lib\": \"${lib:-HEAD}\", \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/r2k_ab.jsonl
      AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/r2k_ab.jsonl
      echo "}" >> gpurun_out/r2k_ab.jsonl
    done
  done
done
