#!/bin/bash
# round 2: packed-RGB regression bisection by revision
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
for rep in 1 2; do
  for lib in "$PWD/build/rev_d5be606/libaol.so" "$PWD/build/rev_ef7ef9d/libaol.so" "$PWD/build/rev_fabf9c5/libaol.so" ""; do
    for cfg in "--dtype rgb8"; do
      echo -n "{\"lib\": \"${lib:-HEAD}\", \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/r2l_ab.jsonl
      AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/r2l_ab.jsonl
      echo "}" >> gpurun_out/r2l_ab.jsonl
    done
  done
done
