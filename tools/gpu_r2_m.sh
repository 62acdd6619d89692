#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
for rep in 1 2; do
  for lib in "$PWD/build/rev_d5be606/libaol.so" ""; do
    for cfg in "--dtype rgb8" "--dtype u8 --out-dtype i16"; do
      echo -n "{\"lib\": \"${lib:-HEAD}\", \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/r2m_ab.jsonl
      AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/r2m_ab.jsonl
      echo "}" >> gpurun_out/r2m_ab.jsonl
    done
  done
done
