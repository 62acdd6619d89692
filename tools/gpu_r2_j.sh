#!/bin/bash
# round 2: chain fix, plan epilogue (acq_rel), packed-RGB A/B against the round-1 library
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_chain.py tests/test_gpu_plan.py -q -x > gpurun_out/r2j_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2j_tests.log
timeout 300 python bench.py --extras d1 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2j_bench_d1.json 2> gpurun_out/r2j.err
timeout 600 python tools/chain_probe.py > gpurun_out/r2j_chain.jsonl 2>> gpurun_out/r2j.err
for rep in 1 2 3; do
  for lib in "$PWD/build/rev_d5be606/libaol.so" ""; do
    for cfg in "--dtype rgb8" "--dtype u8"; do
      echo -n "{\"lib\": \"${lib:-HEAD}\", \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/r2j_ab.jsonl
      AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/r2j_ab.jsonl
      echo "}" >> gpurun_out/r2j_ab.jsonl
    done
  done
done
