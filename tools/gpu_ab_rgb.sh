#!/bin/bash
# packed-pixel path: previous build (build/rev_$REV) vs working tree, interleaved 3x
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "packed" > gpurun_out/pytest_rgb5.log 2>&1; echo "rc=$?" >> gpurun_out/pytest_rgb5.log
rm -f gpurun_out/ab_rgb.jsonl
for rep in 1 2 3; do for out in i32 i16; do for lib in "$PWD/build/rev_${REV}/libaol.so" ""; do
  echo -n "{\"lib\": \"${lib:-HEAD}\", \"out\": \"$out\", \"line\": " >> gpurun_out/ab_rgb.jsonl
  AOL_LIB_PATH=$lib timeout 300 python bench.py --dtype rgb8 --out-dtype $out --steps 50 --no-e2e --no-cpu-baseline | tr -d '\n' >> gpurun_out/ab_rgb.jsonl
  echo "}" >> gpurun_out/ab_rgb.jsonl
done; done; done
