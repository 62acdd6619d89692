#!/bin/bash
# packed 24-bit pixel path: CTAs per SM x unit size x ring depth (int32 and int16 outputs), interleaved twice.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/rgb_sweep.jsonl
for rep in 1 2; do
  for out in i32 i16; do
    for o in '{}' '{"ctas_per_sm":2}' '{"ctas_per_sm":2,"stages":4}' '{"bands_per_unit":8}' '{"bands_per_unit":30}' '{"stages":5}' '{"stages":10}'; do
      echo -n "{\"out\": \"$out\", \"opts\": $o, \"line\": " >> gpurun_out/rgb_sweep.jsonl
      timeout 300 python bench.py --dtype rgb8 --out-dtype $out --steps 50 --no-cpu-baseline --opts "$o" | tr -d '\n' >> gpurun_out/rgb_sweep.jsonl
      echo "}" >> gpurun_out/rgb_sweep.jsonl
    done
  done
done
