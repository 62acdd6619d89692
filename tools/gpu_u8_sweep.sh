#!/bin/bash
# uint8 launch-option sweep (int32 and int16 outputs): ring depth, bands per unit, CTAs per SM.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/u8_sweep.jsonl
run() { echo -n "{\"out\": \"$1\", \"opts\": $2, \"line\": " >> gpurun_out/u8_sweep.jsonl
        timeout 300 python bench.py --dtype u8 --out-dtype $1 --steps 50 --no-e2e --no-cpu-baseline --opts "$2" | tr -d '\n' >> gpurun_out/u8_sweep.jsonl
        echo "}" >> gpurun_out/u8_sweep.jsonl; }
for rep in 1 2; do
  for o in '{}' '{"stages":6}' '{"stages":8}' '{"stages":14}' '{"bands_per_unit":6}' '{"bands_per_unit":24}'; do run i32 "$o"; done
  for o in '{}' '{"stages":4}' '{"stages":6}' '{"stages":10}' '{"bands_per_unit":6}' '{"bands_per_unit":24}' '{"ctas_per_sm":4}' '{"ctas_per_sm":4,"flags":32}'; do run i16 "$o"; done
done
