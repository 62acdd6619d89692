#!/bin/bash
# bands-per-unit sweep (work-unit size) for uint8 (int32 / int16 outputs) and int32 HD, 4K.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/nb_sweep.jsonl
run() { echo -n "{\"case\": \"$1\", \"opts\": $2, \"line\": " >> gpurun_out/nb_sweep.jsonl
        timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --opts "$2" "${@:3}" | tr -d '\n' >> gpurun_out/nb_sweep.jsonl
        echo "}" >> gpurun_out/nb_sweep.jsonl; }
for rep in 1 2; do
  for nb in 0 20 24 30 40 60 120; do run u8i32 "{\"bands_per_unit\":$nb}" --dtype u8; done
  for nb in 0 20 24 30 40 60 120; do run u8i16 "{\"bands_per_unit\":$nb}" --dtype u8 --out-dtype i16; done
  for nb in 0 10 12 20 24 30; do run i32 "{\"bands_per_unit\":$nb}"; done
  for nb in 0 12 16 20 30 60; do run u8_4k "{\"bands_per_unit\":$nb}" --dtype u8 --W 3840 --H 2160 --frames 64; done
  for nb in 0 8 16 32; do run u8_cif "{\"bands_per_unit\":$nb}" --dtype u8 --W 352 --H 288 --frames 2000; done
done
