#!/bin/bash
# the planner's new unit sizes vs the best measured explicit ones (interleaved)
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
rm -f gpurun_out/nb_verify.jsonl
run() { echo -n "{\"case\": \"$1\", \"opts\": $2, \"line\": " >> gpurun_out/nb_verify.jsonl
        timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --opts "$2" "${@:3}" | tr -d '\n' >> gpurun_out/nb_verify.jsonl
        echo "}" >> gpurun_out/nb_verify.jsonl; }
for rep in 1 2; do
  for o in '{}' '{"bands_per_unit":15}' '{"bands_per_unit":12}'; do run i32 "$o"; done
  for o in '{}' '{"bands_per_unit":24}'; do run i32_4k "$o" --W 3840 --H 2160 --frames 64; done
  for o in '{}' '{"bands_per_unit":4}'; do run i32_cif "$o" --W 352 --H 288 --frames 2000; done
  for o in '{}' '{"bands_per_unit":12}'; do run u8i32 "$o" --dtype u8; done
  for o in '{}' '{"bands_per_unit":20}' '{"bands_per_unit":10}'; do run u8i16 "$o" --dtype u8 --out-dtype i16; done
  for o in '{}' '{"bands_per_unit":8}'; do run u8_cif "$o" --dtype u8 --W 352 --H 288 --frames 2000; done
done
