#!/bin/bash
# int32 ring stages of one row vs one row triple: 4K (default now 1 row) and HD (default triple), A/B interleaved.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
rm -f gpurun_out/rowstage_ab.jsonl
run() { echo -n "{\"case\": \"$1\", \"opts\": $2, \"line\": " >> gpurun_out/rowstage_ab.jsonl
        timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --opts "$2" "${@:3}" | tr -d '\n' >> gpurun_out/rowstage_ab.jsonl
        echo "}" >> gpurun_out/rowstage_ab.jsonl; }
for rep in 1 2; do
  for o in '{}' '{"stages":6}' '{"stages":7}' '{"stages":9}' '{"stages":10}' '{"flags":1024}' '{"flags":1024,"bands_per_unit":24}'; do run 4k "$o" --W 3840 --H 2160 --frames 64; done
  for o in '{}' '{"flags":512}' '{"flags":512,"stages":12}' '{"flags":512,"stages":18}'; do run hd "$o"; done
  for o in '{}' '{"flags":1024}'; do run 4008 "$o" --W 4008 --H 2160 --frames 64; done
done
