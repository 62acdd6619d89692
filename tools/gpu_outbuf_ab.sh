#!/bin/bash
# Output staging: two buffers / one barrier per band (default) vs one buffer / two barriers (AOL_FLAG_ONE_OUTBUF).
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_outbuf.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_outbuf.log
rm -f gpurun_out/outbuf_ab.jsonl
for rep in 1 2; do for o in '{}' '{"flags":2048}'; do
  for cfg in "" "--dtype u8" "--dtype u8 --out-dtype i16" "--W 3840 --H 2160 --frames 64" "--W 352 --H 288 --frames 2000" "--W 352 --H 288 --frames 2000 --dtype u8"; do
    echo -n "{\"opts\": $o, \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/outbuf_ab.jsonl
    timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --opts "$o" $cfg | tr -d '\n' >> gpurun_out/outbuf_ab.jsonl
    echo "}" >> gpurun_out/outbuf_ab.jsonl
  done
done; done
