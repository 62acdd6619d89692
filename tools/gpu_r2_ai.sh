#!/bin/bash
# launch-option sweep for the direct-store int16 paths
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
: > gpurun_out/r2ai.jsonl
for dt in "u8 --out-dtype i16" "rgb8 --out-dtype i16"; do
  for o in '{}' '{"ctas_per_sm":2}' '{"ctas_per_sm":3}' '{"ctas_per_sm":4}' '{"stages":4}' '{"stages":6}' '{"stages":9}' '{"stages":12}' '{"bands_per_unit":10}' '{"bands_per_unit":30}' '{"bands_per_unit":40}'; do
    timeout 300 python bench.py --dtype $dt --extras none --no-cpu-baseline --no-e2e --steps 50 --opts "$o" 2>>gpurun_out/r2ai.err | python -c "
import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print(json.dumps({'dtype':'$dt','opts':'$o','ms':d['ms_per_step'],'fps':d['value'],'plan':d.get('launch',{}).get('plan') or d.get('config',{}).get('plan')}))" >> gpurun_out/r2ai.jsonl
  done
done
