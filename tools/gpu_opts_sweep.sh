#!/bin/bash
# launch-option sweep of one bench configuration: BASE = bench.py args, OPTS = ';'-separated JSON option sets
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out; T=${TAG:-opts}
IFS=';' read -ra OS <<< "${OPTS:-{\}}"
for rep in 1 2; do
  for o in "${OS[@]}"; do
    timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --extras none $BASE --opts "$o" \
      | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print(json.dumps({'base': '$BASE', 'opts': '$o', 'ms': d['ms_per_step'], 'value': d['value'], 'plan': d['launch']['plan']}))" >> gpurun_out/${T}.jsonl
  done
done
