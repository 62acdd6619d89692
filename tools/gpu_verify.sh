#!/bin/bash
# quick verification of a change: selected GPU tests (PYTEST_K), the default bench line, bench configurations (CFGS)
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out; T=${TAG:-verify}
timeout 1200 python -m pytest tests -m gpu -x -q ${PYTEST_K:+-k "$PYTEST_K"} > gpurun_out/${T}_pytest.log 2>&1; echo "pytest rc=$?" >> gpurun_out/${T}_pytest.log
[ "${DEFAULT_BENCH:-1}" = 1 ] && timeout 900 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
IFS=';' read -ra CF <<< "${CFGS:-}"
for c in "${CF[@]}"; do
  timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline --extras none $c \
    | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print(json.dumps({'cfg': '$c', 'ms': d['ms_per_step'], 'value': d['value'], 'plan': d['launch']['plan'], 'mix': d['roofline'].get('mix_ceiling')}))" >> gpurun_out/${T}_cfg.jsonl
done
