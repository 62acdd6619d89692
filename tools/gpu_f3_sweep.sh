#!/bin/bash
# f3 register-resident separable chain: X row buffers (AOL_SEP_NBUF) x bands per unit (AOL_SEP_BANDS)
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out; T=${TAG:-f3sweep}
for nbuf in ${NBUFS:-3 4 6 8}; do
  for bands in ${BANDS:-8 16 24}; do
    AOL_SEP_NBUF=$nbuf AOL_SEP_BANDS=$bands timeout 300 python bench.py --extras f3 --no-cpu-baseline --no-e2e --steps 5 \
      | python -c "import json,sys; d=json.loads(sys.stdin.readline()); r=d['records']['f3']; print(json.dumps({'nbuf': $nbuf, 'bands': $bands, 'ms': r['ms'], 'frac': r['frac'], 'parity': r['parity'], 'kernel': r['kernel']}))" >> gpurun_out/${T}.jsonl
  done
done
