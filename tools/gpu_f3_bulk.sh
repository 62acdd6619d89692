#!/bin/bash
# f3 register-resident separable chain: bulk-copy (TMA) row staging vs cp.async (AOL_SEP_BULK=0), x row buffers
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out; T=${TAG:-f3bulk}
timeout 900 python -m pytest tests/test_gpu_chain.py -x -q > gpurun_out/${T}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${T}_pytest.log
for rep in 1 2; do
  for bulk in 1 0; do
    for nbuf in ${NBUFS:-3 4}; do
      AOL_SEP_BULK=$bulk AOL_SEP_NBUF=$nbuf timeout 300 python bench.py --extras f3 --no-cpu-baseline --no-e2e --steps 5 \
        | python -c "import json,sys; d=json.loads(sys.stdin.readline()); r=d['records']['f3']; print(json.dumps({'bulk': $bulk, 'nbuf': $nbuf, 'ms': r['ms'], 'two_ms': r['two_launches_ms'], 'frac': r['frac'], 'parity': r['parity'], 'two_equal': r['two_launches_equal']}))" >> gpurun_out/${T}.jsonl
    done
  done
done
