#!/bin/bash
# f3 separable chain: GPU chain tests with the register-resident column filter (default) and with the Y ring
# (AOL_SEP_REG=0), then the f3 bench record under both, interleaved
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out; T=${TAG:-f3ab}
timeout 900 python -m pytest tests/test_gpu_chain.py -x -q > gpurun_out/${T}_pytest_reg.log 2>&1; echo "rc=$?" >> gpurun_out/${T}_pytest_reg.log
AOL_SEP_REG=0 timeout 900 python -m pytest tests/test_gpu_chain.py -x -q > gpurun_out/${T}_pytest_ring.log 2>&1; echo "rc=$?" >> gpurun_out/${T}_pytest_ring.log
for rep in 1 2; do
  for v in 1 0; do
    AOL_SEP_REG=$v timeout 300 python bench.py --extras f3 --no-cpu-baseline --no-e2e --steps 5 \
      | python -c "import json,sys; d=json.loads(sys.stdin.readline()); r=d['records']['f3']; print(json.dumps({'sep_reg': $v, 'ms': r['ms'], 'frac': r['frac'], 'parity': r['parity'], 'kernel': r['kernel']}))" >> gpurun_out/${T}.jsonl
  done
done
