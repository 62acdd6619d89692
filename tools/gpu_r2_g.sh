#!/bin/bash
# round 2: box geometry in smem; fused chain kernel (f3)
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py tests/test_gpu_chain.py -q -x > gpurun_out/r2g_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2g_tests.log
timeout 300 python bench.py --extras d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2g_bench.json 2> gpurun_out/r2g.err
timeout 600 python tools/chain_probe.py > gpurun_out/r2g_chain.jsonl 2>> gpurun_out/r2g.err
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler_box|chain" -c 12 \
    -o gpurun_out/r2g_prof -f python tools/chain_probe.py --ncu > gpurun_out/r2g_ncu.log 2>&1
