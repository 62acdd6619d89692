#!/bin/bash
# A/B: pre-PDL-chain build (build/rev_$REV) vs HEAD with 256-byte L2 promotion (isolates the PDL chain) vs HEAD.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
rm -f gpurun_out/ab_pdl.jsonl
cat > /tmp/d1_min.py <<'PY'
import json, os, sys
sys.path.insert(0, os.getcwd())
import torch
import paper_conf_ipps_guortgbs11_b200 as aol
sys.argv = [sys.argv[0]]
exec(open("tools/d1_sweep.py").read().split("x = aol.synth_frames")[0])
x = aol.synth_frames(0, 0, 1, 3, 1080, 1920)
z = torch.empty((1, 3, 480, 720), dtype=torch.int32, device="cuda")
cs = torch.empty(1, dtype=torch.uint64, device="cuda")
print(json.dumps({"d1_cs_us": graph_us(x, z, cs, None), "d1_nocs_us": graph_us(x, z, None, None)}))
PY
for rep in 1 2 3; do
  for v in old promo3 head; do
    lib=""; env=""
    [ $v = old ] && lib="$PWD/build/rev_${REV}/libaol.so"
    [ $v = promo3 ] && env="AOL_TMA_L2_PROMO=3"
    d1=$(env $env AOL_LIB_PATH=$lib timeout 300 python /tmp/d1_min.py | tail -1)
    b=$(env $env AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline | tr -d '\n')
    u=$(env $env AOL_LIB_PATH=$lib timeout 300 python bench.py --dtype u8 --steps 50 --no-e2e --no-cpu-baseline | tr -d '\n')
    echo "{\"v\": \"$v\", \"d1\": $d1, \"i32\": $b, \"u8\": $u}" >> gpurun_out/ab_pdl.jsonl
  done
done
