#!/bin/bash
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out /tmp/aolprobe
NV="/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -Xcompiler -fPIC,-fvisibility=hidden -DAOL_PROBE_STREAM_ONLY"
for f in paper_conf_ipps_guortgbs11_b200/csrc/*.cu; do $NV -c -o /tmp/aolprobe/$(basename $f .cu).o $f & done; wait
/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o /tmp/aolprobe/libaol.so /tmp/aolprobe/*.o -lrt -ldl -lpthread
for o in "{}" "{\"stages\":24}" "{\"ctas_per_sm\":1}" "{\"ctas_per_sm\":4,\"stages\":8}"; do
  AOL_LIB_PATH=/tmp/aolprobe/libaol.so timeout 300 python bench.py --dtype u8 --steps 50 --no-e2e --no-cpu-baseline --opts "$o" >> gpurun_out/stream_probe_u8.jsonl 2>> gpurun_out/stream_probe.err
done
