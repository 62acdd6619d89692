#!/bin/bash
# int32 smem-layout A/B: linear rows (1-D bulk copies) vs SWIZZLE_32B lines (W % 32 != 0) and vs SWIZZLE_128B
# tensor loads (W % 32 == 0), each config run twice, interleaved.  Parity tests of the affected paths first.
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "unaligned or linear_rows or wide_unaligned or width_limits or swizzle or fused" \
    > gpurun_out/pytest_layout.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_layout.log
rm -f gpurun_out/ab_layout.jsonl
run() { echo -n "{\"case\": \"$1\", \"line\": " >> gpurun_out/ab_layout.jsonl
        timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline "${@:2}" | tr -d '\n' >> gpurun_out/ab_layout.jsonl
        echo "}" >> gpurun_out/ab_layout.jsonl; }
for rep in 1 2; do
  run "720x576 linear" --W 720 --H 576 --frames 1000
  run "720x576 swz32" --W 720 --H 576 --frames 1000 --opts '{"flags":256}'
  run "1000x1080 linear" --W 1000 --H 1080 --frames 300
  run "1000x1080 swz32" --W 1000 --H 1080 --frames 300 --opts '{"flags":256}'
  run "4008x2160 linear" --W 4008 --H 2160 --frames 64
  run "4008x2160 generic" --W 4008 --H 2160 --frames 64 --opts '{"kernel":2}'
  run "1920x1080 swz128" --frames 300
  run "1920x1080 linear" --frames 300 --opts '{"flags":128}'
  run "3840x2160 swz128" --W 3840 --H 2160 --frames 64
  run "3840x2160 linear" --W 3840 --H 2160 --frames 64 --opts '{"flags":128}'
done
