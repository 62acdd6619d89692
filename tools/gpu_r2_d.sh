#!/bin/bash
# round 2: box (table) tilers, plans with PDL, u8 neighbour-word shuffle A/B
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tiler_box.py tests/test_gpu_plan.py tests/test_gpu_example.py -x -q > gpurun_out/r2d_tests.log 2>&1
echo "tests rc=$?" >> gpurun_out/r2d_tests.log
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "u8 or rgb or packed or tiler or fused" >> gpurun_out/r2d_tests.log 2>&1
echo "tests2 rc=$?" >> gpurun_out/r2d_tests.log
timeout 300 python bench.py --extras d1,d3 --steps 5 --no-e2e --no-cpu-baseline > gpurun_out/r2d_bench.json 2> gpurun_out/r2d.err
for rep in 1 2 3; do
  for lib in "$PWD/build/ab_nbrlds/libaol.so" ""; do
    for cfg in "--dtype u8" "--dtype u8 --out-dtype i16"; do
      echo -n "{\"lib\": \"${lib:-HEAD}\", \"cfg\": \"$cfg\", \"line\": " >> gpurun_out/r2d_u8ab.jsonl
      AOL_LIB_PATH=$lib timeout 300 python bench.py --steps 50 --no-e2e --no-cpu-baseline $cfg | tr -d '\n' >> gpurun_out/r2d_u8ab.jsonl
      echo "}" >> gpurun_out/r2d_u8ab.jsonl
    done
  done
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"tiler_box" -c 12 \
    -o gpurun_out/r2d_box -f python tools/tiler_probe_all.py tilers > gpurun_out/r2d_ncu_box.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
    -o gpurun_out/r2d_u8i16 -f python bench.py --dtype u8 --out-dtype i16 --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/r2d_ncu_u8i16.log 2>&1
