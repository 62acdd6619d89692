cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out /tmp/ncu
B="python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --extras none"
$B --frames 1 > gpurun_out/p1_d1_plain.log 2>&1 && \
ncu --metrics gpu__time_duration.sum,sm__cycles_active.avg,launch__grid_size --clock-control none --csv --log-file gpurun_out/p1_d1_launches.csv $B --frames 1 > /dev/null 2>&1
for v in base c4; do
  L=$PWD/paper_conf_ipps_guortgbs11_b200/libaol.so; [ $v = base ] || L=$PWD/build/var_$v/libaol.so
  AOL_LIB_PATH=$L timeout 600 ncu --set full --clock-control none --import-source on -k regex:fused_tma -s 3 -c 1 \
     -o /tmp/ncu/p1_$v -f $B --steps 1 --dtype u8 --out-dtype i16 > gpurun_out/p1_ncu_$v.log 2>&1
  ncu -i /tmp/ncu/p1_$v.ncu-rep --page source --csv --print-source sass > gpurun_out/p1_src_$v.csv 2>&1
  ncu -i /tmp/ncu/p1_$v.ncu-rep --page raw --csv > gpurun_out/p1_raw_$v.csv 2>&1
done
