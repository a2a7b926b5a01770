#!/bin/bash
# One GPU session: tests, smoke, bench (both arms), ncu launch list + full captures + Table-1 sizes.
# usage: tools/gpu_round.sh TAG [quick]   (then: python tools/make_profiles.py TAG <prefix>)
set -u
TAG=${1:-r02}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1 || { echo BUILD FAILED; tail -30 $OUT/build.log; exit 1; }
if [ "${2:-}" != "quick" ]; then
  timeout 1800 python -m pytest tests -m gpu -q --timeout 600 -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> $OUT/pytest_gpu.log
  tail -3 $OUT/pytest_gpu.log
  timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo "smoke rc=$?" >> $OUT/smoke.log
fi
timeout 900 python bench.py > $OUT/bench.json 2> $OUT/bench.err; echo "bench rc=$?" >> $OUT/bench.err
timeout 600 python bench.py --impl reference > $OUT/bench_ref.json 2> $OUT/bench_ref.err
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:k_ --csv --log-file $OUT/launches.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-table1 > $OUT/ncu_bench.log 2>&1
for spec in "gemv 4096 4096 auto k_gemv gemv4096" "gesummv 8192 8192 auto k_gemv gesummv8192" "atax 8192 8192 fused k_atax_fused atax8192" "atax 4096 4096 fused k_atax_fused atax4096" "gemv 65536 32768 auto k_gemv gemv65536" "dot 2147483648 0 x k_dot dot2p31" "atax 8192 8192 twopass k_atax_cols atax8192cols" "partial_dot 268435456 0 x k_listing1 listing1_2p28" "sgemv_t 8192 8192 x k_atax_cols sgemvt8192" "atax 8192 32768 fused k_atax_fused_wide atax8192x32768"; do
  set -- $spec
  # (the wide-row kernel's cooperative cluster launch cannot be replayed by ncu: profile its plain launch)
  LIFT_WIDE_COOPERATIVE=0 timeout 300 ncu --set full --clock-control none --import-source on -k regex:$5 -s 2 -c 1 -o $OUT/full_$6 python tools/one_op.py $1 $2 $3 $4 >> $OUT/ncu_full.log 2>&1
done
for name in $(python -c "import bench; print(' '.join(t[0] for t in bench.TABLE1))"); do
  LIFT_WIDE_COOPERATIVE=0 timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed --clock-control none -k regex:^k_ --csv --log-file $OUT/table1_$name.csv python tools/table1.py $name >> $OUT/ncu_table1.log 2>&1
done
cat $OUT/bench.json
