set -u
OUT=gpurun_out/r01u; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1 || { tail -20 $OUT/build.log; exit 1; }
timeout 300 python tools/atax_grid.py > $OUT/atax_grid.txt 2>&1; echo "rc=$?" >> $OUT/atax_grid.txt
timeout 300 python tools/table1.py > $OUT/table1.txt 2>&1; echo "rc=$?" >> $OUT/table1.txt
for name in partial_dot_2^20 partial_dot_2^28 dot_listing1_2^28 sgemv_t_8192x8192 sgemv_t_8192x8192_beta; do
  timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed --clock-control none -k regex:^k_ --csv --log-file $OUT/table1_$name.csv python tools/table1.py $name >> $OUT/ncu_table1.log 2>&1
done
cat $OUT/atax_grid.txt $OUT/table1.txt
