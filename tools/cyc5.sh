python -c "import __graft_entry__ as g; g.build()"
B="python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline"
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_hist_joint -s 6 -c 1 -o gpurun_out/prof_hj $B > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_scatter -s 6 -c 1 -o gpurun_out/prof_sc1 $B > /dev/null 2>&1
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv --log-file gpurun_out/launches_j1.csv $B > /dev/null 2>&1
ls gpurun_out
