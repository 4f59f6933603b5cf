#!/bin/bash
# Round profiling artefacts (run under gpurun): bench line, clocks, per-launch
# ncu list of one bench step, and one --set full capture per hot kernel.
TAG=${1:-r1}
CFG=${2:-c2}
mkdir -p gpurun_out
nvidia-smi --query-gpu=index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active --format=csv -lms 200 > gpurun_out/clocks_${TAG}_${CFG}.csv &
SMI=$!
timeout 600 python bench.py --config $CFG > gpurun_out/bench_${TAG}_${CFG}.json 2> gpurun_out/bench_${TAG}_${CFG}.err
kill $SMI
B="python bench.py --config $CFG --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-ablation --no-coprocess"
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}_${CFG}.csv $B > /dev/null 2>&1
# per-launch skip counts: 3 warm-up steps precede the profiled one
# (two-pass plans: one joint histogram per relation and step, 4 scatters)
NH=$((3*2)); NS=$((3*4)); NB=3; HK=k_hist_joint
if [ "$CFG" = "c1" ]; then NH=6; NS=6; HK=k_hist; fi
for K in $HK:$NH k_scatter:$NS k_build_probe:$NB; do
  N=${K%%:*}; S=${K##*:}
  R=gpurun_out/full_${TAG}_${CFG}_${N}
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$N -s $S -c 1 -o $R $B > /dev/null 2>&1
  # exports instead of the report (gpurun returns at most 64 MiB): the raw
  # metrics page and the per-SASS-line source page
  ncu -i $R.ncu-rep --page raw --csv > $R.raw.csv 2>/dev/null
  ncu -i $R.ncu-rep --page source --csv --print-source sass 2>/dev/null | gzip > $R.sass.csv.gz
  [ -z "$NCU_KEEP_REP" ] && rm -f $R.ncu-rep
done
ls -la gpurun_out
