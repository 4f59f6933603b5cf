#!/bin/bash
# one --set full capture of the first launch of kernel K after S skips, with
# an env variant: tools/ncu_one.sh TAG KERNEL SKIP "ENV=..." [bench args]
TAG=$1; K=$2; S=$3; E=$4; shift 4
mkdir -p gpurun_out
B="python bench.py --steps 1 --warmup 3 --legs none --no-e2e --no-cpu-baseline --no-ablation --no-coprocess $*"
R=gpurun_out/full_${TAG}_${K}
env $E timeout 600 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 -o $R $B > /dev/null 2>&1
ncu -i $R.ncu-rep --page raw --csv > $R.raw.csv 2>/dev/null
ncu -i $R.ncu-rep --page source --csv --print-source sass 2>/dev/null | gzip > $R.sass.csv.gz
rm -f $R.ncu-rep
