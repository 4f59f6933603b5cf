#!/bin/bash
# full ncu captures of the hot kernels: tools/ncu_full.sh TAG [bench args]
TAG=$1; shift
B="python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline $*"
for K in ${KERNELS:-k_scatter:12 k_build_probe:3 k_hist:12}; do
  N=${K%%:*}; S=${K##*:}
  timeout 300 ncu --set full --clock-control none --import-source on -k regex:$N -s $S -c 1 -o gpurun_out/prof_${N}_$TAG $B > /dev/null 2>&1
done
ls gpurun_out
