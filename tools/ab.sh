#!/bin/bash
# same-box A/B of env variants on one bench workload: prints step ms and stages
#   tools/ab.sh TAG "ENV1=a ENV2=b" "ENV3=c" ...   (BENCH_ARGS passes through)
TAG=$1; shift
mkdir -p gpurun_out
B="python bench.py --steps 10 --legs none --no-e2e --no-cpu-baseline --no-ablation --no-coprocess $BENCH_ARGS"
for v in "base" "$@"; do
  if [ "$v" = "base" ]; then E=""; else E="$v"; fi
  echo "== $v"
  env $E timeout 600 $B 2> gpurun_out/ab_${TAG}.err | tail -1 | tee -a gpurun_out/ab_$TAG.jsonl | python tools/stages.py
done
