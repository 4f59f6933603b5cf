#!/bin/bash
# same-box A/B of env variants on bench legs: tools/ab_legs.sh TAG LEGS "ENV=..." ...
TAG=$1; LEGS=$2; shift 2
mkdir -p gpurun_out
B="python bench.py --steps 2 --warmup 3 --legs $LEGS --no-e2e --no-cpu-baseline --no-ablation --no-coprocess"
for v in "base" "$@"; do
  if [ "$v" = "base" ]; then E=""; else E="$v"; fi
  echo "== $v"
  env $E timeout 900 $B 2> gpurun_out/abl_${TAG}.err | tail -1 > gpurun_out/abl_${TAG}_cur.json
  cat gpurun_out/abl_${TAG}_cur.json >> gpurun_out/abl_$TAG.jsonl
  python tools/legs.py gpurun_out/abl_${TAG}_cur.json
done
