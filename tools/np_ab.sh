#!/bin/bash
# A/B of the non-partitioned join (bench nonpartitioned_gpu) across env variants
for v in "base" "$@"; do
  if [ "$v" = "base" ]; then E=""; else E="$v"; fi
  echo "== $v"
  env $E timeout 600 python bench.py --steps 2 --warmup 3 --legs none --no-e2e --no-cpu-baseline --no-coprocess $BENCH_ARGS 2>/dev/null | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); n=d.get('nonpartitioned_gpu'); print(d['config']['workload'][:3], n['ms_per_step'], n['stages_ms'], n['radix_speedup'], n['same_result_as_radix'])"
done
