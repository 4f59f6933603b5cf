#!/bin/bash
# sweep an env var over values, print per-stage ms: tools/sweep.sh VAR "v1 v2 ..." [bench args]
VAR=$1; VALS=$2; shift 2
for x in $VALS; do
  env $VAR=$x timeout 300 python bench.py --no-e2e --no-cpu-baseline --steps 5 "$@" 2>&1 | tail -1 | python -c "
import json,sys
l=sys.stdin.readline()
try:
  d=json.loads(l); print('$VAR=$x', round(d['ms_per_step'],3), {k:v['ms'] for k,v in d['roofline']['stages'].items()})
except Exception as e: print('$VAR=$x FAILED', l[:300])"
done
