#!/bin/bash
# build+probe with the S tile ring (SR): parity (default and forced SR) + A/B
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_join.py -x -q -m gpu 2>&1 | tail -2
HAPE_JN_SR=1 timeout 600 python -m pytest tests/test_gpu_join.py -x -q -m gpu 2>&1 | tail -2
B="timeout 300 python bench.py --no-e2e --no-cpu-baseline --no-ablation"
for v in "HAPE_JN_SR=0" "HAPE_JN_SR=1" "HAPE_JN_SR=1 HAPE_JN_NSB=2" "HAPE_JN_SR=1 HAPE_JN_NSB=4" "HAPE_JN_SR=1 HAPE_JN_NRB=2"; do
  echo "== $v"
  for c in c3 c2; do env $v $B --config $c 2>/dev/null | tail -1 | python tools/stages.py; done
done
