#!/bin/bash
# build+probe: 512 consumer threads per CTA vs 256
B="timeout 300 python bench.py --no-e2e --no-cpu-baseline --no-ablation --no-coprocess"
for v in "HAPE_JN_NC=256" "HAPE_JN_NC=512" "HAPE_JN_NC=512 HAPE_JN_SU=2" "HAPE_JN_NC=512 HAPE_JN_SU=1" "HAPE_JN_NC=512 HAPE_JN_SU=2 HAPE_JN_NSB=3"; do
  echo "== $v"; for c in c3 c2; do env $v $B --config $c 2>/dev/null | tail -1 | python tools/stages.py; done; done
HAPE_JN_NC=512 timeout 900 python -m pytest tests/test_gpu_join.py -m gpu -q -x 2>&1 | tail -2
