#!/bin/bash
# A/B: build+probe unique path with 4-CTA register cap (a) vs uncapped (b)
P=paper_conf_cidr_chrysogelossa19_b200
mkdir -p gpurun_out
for v in a b; do
  cp variants/libhape_$v.so $P/libhape.so
  echo "== $v"
  timeout 600 python -m pytest tests/test_gpu_join.py -x -q -m gpu 2>&1 | tail -2
  for c in c2 c3; do timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline 2>/dev/null | tail -1 | python tools/stages.py; done
  HAPE_SLOT_EXTRA=1 timeout 300 python bench.py --config c2 --no-e2e --no-cpu-baseline 2>/dev/null | tail -1 | python tools/stages.py
done
