#!/bin/bash
# A/B: 16-bit chain heads (HAPE_H16) vs 32-bit; slot bits grow while occupancy holds
P=paper_conf_cidr_chrysogelossa19_b200
for v in u32 h16; do cp variants/lib_$v.so $P/libhape.so; echo "== $v"
  for c in c2 c3 c2; do timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline --no-ablation 2>/dev/null | tail -1 | python tools/stages.py; done
done
cp variants/lib_h16.so $P/libhape.so
timeout 900 python -m pytest tests/test_gpu_join.py -m gpu -q -x 2>&1 | tail -2
