#!/bin/bash
P=paper_conf_cidr_chrysogelossa19_b200
mkdir -p gpurun_out
cp variants/lib_prev.so $P/libhape.so; echo "== prev"; timeout 300 python tools/dbg_exchange.py c1:262144:262151 2>&1 | tail -2
cp variants/lib_base.so $P/libhape.so; echo "== base gdb"
timeout 600 cuda-gdb -batch -ex run -ex bt -ex "info registers rip" --args python tools/dbg_exchange.py c1:262144:262151 2>&1 | grep -vE "^\[New Thread|^\[Thread|Detaching|^$" | tail -30
for v in base lean56 lean65; do cp variants/lib_$v.so $P/libhape.so; echo "== $v"
  for i in 1 2; do timeout 300 python bench.py --config c2 --no-e2e --no-cpu-baseline --no-ablation 2>/dev/null | tail -1 | python tools/stages.py; done; done
