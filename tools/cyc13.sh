#!/bin/bash
# C3/C2 build+probe: L2 prefetch window sweep (HAPE_JN_PF); host facts for the out-of-HBM design
mkdir -p gpurun_out
nproc; free -g | head -2; lscpu | grep -E "Model name|Socket|NUMA node\(s\)|Thread"
for pf in 0 32768 131072 262144 1048576; do
  echo "pf=$pf"
  for c in c3 c2; do HAPE_JN_PF=$pf timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline 2>/dev/null | tail -1 | python tools/stages.py; done
done
