#!/bin/bash
# S-tile size sweep of the SR build+probe; co-processing parity + bench leg
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_coprocess.py -x -q -m gpu 2>&1 | tail -4
B="timeout 300 python bench.py --no-e2e --no-cpu-baseline --no-ablation"
for v in "HAPE_JN_SU=0" "HAPE_JN_SU=1" "HAPE_JN_SU=2" "HAPE_JN_SU=2 HAPE_JN_NSB=3" "HAPE_JN_SU=4" "HAPE_JN_SU=1 HAPE_JN_NSB=3"; do
  echo "== $v"
  for c in c3 c2; do env $v $B --config $c 2>/dev/null | tail -1 | python tools/stages.py; done
done
timeout 600 python bench.py --config c2 --no-cpu-baseline --no-ablation > gpurun_out/bench_cp_c2.json 2> gpurun_out/bench_cp_c2.err
python -c "import json;d=json.loads(open('gpurun_out/bench_cp_c2.json').readlines()[-1]);print(d['e2e']);print(d.get('coprocess'))"
HAPE_JN_SU=1 timeout 600 python -m pytest tests/test_gpu_join.py -x -q -m gpu 2>&1 | tail -2
