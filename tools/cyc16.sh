#!/bin/bash
# full GPU suite + smoke + round profiles (r1c) for c2 and c3
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke.log 2>&1; tail -1 gpurun_out/smoke.log
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -4
bash tools/profile_round.sh r1c c2 > /dev/null 2>&1
bash tools/profile_round.sh r1c c3 > /dev/null 2>&1
for c in c2 c3; do tail -1 gpurun_out/bench_r1c_$c.json | python tools/stages.py; python -c "import json;d=json.loads(open('gpurun_out/bench_r1c_$c.json').readlines()[-1]);print(d['e2e']);print(d.get('coprocess'));print(d.get('nonpartitioned_gpu',{}).get('radix_speedup'))"; done
