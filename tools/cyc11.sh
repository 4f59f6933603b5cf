#!/bin/bash
# re-entry check: full GPU parity suite, smoke, fresh round profiles for c2 and c3
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke.log 2>&1; tail -2 gpurun_out/smoke.log
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -8 > gpurun_out/tests_all.log; cat gpurun_out/tests_all.log
bash tools/profile_round.sh r1b c2 > /dev/null 2>&1
bash tools/profile_round.sh r1b c3 > /dev/null 2>&1
tail -1 gpurun_out/bench_r1b_c2.json | python tools/stages.py
tail -1 gpurun_out/bench_r1b_c3.json | python tools/stages.py
