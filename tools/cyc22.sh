#!/bin/bash
# full GPU suite + smoke + c2 round profile (r1c)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke.log 2>&1; tail -1 gpurun_out/smoke.log
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -3 > gpurun_out/tests_r1c.log; cat gpurun_out/tests_r1c.log
bash tools/profile_round.sh r1c c2 > /dev/null 2>&1
tail -1 gpurun_out/bench_r1c_c2.json | python tools/stages.py
ls -la gpurun_out | head -30
