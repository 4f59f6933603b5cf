#!/bin/bash
# full GPU suite + smoke + round profile r1d for the config given
CFG=${1:-c2}
mkdir -p gpurun_out
if [ "$CFG" = "c2" ]; then
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke.log 2>&1; tail -1 gpurun_out/smoke.log
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -3 > gpurun_out/tests_r1d.log; cat gpurun_out/tests_r1d.log
fi
bash tools/profile_round.sh r1d $CFG > /dev/null 2>&1
tail -1 gpurun_out/bench_r1d_$CFG.json | python tools/stages.py
