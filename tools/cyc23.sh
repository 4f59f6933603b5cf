#!/bin/bash
mkdir -p gpurun_out
bash tools/profile_round.sh r1c c3 > /dev/null 2>&1
tail -1 gpurun_out/bench_r1c_c3.json | python tools/stages.py
