#!/bin/bash
# round-2 GPU round trip: GPU suite (or a -k selection), default bench line
# (with legs), per-launch ncu list of one C2 step.
#   TESTS="-k loopback" selects tests; NO_TESTS / NO_BENCH / NO_NCU skip parts
TAG=${1:-x}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv,noheader
if [ -z "$NO_TESTS" ]; then
  timeout 1500 python -m pytest tests -m gpu -x -q $TESTS 2>&1 | tail -15 > gpurun_out/tests_$TAG.log
  cat gpurun_out/tests_$TAG.log
fi
if [ -z "$NO_BENCH" ]; then
  timeout 900 python bench.py $BENCH_ARGS > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err
  tail -3 gpurun_out/bench_$TAG.err; tail -1 gpurun_out/bench_$TAG.json | python tools/stages.py
fi
if [ -z "$NO_NCU" ]; then
  timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv --log-file gpurun_out/launches_$TAG.csv python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-ablation --no-coprocess --legs none $NCU_ARGS > /dev/null 2>&1
  python tools/launches.py gpurun_out/launches_$TAG.csv | tail -25
fi
