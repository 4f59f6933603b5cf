#!/bin/bash
# one GPU round-trip: parity tests, bench line, per-launch ncu list
#   NO_TESTS=1 skips pytest, NO_NCU=1 skips the launch list, BENCH_ARGS passes through
TAG=${1:-x}
mkdir -p gpurun_out
if [ -z "$NO_TESTS" ]; then
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -5 > gpurun_out/tests_$TAG.log
cat gpurun_out/tests_$TAG.log
fi
timeout 300 python bench.py ${BENCH_ARGS} 2>&1 | tail -2 > gpurun_out/bench_$TAG.log
cat gpurun_out/bench_$TAG.log
if [ -z "$NO_NCU" ]; then
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv --log-file gpurun_out/launches_$TAG.csv python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline ${BENCH_ARGS} > /dev/null 2>&1
fi
