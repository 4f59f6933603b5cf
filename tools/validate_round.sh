#!/bin/bash
# Round validation on the GPU box: smoke, full GPU suite, sanitizers (incl. the
# SR build+probe form forced on int32), the default bench line, the reference arm.
TAG=${1:-r1}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" 2>&1 | tail -1
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -2
S=gpurun_out/sanitizers_$TAG.txt; : > $S
for tool in memcheck racecheck synccheck; do
  echo "== compute-sanitizer --tool $tool --kernel-regex kns=hape python tools/sanitize_case.py" >> $S
  timeout 900 compute-sanitizer --tool $tool --kernel-regex kns=hape python tools/sanitize_case.py 2>&1 | grep -E "SANITIZE|SUMMARY|Invalid|Race|error" | head -8 >> $S
done
echo "== HAPE_JN_SU=2 compute-sanitizer --tool memcheck (SR form on int32 joins)" >> $S
HAPE_JN_SU=2 timeout 900 compute-sanitizer --tool memcheck --kernel-regex kns=hape python tools/sanitize_case.py 2>&1 | grep -E "SANITIZE|SUMMARY|Invalid|error" | head -8 >> $S
cat $S
timeout 900 python bench.py > gpurun_out/bench_default_$TAG.json 2> gpurun_out/bench_default_$TAG.err; tail -1 gpurun_out/bench_default_$TAG.json | python tools/stages.py
timeout 900 python bench.py --impl reference > gpurun_out/bench_reference_$TAG.json 2>&1; tail -1 gpurun_out/bench_reference_$TAG.json | head -c 300; echo
