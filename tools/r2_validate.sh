#!/bin/bash
# Round-2 validation on the GPU box: smoke, full GPU suite, sanitizers, the
# default bench line, the reference arm, the C2 launch list and one
# ncu --set full capture per hot kernel (raw metrics + per-SASS-line export).
TAG=${1:-r2v}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" 2>&1 | tail -1
timeout 1800 python -m pytest tests -m gpu -q 2>&1 | tail -4 | tee gpurun_out/tests_$TAG.log
# compute-sanitizer: closed on this GPU pool from round 2 on ("runs under it
# have left GPUs needing a reset"); the last sanitizer evidence is
# profiles/r2/sanitizers_r2w.txt.  SANITIZE=1 runs it where it is allowed.
S=gpurun_out/sanitizers_$TAG.txt; : > $S
if [ -n "$SANITIZE" ]; then
for tool in memcheck racecheck synccheck; do
  echo "== compute-sanitizer --tool $tool --kernel-regex kns=hape python tools/sanitize_case.py" >> $S
  timeout 1200 compute-sanitizer --tool $tool --kernel-regex kns=hape python tools/sanitize_case.py 2>&1 | grep -E "SANITIZE|SUMMARY|Invalid|Race|error" | head -8 >> $S
done
for envv in HAPE_JN_SU=2 HAPE_JN_OA=1 HAPE_JN_LAY=1 HAPE_JN_LAY=2; do
  echo "== $envv compute-sanitizer --tool memcheck" >> $S
  env $envv timeout 900 compute-sanitizer --tool memcheck --kernel-regex kns=hape python tools/sanitize_case.py 2>&1 | grep -E "SANITIZE|SUMMARY|Invalid|error" | head -8 >> $S
done
fi
# the sanitizer case without the sanitizer (every kernel family, bag and unique layouts)
for envv in HAPE_JN_LAY=-1 HAPE_JN_LAY=0 HAPE_JN_LAY=1 HAPE_JN_LAY=2 HAPE_JN_SU=2; do
  echo "== $envv python tools/sanitize_case.py" >> $S
  env $envv timeout 600 python tools/sanitize_case.py 2>&1 | grep -E "SANITIZE|Error|error" | head -3 >> $S
done
cat $S
timeout 900 python bench.py > gpurun_out/bench_default_$TAG.json 2> gpurun_out/bench_default_$TAG.err
tail -1 gpurun_out/bench_default_$TAG.json | python tools/stages.py; python tools/legs.py gpurun_out/bench_default_$TAG.json
timeout 900 python bench.py --impl reference > gpurun_out/bench_reference_$TAG.json 2>&1; tail -1 gpurun_out/bench_reference_$TAG.json | head -c 300; echo
B="python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-ablation --no-coprocess --legs none"
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}_c2.csv $B > /dev/null 2>&1
for K in k_hist_joint:6 k_scatter:12 k_build_probe:3; do
  N=${K%%:*}; SK=${K##*:}
  R=gpurun_out/full_${TAG}_c2_${N}
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$N -s $SK -c 1 -o $R $B > /dev/null 2>&1
  ncu -i $R.ncu-rep --page raw --csv > $R.raw.csv 2>/dev/null
  ncu -i $R.ncu-rep --page source --csv --print-source sass 2>/dev/null | gzip > $R.sass.csv.gz
  rm -f $R.ncu-rep
done
# the fused exchange scatter (1-rank communicator) and the pass-2 scatter of the wide C4 plan
timeout 600 ncu --set full --clock-control none -k regex:k_scatter -s 6 -c 1 -o gpurun_out/full_${TAG}_x1_peer python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-ablation --no-coprocess --legs none --exchange > /dev/null 2>&1
ncu -i gpurun_out/full_${TAG}_x1_peer.ncu-rep --page raw --csv > gpurun_out/full_${TAG}_x1_peer.raw.csv 2>/dev/null; rm -f gpurun_out/full_${TAG}_x1_peer.ncu-rep
ls gpurun_out | grep $TAG
