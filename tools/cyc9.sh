python -c "import __graft_entry__ as g; g.build()" 2>&1 | tail -2
mkdir -p gpurun_out
for c in c2 c3; do timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline > gpurun_out/bench9_$c.json 2>gpurun_out/bench9_$c.err; tail -1 gpurun_out/bench9_$c.json | python tools/stages.py; python -c "import json;d=json.loads(open('gpurun_out/bench9_$c.json').readlines()[-1]);print(d.get('nonpartitioned_gpu'))"; done
timeout 600 python tools/sweep_partitions.py > gpurun_out/fig5_sweep.jsonl 2>gpurun_out/fig5_sweep.err; cat gpurun_out/fig5_sweep.jsonl; tail -3 gpurun_out/fig5_sweep.err
