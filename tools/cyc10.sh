python -c "import __graft_entry__ as g; g.build()" 2>&1 | tail -2
timeout 900 python -m pytest tests/test_gpu_nonpartitioned.py -x -q -m gpu 2>&1 | tail -2
for c in c2 c3; do timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline > gpurun_out/bench10_$c.json 2>gpurun_out/bench10_$c.err; tail -1 gpurun_out/bench10_$c.json | python tools/stages.py; python -c "import json;d=json.loads(open('gpurun_out/bench10_$c.json').readlines()[-1]);print(d.get('nonpartitioned_gpu'))"; done
