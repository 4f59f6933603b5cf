python -c "import __graft_entry__ as g; g.build(); g.smoke()" 2>&1 | tail -1
timeout 600 python -m pytest tests/test_gpu_join.py -x -q -m gpu -k "random_small or recipes or partition or joint or skew" 2>&1 | tail -2
for sc in 0 1; do for c in c2 c3; do echo "SC=$sc"; HAPE_SC=$sc timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline 2>&1 | tail -1 | python tools/stages.py; done; done
