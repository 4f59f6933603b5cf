python -c "import __graft_entry__ as g; g.build(); g.smoke()" 2>&1 | tail -2
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -15
for c in c2 c3; do timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline 2>&1 | tail -1 | python tools/stages.py; done
