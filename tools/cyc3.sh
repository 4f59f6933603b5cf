python -c "import __graft_entry__ as g; g.build()"
for c in c2 c3; do timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline 2>&1 | tail -1 | python tools/stages.py; done
