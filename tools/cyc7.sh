python -c "import __graft_entry__ as g; g.build()" 
for v in "HAPE_SLOT_EXTRA=1" "HAPE_SLOT_EXTRA=-1" "HAPE_CHUNK=16384" "HAPE_CHUNK=65536" "HAPE_JN_PF=0"; do for c in c2 c3; do echo "$v"; env $v timeout 300 python bench.py --config $c --no-e2e --no-cpu-baseline 2>&1 | tail -1 | python tools/stages.py; done; done
