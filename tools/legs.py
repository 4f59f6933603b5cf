"""Summarise the `legs` of a bench.py JSON line (file argument or stdin)."""
import json
import sys

src = open(sys.argv[1]) if len(sys.argv) > 1 else sys.stdin
d = json.loads(src.read().strip().splitlines()[-1])
for k, v in d.get("legs", {}).items():
    if isinstance(v, dict) and "roofline" in v:
        st = v["roofline"]["stages"]
        print(k, v["ms_per_step"], round(v["value"] / 1e9, 1), v["bits"], v.get("count_ok"),
              " ".join(f"{s}={x['ms']:.3f}({x['frac']:.2f})" for s, x in st.items()))
    else:
        print(k, v)
