"""Summarise a bench.py JSON line from stdin: ms/step and per-stage ms / frac."""
import json
import sys

for line in sys.stdin:
    try:
        d = json.loads(line)
    except Exception:
        print("NOT JSON:", line[:300])
        continue
    st = d["roofline"]["stages"]
    print(d["config"]["workload"][:3], f"{d['ms_per_step']:.3f} ms", f"{d['value']/1e9:.1f} G/s",
          " ".join(f"{k}={v['ms']:.3f}({v.get('frac', 0):.2f})" for k, v in st.items()))
