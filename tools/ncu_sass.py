#!/usr/bin/env python
"""Print a kernel's SASS with executed-instruction counts and stall samples
from an ncu report (ncu -i X --page source --print-source sass)."""
import csv, subprocess, sys

rep = sys.argv[1]
minfrac = float(sys.argv[2]) if len(sys.argv) > 2 else 0.002
if rep.endswith(".sass.csv.gz"):  # exported on the GPU box by profile_round.sh
    import gzip
    out = gzip.open(rep, "rt").read()
else:
    out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                         capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
data = [dict(zip(h, r)) for r in rows[2:] if len(r) >= len(h) - 1]
def f(x):
    try: return float(x.replace(",", ""))
    except Exception: return 0.0
tot_i = sum(f(d["Instructions Executed"]) for d in data) or 1
tot_s = sum(f(d["Warp Stall Sampling (All Samples)"]) for d in data) or 1
print(f"total warp instructions {tot_i:.4g}, stall samples {tot_s:.4g}")
for d in data:
    ie, ss = f(d["Instructions Executed"]), f(d["Warp Stall Sampling (All Samples)"])
    if ie / tot_i >= minfrac or ss / tot_s >= minfrac:
        print(f"{100*ie/tot_i:5.1f}% {100*ss/tot_s:5.1f}%s  {d['Address'][-5:]}  {d['Source'].strip()[:90]}")

# histogram of execution counts: how many static instructions run how often
import collections
hist = collections.Counter()
for d in data:
    ie = f(d["Instructions Executed"])
    if ie > 0:
        b = round(ie / 1e5) * 1e5
        hist[b] += 1
print("exec-count buckets (count -> #static instrs, share of dynamic):")
for b, c in sorted(hist.items(), key=lambda x: -x[0] * x[1])[:12]:
    print(f"  {b:12.0f} x {c:4d} = {100*b*c/tot_i:5.1f}%")
