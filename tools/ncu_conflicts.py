#!/usr/bin/env python
"""Top shared-memory instructions by wavefronts / conflicts in an ncu report."""
import csv, subprocess, sys
rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
data = [dict(zip(h, r)) for r in rows[2:] if len(r) >= len(h) - 1]
f = lambda x: float((x or '0').replace(',', '') or 0)
items = [(f(d.get("L1 Wavefronts Shared", "0")), f(d.get("L1 Wavefronts Shared Ideal", "0")), f(d["Instructions Executed"]), i, d["Source"].strip()[:70]) for i, d in enumerate(data)]
items.sort(reverse=True)
for w, wi, ie, i, src in items[:25]:
    print(f"{i:5d} wavefronts {w/1e6:7.2f}M ideal {wi/1e6:7.2f}M  exec {ie/1e6:6.2f}M  {src}")
