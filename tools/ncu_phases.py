#!/usr/bin/env python
"""Stall samples and executed instructions of a kernel's SASS in windows of
N instructions, with the memory/barrier opcodes of each window -- a coarse
'which phase stalls' view.  Usage: ncu_phases.py report [window]"""
import csv, subprocess, sys
rep = sys.argv[1]
win = int(sys.argv[2]) if len(sys.argv) > 2 else 20
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
hi = next(i for i, r in enumerate(rows) if r and r[0] == "Address")
h = rows[hi]
data = []
for r in rows[hi + 1:]:
    if r and r[0] == "Kernel Name":
        break
    if len(r) >= len(h) - 1:
        data.append(dict(zip(h, r)))
f = lambda x: float((x or '0').replace(',', '') or 0)
tot = sum(f(d["Warp Stall Sampling (All Samples)"]) for d in data) or 1
for i in range(0, len(data), win):
    w = data[i:i + win]
    ss = sum(f(d["Warp Stall Sampling (All Samples)"]) for d in w)
    ie = sum(f(d["Instructions Executed"]) for d in w)
    ops = set()
    for d in w:
        t = d["Source"].split()
        if not t:
            continue
        op = t[1] if t[0].startswith("@") and len(t) > 1 else t[0]
        if op.startswith(("LDS", "STS", "ATOMS", "LDG", "STG", "BAR", "SYNCS", "SHFL", "UBLK", "REDG", "ATOMG")):
            ops.add(op)
    if ss / tot > 0.01:
        print(f"{i:4d}-{i + win - 1:4d} stall {100 * ss / tot:5.1f}% inst {ie / 1e6:6.1f}M  {' '.join(sorted(ops))}")
