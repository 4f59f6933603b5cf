#!/usr/bin/env python
"""Summarise a round's profiling artefacts (tools/profile_round.sh) into
profiles/: the per-launch ncu list of one bench step, the per-kernel
--set full metrics, and profiles/ncu_traffic.json (dram read+write per bench
stage, consumed by bench.py's roofline.traffic)."""
import collections
import csv
import json
import os
import subprocess
import sys

TAG, CFG = sys.argv[1], sys.argv[2]
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
G = os.path.join(ROOT, "gpurun_out")
P = os.path.join(ROOT, "profiles")
os.makedirs(P, exist_ok=True)


def launches():
    rows = list(csv.reader(open(os.path.join(G, f"launches_{TAG}_{CFG}.csv"))))
    hdr = None
    data = collections.OrderedDict()
    for r in rows:
        if len(r) > 10 and r[0] == "ID":
            hdr = r
            continue
        if hdr is None or len(r) < len(hdr):
            continue
        d = dict(zip(hdr, r))
        key = (int(d["ID"]), d["Kernel Name"].split("(")[0].replace("void ", ""), d["Grid Size"], d["Block Size"])
        unit = d["Metric Unit"]
        scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1, "usecond": 1e3, "msecond": 1e6}.get(unit, 1)
        data.setdefault(key, {})[d["Metric Name"]] = float(d["Metric Value"].replace(",", "")) * scale
    return data


def full_metrics(path):
    if path.endswith(".csv"):  # raw page exported on the GPU box (profile_round.sh)
        out = open(path).read()
    else:
        out = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    r = list(csv.reader(out.splitlines()))
    res = []
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1, "usecond": 1e3, "msecond": 1e6, "ns": 1, "us": 1e3, "ms": 1e6,
             "second": 1e9}
    for row in r[2:]:
        d = dict(zip(r[0], row))
        u = dict(zip(r[0], r[1]))

        def g(k):
            try:
                return float(d[k].replace(",", "")) * scale.get(u.get(k, ""), 1)
            except Exception:
                return float("nan")
        stalls = sorted(((g(k), k.split("stalled_")[1].split("_per_issue")[0]) for k in r[0]
                         if k.startswith("smsp__average_warps_issue_stalled_") and k.endswith("_per_issue_active.ratio")),
                        reverse=True)[:5]
        res.append(dict(kernel=d.get("Kernel Name", "")[:90], grid=d.get("Grid Size"), block=d.get("Block Size"),
                        ns=g("gpu__time_duration.sum"), rd=g("dram__bytes_read.sum"), wr=g("dram__bytes_write.sum"),
                        inst=g("smsp__inst_executed.sum"), ipc=g("sm__inst_executed.avg.per_cycle_active"),
                        occ=g("sm__warps_active.avg.pct_of_peak_sustained_active"),
                        regs=g("launch__registers_per_thread"),
                        smem_wf=g("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum"),
                        l1pct=g("l1tex__throughput.avg.pct_of_peak_sustained_elapsed"),
                        drampct=g("gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed"),
                        stalls=[f"{n} {v:.2f}" for v, n in stalls]))
    return res


L = launches()
items = list(L.items())
# the profiled step = the launches after the previous step's build+probe up
# to the last build+probe (ablation kernels after it are not part of a step)
bps = [k for k, ((i, n, g, b), m) in enumerate(items) if "k_build_probe" in n]
if len(bps) >= 2:
    step = items[bps[-2] + 1: bps[-1] + 1]
else:
    per_step = {"c1": 8, "c2": 14, "c3": 14}.get(CFG, 14)
    step = items[-per_step:]
lines = [f"# ncu summary {TAG} / {CFG}\n",
         "Per-launch list of ONE bench step (`ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,"
         "dram__bytes_write.sum --clock-control none`): cold-cache, serialised launches -- compare shares, "
         "not absolutes.\n",
         "| # | kernel | grid | us | DRAM rd MB | DRAM wr MB | TB/s | share |", "|---|---|---|---|---|---|---|---|"]
tot = sum(m.get("gpu__time_duration.sum", 0) for _, m in step)
for (i, n, g, b), m in step:
    t = m.get("gpu__time_duration.sum", 0)
    rd, wr = m.get("dram__bytes_read.sum", 0), m.get("dram__bytes_write.sum", 0)
    lines.append(f"| {i} | {n} | {g} | {t/1e3:.1f} | {rd/1e6:.1f} | {wr/1e6:.1f} | {(rd+wr)/max(t,1):.2f} | {100*t/max(tot,1):.1f}% |")
lines.append(f"\nStep total (serialised): {tot/1e3:.1f} us\n")
traffic = {}
lines.append("## --set full captures (per launch)\n")
lines.append("| kernel | us | DRAM rd+wr MB | TB/s | warp inst M | IPC | occ % | regs | smem wavefronts M | L1 % | DRAM % | top stalls |")
lines.append("|---|---|---|---|---|---|---|---|---|---|---|---|")
for name in ("k_hist", "k_hist_joint", "k_scatter", "k_build_probe"):
    path = os.path.join(G, f"full_{TAG}_{CFG}_{name}.ncu-rep")
    if not os.path.exists(path):
        path = os.path.join(G, f"full_{TAG}_{CFG}_{name}.raw.csv")
    if not os.path.exists(path):
        continue
    for m in full_metrics(path):
        lines.append(f"| {m['kernel']} | {m['ns']/1e3:.1f} | {(m['rd']+m['wr'])/1e6:.1f} | {(m['rd']+m['wr'])/m['ns']:.2f} | "
                     f"{m['inst']/1e6:.1f} | {m['ipc']:.2f} | {m['occ']:.1f} | {m['regs']:.0f} | {m['smem_wf']/1e6:.1f} | "
                     f"{m['l1pct']:.1f} | {m['drampct']:.1f} | {'; '.join(m['stalls'])} |")
# traffic per bench stage from the launch list (sum of the stage's launches)
names = [(n, (m.get("dram__bytes_read.sum", 0) + m.get("dram__bytes_write.sum", 0))) for (i, n, g, b), m in step]
stage_of = []
hist_seen = scatter_seen = 0
for n, by in names:
    if "k_hist" in n:
        st = "hist1" if hist_seen < 2 else "hist2"; hist_seen += 1
    elif "k_scatter" in n:
        st = "scatter1" if scatter_seen < 2 else "scatter2"; scatter_seen += 1
    elif "k_build_probe" in n:
        st = "build_probe"
    else:
        continue
    traffic[st] = traffic.get(st, 0) + int(by)
tj = os.path.join(P, "ncu_traffic.json")
allt = json.load(open(tj)) if os.path.exists(tj) else {}
allt[CFG] = traffic
allt["_note"] = ("dram__bytes_read.sum + dram__bytes_write.sum per bench stage (sum over the stage's launches, "
                 "R and S), from the ncu launch list of one step; same unit as roofline.achieved's stage bytes")
json.dump(allt, open(tj, "w"), indent=1)
open(os.path.join(P, f"{TAG}_{CFG}_ncu_summary.md"), "w").write("\n".join(lines) + "\n")
# trimmed launch csv of the profiled step
src = os.path.join(G, f"launches_{TAG}_{CFG}.csv")
ids = {str(i) for (i, n, g, b), m in step}
with open(src) as f, open(os.path.join(P, f"{TAG}_{CFG}_launches.csv"), "w") as o:
    for line in f:
        cells = line.split('","')
        if line.startswith('"ID"') or (cells and cells[0].strip('"') in ids):
            o.write(line)
bj = os.path.join(G, f"bench_{TAG}_{CFG}.json")
if os.path.exists(bj):
    txt = open(bj).read().strip().splitlines()
    if txt:
        open(os.path.join(P, f"{TAG}_{CFG}_bench.json"), "w").write(txt[-1] + "\n")
print("\n".join(lines))
print(json.dumps(traffic))
