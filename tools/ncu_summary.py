#!/usr/bin/env python
"""Key metrics + top stall reasons of an ncu --set full report."""
import csv, subprocess, sys
for rep in sys.argv[1:]:
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    r = list(csv.reader(out.splitlines()))
    h, units, v = r[0], r[1], r[2]
    d = dict(zip(h, v))
    U = dict(zip(h, units))
    SCALE = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1, "usecond": 1e3,
             "msecond": 1e6, "second": 1e9, "ns": 1, "us": 1e3, "ms": 1e6}
    def g(k):
        try: return float(d[k].replace(",", "")) * SCALE.get(U.get(k, ""), 1)
        except Exception: return float("nan")
    dur = g("gpu__time_duration.sum")
    rd, wr = g("dram__bytes_read.sum"), g("dram__bytes_write.sum")
    print(f"== {rep}: {d.get('Kernel Name','')[:60]}")
    print(f"  duration {dur/1e3:.1f} us  dram rd {rd/1e6:.1f} MB wr {wr/1e6:.1f} MB  -> {(rd+wr)/dur:.2f} TB/s"
          f"  inst {g('smsp__inst_executed.sum')/1e6:.1f} M  ipc {g('sm__inst_executed.avg.per_cycle_active'):.2f}"
          f"  occ {g('sm__warps_active.avg.pct_of_peak_sustained_active'):.1f}%  regs {g('launch__registers_per_thread'):.0f}")
    print(f"  smem wavefronts {g('l1tex__data_pipe_lsu_wavefronts_mem_shared.sum')/1e6:.1f} M  bank conflicts "
          f"{g('l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum')/1e6:.1f} M  L2 wr sectors "
          f"{g('lts__t_sectors_srcunit_tex_op_write.sum')/1e6:.1f} M  L2 rd sectors {g('lts__t_sectors_srcunit_tex_op_read.sum')/1e6:.1f} M")
    st = sorted(((g(k), k) for k in h if k.startswith("smsp__average_warps_issue_stalled_") and k.endswith("_per_issue_active.ratio")), reverse=True)
    print("  stalls/issue: " + ", ".join(f"{k.split('stalled_')[1].split('_per_issue')[0]} {x:.2f}" for x, k in st[:7]))
