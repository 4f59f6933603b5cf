#!/usr/bin/env python
"""Summarise an ncu --csv launch list: per launch time and DRAM bytes."""
import collections, csv, sys
rows = list(csv.reader(open(sys.argv[1])))
last = int(sys.argv[2]) if len(sys.argv) > 2 else 20
hdr = None
data = collections.OrderedDict()
for r in rows:
    if len(r) > 10 and r[0] == 'ID':
        hdr = r; continue
    if hdr is None or len(r) < len(hdr):
        continue
    d = dict(zip(hdr, r))
    key = (int(d['ID']), d['Kernel Name'].split('(')[0][:40], d['Grid Size'])
    data.setdefault(key, {})[d['Metric Name']] = float(d['Metric Value'].replace(',', ''))
tot = 0
for (i, n, g), m in list(data.items())[-last:]:
    t = m.get('gpu__time_duration.sum', 0) / 1e3
    rd = m.get('dram__bytes_read.sum', 0) / 1e6
    wr = m.get('dram__bytes_write.sum', 0) / 1e6
    tot += t
    print(f"{i:4d} {n:40s} {g:>14s} {t:9.1f}us  rd {rd:8.1f}MB wr {wr:8.1f}MB  {(rd+wr)/max(t,1e-9):6.2f} TB/s")
print(f"sum {tot:.1f} us")
