import os, sys, time, ctypes
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
"""Host partitioning throughput into pageable vs pinned outputs (co-processing host step)."""
import torch
from paper_conf_cidr_chrysogelossa19_b200 import _lib
n = 1 << 27
k = torch.randint(-2**31, 2**31, (n,), dtype=torch.int32)
p = torch.randint(-2**31, 2**31, (n,), dtype=torch.int32)
for kind in ("pageable", "pinned"):
    ok, op = torch.empty(n, dtype=torch.int32), torch.empty(n, dtype=torch.int32)
    if kind == "pinned":
        ok, op = ok.pin_memory(), op.pin_memory()
    ok.fill_(0); op.fill_(0)
    rel = _lib.hape_relation(k.data_ptr(), p.data_ptr(), n, _lib.HAPE_MEM_HOST)
    b = (ctypes.c_uint64 * 9)()
    for T in (16, 8, 16, 4):
        ts = []
        for i in range(3):
            t = time.perf_counter()
            _lib.hape_host_partition(rel, 0, 0, 0, 3, T, ok.data_ptr(), op.data_ptr(), b)
            ts.append(1000 * (time.perf_counter() - t))
        print(kind, "T", T, " ".join(f"{x:.1f}" for x in ts), "ms", flush=True)
