import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
"""Small joins for compute-sanitizer runs (memcheck / racecheck / synccheck):
int32 and int64, 1 and 2 passes, duplicates, materialisation, host inputs,
the 1-rank exchange path."""
import numpy as np
import torch

import datagen
import oracle
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin, _lib

d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
ok = True
for cfg, nr, ns, kw in [("c1", 5000, 7001, {}), ("c3", 3000, 20000, {}), ("dup", 4000, 3000, dict(dup_domain=40)),
                        ("c2", 1 << 16, 1 << 16, {})]:
    wl = datagen.make(cfg, n_r=nr, n_s=ns, **kw)
    kdt = torch.int32 if wl.key_bits == 32 else torch.int64
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    for passes, bits in ((1, (5, 0)), (2, (3, 3))):
        with RadixJoin(key_dtype=kdt, radix_passes=passes, radix_bits=bits) as j:
            n = want["count"]
            out_r = torch.empty(max(n, 1), dtype=kdt, device="cuda")
            out_s = torch.empty(max(n, 1), dtype=kdt, device="cuda")
            res = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload), out_r, out_s)
            got = (res.match_count, res.sum_r_payload, res.sum_s_payload, res.pair_checksum)
            ok &= got == (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
uid = _lib.hape_nccl_unique_id()
st, comm = _lib.hape_nccl_comm_init(uid, 1, 0, 0)
wl = datagen.make("c1", n_r=3000, n_s=4000)
want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
with RadixJoin(key_dtype=torch.int32, world_size=1, nccl_comm=comm) as j:
    res = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
    ok &= res.match_count == want["count"] and res.pair_checksum == want["checksum"]
pin = lambda a: torch.from_numpy(np.ascontiguousarray(a)).pin_memory()
with RadixJoin(key_dtype=torch.int32) as j:
    res = j.join(pin(wl.R.key), pin(wl.R.payload), pin(wl.S.key), pin(wl.S.payload))
    ok &= res.match_count == want["count"] and res.pair_checksum == want["checksum"]
# out-of-HBM co-processing: host co-partitioning + per-pair device joins
wl = datagen.make("c3", n_r=3000, n_s=20000)
want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
with RadixJoin(key_dtype=torch.int64) as j:
    out_r = torch.empty(want["count"], dtype=torch.int64).pin_memory()
    out_s = torch.empty(want["count"], dtype=torch.int64).pin_memory()
    res = j.coprocess_join(pin(wl.R.key), pin(wl.R.payload), pin(wl.S.key), pin(wl.S.payload), out_r, out_s,
                           fanout_bits=2)
    ok &= res.match_count == want["count"] and res.pair_checksum == want["checksum"]
_lib.hape_nccl_comm_destroy(comm)
print("SANITIZE_CASE_OK" if ok else "SANITIZE_CASE_MISMATCH")
