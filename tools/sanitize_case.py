import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
"""Small joins for compute-sanitizer runs (memcheck / racecheck / synccheck):
int32 and int64, 1 and 2 passes, duplicates, materialisation, host inputs,
the 1-rank exchange path (fused peer scatter), the linked-buffer pass 1,
the loopback G>1 path in both exchange forms, the wide-plan claiming path."""
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
    for passes, bits, linked in ((1, (5, 0), False), (2, (3, 3), False), (2, (3, 3), True), (2, (9, 9), False)):
        with RadixJoin(key_dtype=kdt, radix_passes=passes, radix_bits=bits, linked=linked) as j:
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
# G simulated ranks on this GPU, both exchange forms
wl = datagen.make("dup", n_r=6000, n_s=7000, dup_domain=97)
want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
with RadixJoin(key_dtype=torch.int32) as j:
    for peer in (False, True):
        cut = [0, 1000, 3000, 6000]
        cs = [0, 3500, 3500, 7000]
        r_sh = [(d(wl.R.key[cut[g]:cut[g + 1]]), d(wl.R.payload[cut[g]:cut[g + 1]])) for g in range(2)] + \
            [(d(wl.R.key[3000:6000]), d(wl.R.payload[3000:6000])), (d(wl.R.key[:0]), d(wl.R.payload[:0]))]
        s_sh = [(d(wl.S.key[cs[g]:cs[g + 1]]), d(wl.S.payload[cs[g]:cs[g + 1]])) for g in range(3)] + \
            [(d(wl.S.key[:0]), d(wl.S.payload[:0]))]
        tot, _ = j.loopback_join(r_sh, s_sh, peer=peer)
        ok &= tot.as_tuple() == (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
_lib.hape_nccl_comm_destroy(comm)
print("SANITIZE_CASE_OK" if ok else "SANITIZE_CASE_MISMATCH")
