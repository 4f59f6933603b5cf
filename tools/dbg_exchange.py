import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
"""Debug: the 1-rank exchange path per config, printing progress (locates a crash)."""
import numpy as np
import torch
import datagen
import oracle
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin, _lib
d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
uid = _lib.hape_nccl_unique_id()
st, comm = _lib.hape_nccl_comm_init(uid, 1, 0, 0)
print("comm", st, flush=True)
for cfg, nr, ns in [(a, int(b), int(c)) for a, b, c in (x.split(":") for x in sys.argv[1:])]:
    kw = dict(dup_domain=50) if cfg == "dup" else {}
    wl = datagen.make(cfg, n_r=nr, n_s=ns, **kw)
    kdt = torch.int32 if wl.key_bits == 32 else torch.int64
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    print(cfg, "joining", flush=True)
    with RadixJoin(key_dtype=kdt, world_size=1, rank=0, nccl_comm=comm) as j:
        res = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
    print(cfg, "ok" if res.match_count == want["count"] and res.pair_checksum == want["checksum"] else "MISMATCH", flush=True)
_lib.hape_nccl_comm_destroy(comm)
