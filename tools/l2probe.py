"""Per-tuple stage cost of the C2 recipe (8+8 bits) as the relations shrink
into the 126 MB L2: how much of pass 2 and build+probe is HBM time.
(developer probe; prints one JSON line per size)"""
import json, sys
sys.path.insert(0, '.')
import torch
import datagen
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin

s = torch.cuda.Stream()
torch.cuda.set_stream(s)
for lg in (20, 21, 22, 23, 24, 25, 27):
    n = 1 << lg
    wl = datagen.make("c2", n_r=n, n_s=n, backend="torch", device="cuda")
    j = RadixJoin(key_dtype=torch.int32, r_unique=True, stream=s, radix_passes=2, radix_bits=(8, 8))
    for _ in range(5):
        r = j.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    acc = {}
    N = 20
    for _ in range(N):
        r = j.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
        for k, v in r.stage_ms.items():
            acc[k] = acc.get(k, 0.0) + v / N
    ns = {k: round(v * 1e6 / (2 * n), 4) for k, v in acc.items() if v > 0}
    print(json.dumps({"log2n": lg, "bytes_MB": 2 * n * 8 / 1e6, "ns_per_tuple": ns,
                      "ms": {k: round(v, 4) for k, v in acc.items() if v > 0}}), flush=True)
    del j, wl
    torch.cuda.empty_cache()
