import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
"""Timing probe of the co-processing join's host step on the GPU box."""
import torch
import datagen
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin
wl = datagen.make("c2", backend="torch", device="cuda")
hk = [x.contiguous().cpu().pin_memory() for x in (wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)]
j = RadixJoin(key_dtype=torch.int32, r_unique=True)
for T in [int(x) for x in sys.argv[1:]] or [0]:
    for i in range(3):
        t = time.perf_counter()
        r = j.coprocess_join(*hk, fanout_bits=3, host_threads=T)
        print(f"T={T} call {i}: {1000*(time.perf_counter()-t):.1f} ms host_part {r.stage_ms['host_part']:.1f} h2d {r.stage_ms['h2d']:.1f}", flush=True)
