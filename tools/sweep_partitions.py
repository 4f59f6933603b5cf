#!/usr/bin/env python
"""PAPER.md Fig. 5 on B200: build+probe time vs co-partition size (SURVEY §8.f
NEXT-4, "equal-partition SM sweep").

The paper's setup (P795-810): two tables of 32 M tuples, each a 4-byte key and
a 4-byte payload, loaded in GPU memory; the number of partitions varies, so the
input size is constant while the elements per partition vary; "we select the
keys so that all produced partitions have exactly the same size".  Here: dense
keys [0, 2^25) in a scrambled order (the c1 recipe at 2^25) with the identity
partition function (HAPE_PART_IDENTITY), so every co-partition holds exactly
2^25 / 2^(B1+B2) tuples of each table.  The partition count is set through
radix_bits; the table reports the build+probe stage (one launch of
k_build_probe: the scratchpad "SM" variant, the one the paper keeps) and the
whole join, and checks every result against the generator provenance.

    python tools/sweep_partitions.py [--log2n 25] [--steps 5] > profiles/<round>_fig5_sweep.jsonl
"""
from __future__ import annotations

import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--log2n", type=int, default=25)
    ap.add_argument("--steps", type=int, default=5)
    args = ap.parse_args()
    import torch
    import datagen
    from oracle import provenance
    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin

    n = 1 << args.log2n
    wl = datagen.make("c1", n_r=n, n_s=n, backend="torch", device="cuda")
    want = provenance.expected_pkfk(wl.R.payload[wl.idx].cpu().numpy(), wl.S.payload.cpu().numpy())
    args_ = (wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    for per_part_log2 in (8, 9, 10, 11, 12, 13):
        bits = args.log2n - per_part_log2
        b1 = (bits + 1) // 2
        b2 = bits - b1
        with RadixJoin(key_dtype=torch.int32, identity=True, radix_passes=2, radix_bits=(b1, b2),
                       r_unique=True, max_r=n, max_s=n) as j:
            for _ in range(2):
                res = j.join(*args_)
            ok = (res.match_count, res.sum_r_payload, res.sum_s_payload, res.pair_checksum) == \
                (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
            bp, tot = [], []
            for _ in range(args.steps):
                res = j.join(*args_)
                bp.append(res.stage_ms["build_probe"])
                tot.append(res.stage_ms["total"])
        bp.sort()
        tot.sort()
        print(json.dumps({"tuples_per_partition": 1 << per_part_log2, "partitions": 1 << bits,
                          "bits": [b1, b2], "build_probe_ms": round(bp[len(bp) // 2], 4),
                          "join_ms": round(tot[len(tot) // 2], 4), "n_per_table": n,
                          "verified_vs_provenance": ok}), flush=True)


if __name__ == "__main__":
    main()
