"""Expected join results from generator provenance -- TEST INFRASTRUCTURE ONLY.

For the PK-FK recipes of datagen (unique R keys, every S row j copying the key
of R row idx[j]), every S tuple matches exactly one R tuple, so the join bag
of PAPER.md P789-794 is J = {(p_idx[j], q_j)}_j and:
  count         = |S|                      (P793-794: "as many tuples as any
                                            of the inputs")
  sum_s         = sum_j q_j                (a column reduction, no join)
  sum_r         = sum_j p_{idx[j]}         (gather + reduce, no join)
  pair_checksum = sum_j mix(p_{idx[j]}, q_j)
This is a different computation from oracle.c's sort-merge; tests pin the two
against each other on small sizes, and GPU tests use it at full size.
"""
from __future__ import annotations

import numpy as np

from . import mix, u64sum


def expected_pkfk(r_pay_of_idx: np.ndarray, s_pay: np.ndarray, materialize: bool = False) -> dict:
    """r_pay_of_idx[j] = payload of the R row S row j joins with."""
    rp = np.asarray(r_pay_of_idx)
    sp = np.asarray(s_pay)
    res = dict(count=int(sp.shape[0]), sum_r=u64sum(rp), sum_s=u64sum(sp),
               checksum=u64sum(mix(rp, sp)))
    if materialize:
        a = rp.astype(np.int64)
        b = sp.astype(np.int64)
        order = np.lexsort((b, a))
        res["pairs"] = (a[order], b[order])
    return res


def expected_from_workload(wl, r_payload_global=None) -> dict:
    """Expected result for a datagen.Workload of kind pkfk-dense / fk-uniform /
    zipf generated with world=1 (idx are global R rows)."""
    idx = wl.idx
    if hasattr(idx, "cpu"):
        idx = idx.cpu().numpy()
    rp = wl.R.payload if r_payload_global is None else r_payload_global
    if hasattr(rp, "cpu"):
        rp = rp.cpu().numpy()
    sp = wl.S.payload
    if hasattr(sp, "cpu"):
        sp = sp.cpu().numpy()
    return expected_pkfk(np.asarray(rp)[np.asarray(idx).astype(np.int64)], sp)
