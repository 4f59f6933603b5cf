"""Full-size parity of BASELINE configs[3] (C4: |R| = |S| = 2^31 int32, on one
B200) and configs[4] (C5: |R| = 2^28, |S| = 2^30, Zipf theta = 1), in the
launch configuration bench.py times (its handle options, HAPE_FLAG_R_UNIQUE,
the same workspace), against generator provenance: for the
PK-FK recipes every S row j joins exactly R row idx[j], so

    count = |S|,  sum_s = sum_j q_j,  sum_r = sum_j p_idx[j],
    pair_checksum = sum_j mix(p_idx[j], q_j)          (all mod 2^64)

computed on the host by oracle.provenance (numpy), chunk by chunk.  The
relations are generated on the GPU by datagen (the shared input module) and
copied to the host for the oracle side.  C4 is exactly the 2^31 per-relation
size the uint32 tuple indices of the path must carry (n < 2^32 per rank).
"""
import numpy as np
import pytest
import torch

import datagen
from oracle import provenance

pytestmark = [pytest.mark.gpu, pytest.mark.slow]

if torch.cuda.is_available():
    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin

M64 = (1 << 64) - 1
CHUNK = 1 << 27


def _gen(cfg, n_r, n_s, **kw):
    """Device columns of the whole relation, generated chunk by chunk (the
    same sub-shard composition bench.py uses) plus the host R payload column
    and a generator of (idx, S payload) host chunks for the provenance."""
    k = max(1, -(-max(n_r, n_s) // CHUNK))
    first = datagen.make(cfg, n_r=n_r, n_s=n_s, rank=0, world=k, backend="torch", device="cuda", **kw)
    cols = [torch.empty(n_r, dtype=first.R.key.dtype, device="cuda"),
            torch.empty(n_r, dtype=first.R.payload.dtype, device="cuda"),
            torch.empty(n_s, dtype=first.S.key.dtype, device="cuda"),
            torch.empty(n_s, dtype=first.S.payload.dtype, device="cuda")]
    idx_chunks = []
    pr = ps = 0
    for j in range(k):
        wl = first if j == 0 else datagen.make(cfg, n_r=n_r, n_s=n_s, rank=j, world=k, backend="torch",
                                               device="cuda", **kw)
        a, b = wl.R.n, wl.S.n
        cols[0][pr:pr + a] = wl.R.key
        cols[1][pr:pr + a] = wl.R.payload
        cols[2][ps:ps + b] = wl.S.key
        cols[3][ps:ps + b] = wl.S.payload
        idx_chunks.append((ps, wl.idx.cpu().numpy()))
        pr, ps = pr + a, ps + b
        del wl
    assert pr == n_r and ps == n_s
    return cols, idx_chunks


def _expected(cols, idx_chunks):
    rp_host = cols[1].cpu().numpy()
    tot = dict(count=0, sum_r=0, sum_s=0, checksum=0)
    for ps, idx in idx_chunks:
        sp = cols[3][ps:ps + len(idx)].cpu().numpy()
        e = provenance.expected_pkfk(rp_host[idx], sp)
        for f in tot:
            tot[f] = (tot[f] + e[f]) & M64
    return tot


def _run(cols, dt):
    rk, rp, sk, sp = cols
    j = RadixJoin(key_dtype=dt, r_payload_dtype=dt, s_payload_dtype=dt, max_r=rk.shape[0], max_s=sk.shape[0],
                  r_unique=True, stream=torch.cuda.current_stream())
    res = j.join(rk, rp, sk, sp)
    res2 = j.join(rk, rp, sk, sp)          # graph replay, same workspace
    j.close()
    assert res2.as_tuple() == res.as_tuple()
    return res


def test_c4_full_size_one_gpu_vs_provenance():
    n = 1 << 31
    cols, idx_chunks = _gen("c4", n, n)
    res = _run(cols, torch.int32)
    want = _expected(cols, idx_chunks)
    got = dict(count=res.match_count, sum_r=res.sum_r_payload, sum_s=res.sum_s_payload, checksum=res.pair_checksum)
    assert got == want
    assert res.r_local == n and res.s_local == n and res.passes == 2
    del cols
    torch.cuda.empty_cache()


def test_c5_full_size_zipf_vs_provenance():
    n_r, n_s = 1 << 28, 1 << 30
    cols, idx_chunks = _gen("c5", n_r, n_s, theta=1.0)
    # the skew is real: the hottest R row is copied by > 4% of S
    top = max(int(np.bincount(idx, minlength=n_r).max()) for _, idx in idx_chunks[:1])
    assert top > 0.04 * len(idx_chunks[0][1])
    res = _run(cols, torch.int32)
    want = _expected(cols, idx_chunks)
    got = dict(count=res.match_count, sum_r=res.sum_r_payload, sum_s=res.sum_s_payload, checksum=res.pair_checksum)
    assert got == want
    del cols
    torch.cuda.empty_cache()
