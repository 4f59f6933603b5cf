"""GPU parity of the out-of-HBM co-processing join (hape_coprocess_join,
PAPER.md §5 P717-737, Fig. 7) against the CPU oracle: host-resident inputs,
CPU-side co-partitioning, one transfer per co-partition pair, the device radix
join per pair.  Integer results: bit-exact count / sums / checksum and the
sorted pair multiset.  Small device budgets force many co-partitions and the
S-slicing path.
"""
import numpy as np
import pytest
import torch

import datagen
import oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_conf_cidr_chrysogelossa19_b200 import HapeError, RadixJoin, _lib

DT = {np.dtype(np.int32): torch.int32, np.dtype(np.int64): torch.int64}


def host(a):
    return torch.from_numpy(np.ascontiguousarray(a)).pin_memory()


def check(res, want):
    got = dict(count=res.match_count, sum_r=res.sum_r_payload, sum_s=res.sum_s_payload,
               checksum=res.pair_checksum)
    assert got == {k: want[k] for k in got}, (got, want)


def sorted_pairs(a, b):
    a = a.cpu().numpy().astype(np.int64)
    b = b.cpu().numpy().astype(np.int64)
    o = np.lexsort((b, a))
    return a[o], b[o]


@pytest.mark.parametrize("seed", range(12))
def test_coprocess_random_vs_oracle(seed):
    rng = np.random.default_rng(700 + seed)
    kdt = [np.int32, np.int64][seed % 2]
    pdt = [np.int32, np.int64][(seed // 2) % 2]
    nr = int(rng.choice([1, 1000, 70001, 300000]))
    ns = int(rng.choice([1, 999, 65537, 400000]))
    dom = int(rng.choice([7, 5000, 1 << 30]))
    rk = (rng.integers(0, dom, nr) - dom // 2).astype(kdt)
    sk = (rng.integers(0, dom, ns) - dom // 2).astype(kdt)
    if nr * ns / dom > 3e6:
        sk = sk[: max(1, int(3e6 * dom / nr))]
    rp = rng.integers(-2**31, 2**31, nr).astype(pdt)
    sp = rng.integers(-2**31, 2**31, len(sk)).astype(pdt)
    want = oracle.join(rk, rp, sk, sp, materialize=True)
    fb = int(rng.choice([0, 1, 3, 6]))
    j = RadixJoin(key_dtype=DT[np.dtype(kdt)], r_payload_dtype=DT[np.dtype(pdt)], s_payload_dtype=DT[np.dtype(pdt)])
    n = want["count"]
    out_r = torch.empty(max(n, 1), dtype=DT[np.dtype(pdt)]).pin_memory()
    out_s = torch.empty(max(n, 1), dtype=DT[np.dtype(pdt)]).pin_memory()
    res = j.coprocess_join(host(rk), host(rp), host(sk), host(sp), out_r, out_s, fanout_bits=fb,
                           host_threads=int(rng.choice([0, 1, 5])))
    check(res, want)
    assert res.n_written == n and res.n_partitions == 1 << fb
    gr, gs = sorted_pairs(out_r[:n], out_s[:n])
    assert np.array_equal(gr, want["pairs"][0]) and np.array_equal(gs, want["pairs"][1])
    j.close()


def test_coprocess_small_budget_slices_s_and_matches_pkfk():
    """|R| = 2^18 unique keys, |S| = 2^20 FK (C3 recipe shape, int64): a
    budget of ~24 MB forces several co-partitions and S slicing per pair."""
    wl = datagen.make("c3", n_r=1 << 18, n_s=1 << 20)
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)
    j = RadixJoin(key_dtype=torch.int64, r_unique=True)
    out_r = torch.empty(want["count"], dtype=torch.int64, device="cuda")
    out_s = torch.empty(want["count"], dtype=torch.int64, device="cuda")
    res = j.coprocess_join(host(wl.R.key), host(wl.R.payload), host(wl.S.key), host(wl.S.payload), out_r, out_s,
                           device_budget=(64 << 20) + (24 << 20))
    check(res, want)
    assert res.n_partitions > 1
    assert res.stage_ms["host_part"] > 0 and res.stage_ms["h2d"] > 0
    gr, gs = sorted_pairs(out_r, out_s)
    assert np.array_equal(gr, want["pairs"][0]) and np.array_equal(gs, want["pairs"][1])
    j.close()


def test_coprocess_zipf_skew_vs_oracle():
    wl = datagen.make("c5", n_r=1 << 16, n_s=1 << 19)
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    kd = DT[np.dtype(wl.R.key.dtype)]
    j = RadixJoin(key_dtype=kd, r_payload_dtype=DT[np.dtype(wl.R.payload.dtype)],
                  s_payload_dtype=DT[np.dtype(wl.S.payload.dtype)], r_unique=True)
    res = j.coprocess_join(host(wl.R.key), host(wl.R.payload), host(wl.S.key), host(wl.S.payload),
                           device_budget=(64 << 20) + (4 << 20))
    check(res, want)
    j.close()


def test_coprocess_capacity_and_empty():
    rng = np.random.default_rng(5)
    rk = rng.permutation(1 << 16).astype(np.int32)
    sk = rng.integers(0, 1 << 16, 1 << 17).astype(np.int32)
    rp, sp = rk * 3, sk + 1
    want = oracle.join(rk, rp, sk, sp)
    j = RadixJoin(key_dtype=torch.int32)
    cap = want["count"] // 3
    out_r = torch.empty(cap, dtype=torch.int32).pin_memory()
    out_s = torch.empty(cap, dtype=torch.int32).pin_memory()
    with pytest.raises(HapeError):
        j.coprocess_join(host(rk), host(rp), host(sk), host(sp), out_r, out_s, fanout_bits=2)
    res = j.coprocess_join(host(rk), host(rp), host(sk), host(sp), out_r, out_s, fanout_bits=2,
                           raise_on_capacity=False)
    assert res.status == _lib.HAPE_ERR_OUTPUT_CAPACITY
    check(res, want)
    assert res.n_written == cap and res.n_required == want["count"]
    e = np.zeros(0, np.int32)
    res = j.coprocess_join(host(e), host(e), host(sk), host(sp), fanout_bits=3)
    assert res.match_count == 0
    # device-resident inputs are rejected (the entry is for host-resident data)
    with pytest.raises(HapeError):
        j.coprocess_join(torch.from_numpy(rk).cuda(), torch.from_numpy(rp).cuda(), host(sk), host(sp))
    j.close()
