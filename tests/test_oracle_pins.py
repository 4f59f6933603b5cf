"""Pins for the CPU oracle (-m "not gpu").

Each test checks oracle/ against something other than itself: published hash
vectors, a hand-derived worked example, brute force on tiny inputs, closed
forms, a numpy library routine of a different family, and the generator's
provenance.  A dropped term, a wrong sign-extension, a swapped operand in
mix(p, q) or a missed duplicate run fails at least one of them.
"""
import collections
import json
import os

import numpy as np
import pytest

import datagen
import oracle
from oracle import partition, provenance

M64 = (1 << 64) - 1


# ---- independent python-int restatements used only by the brute force ----
def _py_fmix64(x):
    x &= M64
    x ^= x >> 30; x = (x * 0xBF58476D1CE4E5B9) & M64
    x ^= x >> 27; x = (x * 0x94D049BB133111EB) & M64
    return x ^ (x >> 31)


def _py_mix(p, q):
    return _py_fmix64((p & M64) * 0x9E3779B97F4A7C15 + (q & M64))


def brute(rk, rp, sk, sp):
    """Nested loops over all |R|*|S| tuple pairs (the definition, P789-794)."""
    cnt = sr = ss = sx = 0
    pairs = []
    for a in range(len(rk)):
        for b in range(len(sk)):
            if int(rk[a]) == int(sk[b]):
                p, q = int(rp[a]), int(sp[b])
                cnt += 1
                sr += p
                ss += q
                sx += _py_mix(p, q)
                pairs.append((p, q))
    pairs.sort()
    return dict(count=cnt, sum_r=sr & M64, sum_s=ss & M64, checksum=sx & M64), pairs


# ------------------------------------------------------------------------
def test_splitmix64_published_vectors(golden_dir):
    g = json.load(open(os.path.join(golden_dir, "hash_vectors.json")))
    want = [int(v, 16) for v in g["splitmix64_seed0"]]
    states = [(k * 0x9E3779B97F4A7C15) & M64 for k in (1, 2, 3)]
    assert [oracle.fmix64_scalar(s) for s in states] == want
    assert [int(v) for v in oracle.fmix64(np.array(states, np.uint64))] == want
    assert [int(v) for v in partition.fmix64(np.array(states, np.uint64).view(np.int64))] == want
    assert [_py_fmix64(s) for s in states] == want


def test_murmur3_fmix32_published_vectors(golden_dir):
    g = json.load(open(os.path.join(golden_dir, "hash_vectors.json")))
    for seed, want in g["murmur3_x86_32_empty"].items():
        k = np.array([int(seed, 16)], np.uint32).view(np.int32)
        assert int(partition.fmix32(k)[0]) == int(want, 16)


def test_mix_pinned_by_published_splitmix64(golden_dir):
    """The pair-checksum term itself (not a restatement of it): with
    mix(p, q) = fmix64(p*phi + q) (R10), mix(k, 0) = fmix64(k*phi)
    is the k-th published splitmix64 seed-0 output, and so is
    mix(k - 1, phi as int64) -- pinning the multiplier and the additive q
    term (a dropped term, a swapped operand or a missing sign extension of q
    breaks one of the two)."""
    g = json.load(open(os.path.join(golden_dir, "hash_vectors.json")))
    want = [int(v, 16) for v in g["splitmix64_seed0"]]
    phi_i64 = 0x9E3779B97F4A7C15 - (1 << 64)          # negative as int64: sign extension matters
    for k, w in zip((1, 2, 3), want):
        assert oracle.mix_scalar(k, 0) == w
        assert oracle.mix_scalar(k - 1, phi_i64) == w
        assert int(oracle.mix(np.array([k], np.int64), np.array([0], np.int64))[0]) == w
        assert int(oracle.mix(np.array([k - 1], np.int64), np.array([phi_i64], np.int64))[0]) == w
        # 32-bit payloads: p = k fits; the q term through a sign-extended int32
    assert int(oracle.mix(np.array([1], np.int32), np.array([0], np.int32))[0]) == want[0]


def test_mix_orientation_and_sign_extension():
    # mix is orientation-sensitive and sign-extends 32-bit payloads
    assert oracle.mix_scalar(1, 2) != oracle.mix_scalar(2, 1)
    a = oracle.mix(np.array([-1], np.int32), np.array([5], np.int32))[0]
    b = oracle.mix(np.array([-1], np.int64), np.array([5], np.int64))[0]
    assert int(a) == int(b) == _py_mix(-1, 5) == oracle.mix_scalar(-1, 5)


def test_golden_worked_example(golden_dir):
    g = json.load(open(os.path.join(golden_dir, "tiny_join.json")))
    for kdt, pdt in ((np.int32, np.int32), (np.int64, np.int64), (np.int32, np.int64)):
        rk = np.array(g["R"]["key"], kdt); rp = np.array(g["R"]["payload"], pdt)
        sk = np.array(g["S"]["key"], kdt); sp = np.array(g["S"]["payload"], pdt)
        res = oracle.join(rk, rp, sk, sp, materialize=True)
        assert res["count"] == g["count"]
        assert res["sum_r"] == g["sum_r"] & M64
        assert res["sum_s"] == g["sum_s"] & M64
        pairs = list(zip(res["pairs"][0].tolist(), res["pairs"][1].tolist()))
        assert pairs == [tuple(x) for x in g["pairs_sorted"]]
        assert res["checksum"] == sum(_py_mix(p, q) for p, q in g["pairs_sorted"]) & M64


@pytest.mark.parametrize("seed", range(200))
def test_oracle_vs_bruteforce(seed):
    rng = np.random.default_rng(seed)
    kdt = np.int32 if seed % 2 == 0 else np.int64
    rpdt = [np.int32, np.int64][(seed // 2) % 2]
    spdt = [np.int32, np.int64][(seed // 4) % 2]
    nr = int(rng.integers(0, 64 if seed % 7 else 300))
    ns = int(rng.integers(0, 64 if seed % 5 else 300))
    dom = int(rng.choice([1, 2, 16, 1000]))
    ext = np.iinfo(kdt)
    if seed % 3 == 0:  # extreme and negative keys
        pool = np.array([ext.min, ext.max, -1, 0, 1, ext.min + 1, 7][: max(1, min(dom, 7))], kdt)
        rk = rng.choice(pool, nr).astype(kdt); sk = rng.choice(pool, ns).astype(kdt)
    else:
        rk = rng.integers(-dom // 2, dom - dom // 2, nr).astype(kdt) if dom > 1 else np.zeros(nr, kdt)
        sk = rng.integers(-dom // 2, dom - dom // 2, ns).astype(kdt) if dom > 1 else np.zeros(ns, kdt)
    rp = rng.integers(np.iinfo(rpdt).min, np.iinfo(rpdt).max, nr, dtype=rpdt, endpoint=True)
    sp = rng.integers(np.iinfo(spdt).min, np.iinfo(spdt).max, ns, dtype=spdt, endpoint=True)
    want, pairs = brute(rk, rp, sk, sp)
    got = oracle.join(rk, rp, sk, sp, materialize=True)
    assert {k: got[k] for k in want} == want
    assert list(zip(got["pairs"][0].tolist(), got["pairs"][1].tolist())) == pairs


def test_closed_forms():
    rng = np.random.default_rng(7)
    n = 5000
    keys = rng.permutation(n).astype(np.int32)
    pay = rng.integers(-2**31, 2**31, n).astype(np.int32)
    # same key set (P793-794): count = N
    perm = rng.permutation(n)
    r = oracle.join(keys, pay, keys[perm], pay[perm] ^ 5)
    assert r["count"] == n
    # PK-FK: count = N_S
    fk = rng.integers(0, n, 3 * n)
    r = oracle.join(keys, pay, keys[fk], pay[fk % n])
    assert r["count"] == 3 * n
    # disjoint -> 0
    r = oracle.join(keys, pay, keys + n, pay)
    assert r == dict(count=0, sum_r=0, sum_s=0, checksum=0)
    # empty sides -> 0
    e = np.zeros(0, np.int32)
    assert oracle.join(e, e, keys, pay)["count"] == 0
    assert oracle.join(keys, pay, e, e)["count"] == 0
    # all-equal keys: a*b pairs, sum_r = b*sum(p), sum_s = a*sum(q)
    a, b = 300, 200
    rp = rng.integers(-1000, 1000, a).astype(np.int64)
    sp = rng.integers(-1000, 1000, b).astype(np.int64)
    r = oracle.join(np.full(a, -9, np.int64), rp, np.full(b, -9, np.int64), sp)
    assert r["count"] == a * b
    assert r["sum_r"] == (b * int(rp.sum())) & M64
    assert r["sum_s"] == (a * int(sp.sum())) & M64
    # duplicate multiplicities: count = sum_k m_R(k) m_S(k)
    rk = rng.integers(0, 50, 2000).astype(np.int32)
    sk = rng.integers(25, 80, 3000).astype(np.int32)
    cr, cs = collections.Counter(rk.tolist()), collections.Counter(sk.tolist())
    r = oracle.join(rk, np.zeros_like(rk), sk, np.zeros_like(sk))
    assert r["count"] == sum(cr[k] * cs[k] for k in cr)


def _numpy_join_counts(rk, rp, sk, sp):
    """count / sum_r / sum_s via np.unique + np.searchsorted (library routine)."""
    ur, inv_r = np.unique(rk, return_inverse=True)
    mult_r = np.bincount(inv_r, minlength=len(ur))
    psum_r = np.bincount(inv_r, weights=None, minlength=len(ur))  # placeholder shape
    # per-key payload sums in exact integer arithmetic (object-free): use uint64 wrap
    rp_u = rp.astype(np.int64).view(np.uint64)
    order = np.argsort(inv_r, kind="stable")
    starts = np.searchsorted(inv_r[order], np.arange(len(ur)))
    csum = np.concatenate([[np.uint64(0)], np.cumsum(rp_u[order], dtype=np.uint64)])
    ends = np.append(starts[1:], len(order))
    psum_r = csum[ends] - csum[starts]
    pos = np.searchsorted(ur, sk)
    pos_c = np.minimum(pos, len(ur) - 1)
    hit = (len(ur) > 0) & (ur[pos_c] == sk) if len(ur) else np.zeros(len(sk), bool)
    m = np.where(hit, mult_r[pos_c], 0).astype(np.uint64)
    cnt = int(m.sum(dtype=np.uint64))
    sum_s = int(np.add.reduce(m * sp.astype(np.int64).view(np.uint64), dtype=np.uint64))
    sum_r = int(np.add.reduce(np.where(hit, psum_r[pos_c], np.uint64(0)), dtype=np.uint64))
    return cnt, sum_r, sum_s


@pytest.mark.parametrize("n,dom", [(1 << 16, 1 << 16), (1 << 18, 1000), (100_003, 50_000)])
def test_oracle_vs_numpy_library(n, dom):
    rng = np.random.default_rng(n + dom)
    rk = rng.integers(0, dom, n).astype(np.int64)
    sk = rng.integers(0, dom, n + 17).astype(np.int64)
    rp = rng.integers(-2**40, 2**40, n)
    sp = rng.integers(-2**40, 2**40, n + 17)
    r = oracle.join(rk, rp, sk, sp)
    assert (r["count"], r["sum_r"], r["sum_s"]) == _numpy_join_counts(rk, rp, sk, sp)


@pytest.mark.parametrize("cfg,nr,ns", [("c1", 1 << 14, 1 << 14), ("c1", 3001, 3001),
                                       ("c2", 1 << 15, 1 << 15), ("c3", 1 << 12, 1 << 15),
                                       ("c3", 777, 5003), ("c5", 1 << 12, 1 << 14)])
def test_oracle_vs_provenance(cfg, nr, ns):
    wl = datagen.make(cfg, n_r=nr, n_s=ns)
    want = provenance.expected_from_workload(wl)
    got = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)
    exp_pairs = provenance.expected_pkfk(np.asarray(wl.R.payload)[wl.idx.astype(np.int64)],
                                         wl.S.payload, materialize=True)["pairs"]
    assert {k: got[k] for k in want} == want
    assert np.array_equal(got["pairs"][0], exp_pairs[0])
    assert np.array_equal(got["pairs"][1], exp_pairs[1])
    assert got["count"] == ns  # closed form (P793-794)


@pytest.mark.parametrize("threads", [1, 3, 8])
def test_sharded_oracle_equals_oracle(threads):
    """SURVEY §8.d.6's T-thread oracle adds up to the single-thread one."""
    rng = np.random.default_rng(31 + threads)
    rk = rng.integers(-500, 500, 20000).astype(np.int64)
    sk = rng.integers(-600, 600, 30000).astype(np.int64)
    rp = rng.integers(-2**40, 2**40, 20000).astype(np.int64)
    sp = rng.integers(-2**40, 2**40, 30000).astype(np.int32)
    want = oracle.join(rk, rp, sk, sp)
    got = oracle.join_sharded(rk, rp, sk, sp, threads=threads)
    assert {k: got[k] for k in want} == want and got["threads"] == threads
