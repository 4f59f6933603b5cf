"""The G>1 device path on ONE GPU (e; §4 "loopback test").

hape_debug_route runs the destination partition the multi-GPU path runs
before its exchange -- fan-out G on the top log2(G) bits of h, the "hash-
based" router policy of PAPER.md P643-652 (R14).
hape_debug_loopback_join runs G simulated ranks on this GPU: every shard is
routed into a send region, the count matrix is read back, hape_exchange_plan
gives the receive offsets, each destination's segments are copied to its
receive buffer (the all-to-allv, device copies in place of NCCL) and each
destination's local join runs on the received AoS tuples.

Checks (all bit-exact, oracle side = oracle/ only):
  * a routed segment d holds exactly the tuples whose destination (oracle
    partition.destination) is d, as a multiset of (key, payload);
  * the G per-destination results equal the oracle join of the tuples routed
    to d (every rank's share is exact, R14), and sum to the oracle's global
    result; the concatenated pairs equal the oracle's pair multiset.
"""
import numpy as np
import pytest
import torch

import datagen
import oracle
from oracle import partition

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin

DT = {32: torch.int32, 64: torch.int64}
M64 = (1 << 64) - 1


def cuda(a):
    return torch.as_tensor(np.ascontiguousarray(a)).cuda()


def sorted_pairs(a, b):
    a = np.asarray(a).astype(np.int64)
    b = np.asarray(b).astype(np.int64)
    o = np.lexsort((b, a))
    return a[o], b[o]


_handles = {}


def joiner(kb, rb, sb):
    key = (kb, rb, sb)
    if key not in _handles:
        _handles[key] = RadixJoin(key_dtype=DT[kb], r_payload_dtype=DT[rb], s_payload_dtype=DT[sb])
    return _handles[key]


def workload(cfg, nr, ns, seed=0):
    if cfg == "dup":
        return datagen.make("dup", n_r=nr, n_s=ns, dup_domain=97)
    if cfg == "c5":
        return datagen.make("c5", n_r=nr, n_s=ns, theta=1.0)
    if cfg == "mixed":  # int64 keys, int32 R payloads, int64 S payloads, negatives
        rng = np.random.default_rng(77 + seed)
        rk = rng.integers(-2**62, 2**62, nr).astype(np.int64)
        sk = np.where(rng.random(ns) < 0.7, rk[rng.integers(0, nr, ns)], rng.integers(-2**62, 2**62, ns))
        R = datagen.Relation(rk, rng.integers(-2**31, 2**31, nr).astype(np.int32))
        S = datagen.Relation(sk.astype(np.int64), rng.integers(-2**62, 2**62, ns).astype(np.int64))
        return datagen.Workload("mixed", R, S, None, nr, ns, 64, 64, "mixed")
    return datagen.make(cfg, n_r=nr, n_s=ns)


def dtypes(wl):
    return wl.key_bits, (32 if wl.R.payload.dtype == np.int32 else 64), (32 if wl.S.payload.dtype == np.int32 else 64)


# --------------------------------------------------------------------------
@pytest.mark.parametrize("G", [1, 2, 4, 8, 64])
@pytest.mark.parametrize("cfg,n", [("c1", (1 << 18) + 333), ("c3", 70001), ("dup", 9000)])
def test_route_segments_hold_their_destination(G, cfg, n):
    wl = workload(cfg, n, n)
    kb, rb, sb = dtypes(wl)
    j = joiner(kb, rb, sb)
    for rel, is_s in ((wl.R, False), (wl.S, True)):
        k, p, b = j.debug_route(cuda(rel.key), cuda(rel.payload), G, is_s=is_s)
        k, p, b = k.cpu().numpy(), p.cpu().numpy(), b.cpu().numpy()
        assert b[0] == 0 and b[-1] == len(rel.key) and np.all(np.diff(b) >= 0)
        dest = partition.destination(rel.key, G)
        # segment sizes are the destination histogram
        assert np.array_equal(np.diff(b), np.bincount(dest, minlength=G))
        for d in range(G):
            seg_k, seg_p = k[b[d]:b[d + 1]], p[b[d]:b[d + 1]]
            assert np.all(partition.destination(seg_k, G) == d)
            want = sorted_pairs(rel.key[dest == d], rel.payload[dest == d])
            got = sorted_pairs(seg_k, seg_p)
            assert np.array_equal(got[0], want[0]) and np.array_equal(got[1], want[1])


@pytest.mark.parametrize("peer", [False, True])
@pytest.mark.parametrize("G", [2, 4, 8])
@pytest.mark.parametrize("cfg,nr,ns", [("c1", 1 << 18, (1 << 18) + 4097), ("c3", 1 << 16, 1 << 18),
                                       ("dup", 6000, 7001), ("c5", 1 << 17, 1 << 19), ("mixed", 30011, 50021)])
def test_loopback_join_vs_oracle(G, cfg, nr, ns, peer):
    wl = workload(cfg, nr, ns)
    kb, rb, sb = dtypes(wl)
    j = joiner(kb, rb, sb)
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)
    # rank g holds contiguous row shards of R and of S (the bench layout)
    cut = lambda n: [(n * g) // G for g in range(G + 1)]
    cr, cs = cut(nr), cut(ns)
    r_sh = [(cuda(wl.R.key[cr[g]:cr[g + 1]]), cuda(wl.R.payload[cr[g]:cr[g + 1]])) for g in range(G)]
    s_sh = [(cuda(wl.S.key[cs[g]:cs[g + 1]]), cuda(wl.S.payload[cs[g]:cs[g + 1]])) for g in range(G)]
    n = want["count"]
    out_r = torch.empty(max(n, 1), dtype=DT[rb], device="cuda")
    out_s = torch.empty(max(n, 1), dtype=DT[sb], device="cuda")
    tot, per = j.loopback_join(r_sh, s_sh, out_r, out_s, peer=peer)
    got = dict(count=tot.match_count, sum_r=tot.sum_r_payload, sum_s=tot.sum_s_payload, checksum=tot.pair_checksum)
    assert got == {k: want[k] for k in got}
    assert tot.n_written == n
    pr, ps = sorted_pairs(out_r[:n].cpu().numpy(), out_s[:n].cpu().numpy())
    assert np.array_equal(pr, want["pairs"][0]) and np.array_equal(ps, want["pairs"][1])
    # every destination's share is exactly the oracle join of what routes there
    dR = partition.destination(wl.R.key, G)
    dS = partition.destination(wl.S.key, G)
    for d in range(G):
        wd = oracle.join(wl.R.key[dR == d], wl.R.payload[dR == d], wl.S.key[dS == d], wl.S.payload[dS == d])
        pd = per[d]
        assert (pd.local_match_count, pd.local_sum_r, pd.local_sum_s, pd.local_pair_checksum) == \
            (wd["count"], wd["sum_r"], wd["sum_s"], wd["checksum"]), d
        assert pd.r_local == int((dR == d).sum()) and pd.s_local == int((dS == d).sum())


@pytest.mark.parametrize("peer", [False, True])
def test_loopback_ragged_and_empty_shards(peer):
    wl = datagen.make("c1", n_r=50000, n_s=70000)
    j = joiner(32, 32, 32)
    G = 4
    cr = [0, 0, 12345, 49999, 50000]          # rank 0 holds no R, rank 3 one tuple
    cs = [0, 70000, 70000, 70000, 70000]      # rank 0 holds all of S
    r_sh = [(cuda(wl.R.key[cr[g]:cr[g + 1]]), cuda(wl.R.payload[cr[g]:cr[g + 1]])) for g in range(G)]
    s_sh = [(cuda(wl.S.key[cs[g]:cs[g + 1]]), cuda(wl.S.payload[cs[g]:cs[g + 1]])) for g in range(G)]
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    tot, per = j.loopback_join(r_sh, s_sh, peer=peer)
    assert (tot.match_count, tot.sum_r_payload, tot.sum_s_payload, tot.pair_checksum) == \
        (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
    assert sum(p.r_local for p in per) == 50000 and sum(p.s_local for p in per) == 70000


def test_loopback_results_identical_across_G():
    """SURVEY §8.c.4 multi-GPU pin: the G = 1/2/4/8 results are bit-identical
    (both exchange forms)."""
    wl = datagen.make("c2", n_r=1 << 19, n_s=1 << 19)
    j = joiner(32, 32, 32)
    res = set()
    for G, peer in ((1, False), (2, False), (4, False), (8, False), (1, True), (2, True), (8, True), (16, True)):
        cut = [((1 << 19) * g) // G for g in range(G + 1)]
        sh = lambda rel: [(cuda(rel.key[cut[g]:cut[g + 1]]), cuda(rel.payload[cut[g]:cut[g + 1]])) for g in range(G)]
        tot, _ = j.loopback_join(sh(wl.R), sh(wl.S), peer=peer)
        res.add(tot.as_tuple())
    assert len(res) == 1
    assert next(iter(res))[0] == 1 << 19


def test_stream_ordering_after_async_producer():
    """inputs written by torch on its current stream right
    before the call must be visible to the library's kernels."""
    n = 1 << 22
    wl = datagen.make("c2", n_r=n, n_s=n)
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    j = RadixJoin(key_dtype=torch.int32)
    rk = torch.empty(n, dtype=torch.int32, device="cuda")
    rp, sk, sp = torch.empty_like(rk), torch.empty_like(rk), torch.empty_like(rk)
    src = [cuda(a) for a in (wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)]
    for _ in range(3):
        for t in (rk, rp, sk, sp):
            t.fill_(-1)
        torch.cuda._sleep(20_000_000)        # delay the producer on torch's stream
        for t, s in zip((rk, rp, sk, sp), src):
            t.copy_(s, non_blocking=True)
        res = j.join(rk, rp, sk, sp)
        assert (res.match_count, res.sum_r_payload, res.sum_s_payload, res.pair_checksum) == \
            (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
    j.close()
