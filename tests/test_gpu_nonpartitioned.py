"""GPU parity of hape_nonpartitioned_join (the non-partitioned GPU hash join of
PAPER.md Fig. 6, P859-870) against the CPU oracle,
element by element on the same seeded inputs: count, sums, pair checksum
bit-exact and the sorted pair multiset equal.  The method differs from the
radix join (one HBM table over all of R, no partitioning) but the result is
the same plain definition, so the same oracle decides.
"""
import numpy as np
import pytest
import torch

import datagen
import oracle
from oracle import provenance

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_conf_cidr_chrysogelossa19_b200 import HapeError, RadixJoin, _lib

DT = {32: torch.int32, 64: torch.int64}


def cuda(a):
    return torch.as_tensor(np.ascontiguousarray(a)).cuda()


def check(res, want):
    got = dict(count=res.match_count, sum_r=res.sum_r_payload, sum_s=res.sum_s_payload,
               checksum=res.pair_checksum)
    assert got == {k: want[k] for k in got}, (got, want)


def sorted_pairs(a, b):
    a = a.cpu().numpy().astype(np.int64)
    b = b.cpu().numpy().astype(np.int64)
    o = np.lexsort((b, a))
    return a[o], b[o]


_handles = {}


def joiner(kdt, rdt=None, sdt=None, **kw):
    key = (kdt, rdt, sdt, tuple(sorted(kw.items())))
    if key not in _handles:
        _handles[key] = RadixJoin(key_dtype=kdt, r_payload_dtype=rdt or kdt, s_payload_dtype=sdt or kdt, **kw)
    return _handles[key]


@pytest.mark.parametrize("seed", range(24))
def test_random_small_vs_oracle(seed):
    rng = np.random.default_rng(7000 + seed)
    kb = [32, 64][seed % 2]
    rb = [32, 64][(seed // 2) % 2]
    sb = [32, 64][(seed // 4) % 2]
    nr = int(rng.choice([0, 1, 5, 100, 4097, 20000, 70001]))
    ns = int(rng.choice([0, 1, 7, 100, 4096, 30011, 65537]))
    dom = int(rng.choice([1, 3, 64, 5000, 1 << 30]))
    kdt = np.int32 if kb == 32 else np.int64
    rk = (rng.integers(0, dom, nr) - dom // 2).astype(kdt)
    sk = (rng.integers(0, dom, ns) - dom // 2).astype(kdt)
    if nr * ns > 0 and nr * ns * 1.0 / max(dom, 1) > 2e6:  # keep |J| (and the chains) bounded
        sk = sk[: max(1, int(2e6 * dom / nr))]
        ns = len(sk)
    rp = rng.integers(-2**31, 2**31, nr).astype(np.int32 if rb == 32 else np.int64)
    sp = rng.integers(-2**31, 2**31, ns).astype(np.int32 if sb == 32 else np.int64)
    if rb == 64:
        rp = rp * 7919 + (1 << 40)
    want = oracle.join(rk, rp, sk, sp, materialize=True)
    n = want["count"]
    out_r = torch.empty(max(n, 1), dtype=DT[rb], device="cuda")
    out_s = torch.empty(max(n, 1), dtype=DT[sb], device="cuda")
    res = joiner(DT[kb], DT[rb], DT[sb]).join_nonpartitioned(cuda(rk), cuda(rp), cuda(sk), cuda(sp),
                                                              out_r, out_s)
    check(res, want)
    assert res.n_written == n
    a, b = sorted_pairs(out_r[:n], out_s[:n])
    assert np.array_equal(a, want["pairs"][0]) and np.array_equal(b, want["pairs"][1])
    assert res.stage_ms["np_probe"] >= 0 and res.passes == 0


@pytest.mark.parametrize("cfg,nr,ns,unique", [("c1", 1 << 20, 1 << 20, False), ("c2", 1 << 22, 1 << 22, True),
                                              ("c3", 1 << 18, 1 << 21, True), ("c3", 100_003, 700_001, False),
                                              ("c5", 1 << 18, 1 << 20, True)])
def test_config_recipes_vs_oracle(cfg, nr, ns, unique):
    wl = datagen.make(cfg, n_r=nr, n_s=ns)
    kdt = DT[wl.key_bits]
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    res = joiner(kdt, r_unique=unique).join_nonpartitioned(cuda(wl.R.key), cuda(wl.R.payload),
                                                           cuda(wl.S.key), cuda(wl.S.payload))
    check(res, want)
    assert res.match_count == ns  # closed form (P793-794)


@pytest.mark.slow
def test_same_result_as_radix_join_c2_full():
    # both methods on BASELINE configs[1] (2^27 x 2^27): the generator
    # provenance fixes the result; radix and non-partitioned must both hit it
    wl = datagen.make("c2", backend="torch", device="cuda")
    want = provenance.expected_pkfk(wl.R.payload[wl.idx].cpu().numpy(), wl.S.payload.cpu().numpy())
    j = joiner(torch.int32, r_unique=True)
    args = (wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    check(j.join_nonpartitioned(*args), want)
    check(j.join(*args), want)


def test_duplicates_extremes_empty_capacity_host():
    # duplicate-heavy keys (long probe runs), extreme key values, empty sides,
    # the capacity protocol and host-resident inputs/outputs
    rng = np.random.default_rng(9)
    rk = rng.integers(0, 3, 5000).astype(np.int64)
    sk = rng.integers(0, 4, 7000).astype(np.int64)
    rp = rng.integers(-100, 100, 5000).astype(np.int64)
    sp = rng.integers(-100, 100, 7000).astype(np.int64)
    check(joiner(torch.int64).join_nonpartitioned(cuda(rk), cuda(rp), cuda(sk), cuda(sp)),
          oracle.join(rk, rp, sk, sp))
    for kdt in (np.int32, np.int64):
        info = np.iinfo(kdt)
        vals = np.array([info.min, info.max, -1, 0, 1], kdt)
        rk = rng.choice(vals, 300).astype(kdt)
        sk = rng.choice(vals, 500).astype(kdt)
        rp = np.arange(300).astype(kdt)
        sp = np.arange(500).astype(kdt)
        res = joiner(torch.from_numpy(rk).dtype).join_nonpartitioned(cuda(rk), cuda(rp), cuda(sk), cuda(sp))
        check(res, oracle.join(rk, rp, sk, sp))
    e = torch.empty(0, dtype=torch.int32, device="cuda")
    x = torch.arange(100, dtype=torch.int32, device="cuda")
    for args in ((e, e, x, x), (x, x, e, e)):
        assert joiner(torch.int32).join_nonpartitioned(*args).as_tuple() == (0, 0, 0, 0)
    wl = datagen.make("c1", n_r=1 << 16, n_s=1 << 16)
    want = provenance.expected_from_workload(wl)
    out_r = torch.empty(1000, dtype=torch.int32, device="cuda")
    out_s = torch.empty(1000, dtype=torch.int32, device="cuda")
    args = (cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload))
    with pytest.raises(HapeError) as ei:
        joiner(torch.int32).join_nonpartitioned(*args, out_r, out_s)
    assert ei.value.status == _lib.HAPE_ERR_OUTPUT_CAPACITY
    res = joiner(torch.int32).join_nonpartitioned(*args, out_r, out_s, raise_on_capacity=False)
    check(res, want)
    assert res.n_required == 1 << 16 and res.n_written == 1000
    pin = lambda a: torch.from_numpy(np.ascontiguousarray(a)).pin_memory()
    n = want["count"]
    hr = torch.empty(n, dtype=torch.int32).pin_memory()
    hs = torch.empty(n, dtype=torch.int32).pin_memory()
    res = joiner(torch.int32).join_nonpartitioned(pin(wl.R.key), pin(wl.R.payload), pin(wl.S.key),
                                                  pin(wl.S.payload), hr, hs)
    check(res, want)
    a, b = sorted_pairs(hr, hs)
    w = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)["pairs"]
    assert np.array_equal(a, w[0]) and np.array_equal(b, w[1])
