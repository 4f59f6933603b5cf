"""GPU parity: the CUDA path (through the C ABI) vs the CPU oracle, element by
element on the same seeded inputs.  All results are integers, so the bar is
bit-exact: count, sum_r, sum_s, pair_checksum, and the sorted pair multiset.
"""
import numpy as np
import pytest
import torch

import datagen
import oracle
from oracle import partition, provenance

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_conf_cidr_chrysogelossa19_b200 import HapeError, RadixJoin, _lib

M64 = (1 << 64) - 1
DT = {32: torch.int32, 64: torch.int64}


def cuda(a):
    return torch.as_tensor(np.ascontiguousarray(a)).cuda()


def oracle_res(rk, rp, sk, sp, materialize=False):
    return oracle.join(rk, rp, sk, sp, materialize=materialize)


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


# --------------------------------------------------------------------------
@pytest.mark.parametrize("seed", range(40))
def test_random_small_vs_oracle(seed):
    rng = np.random.default_rng(1000 + seed)
    kb = [32, 64][seed % 2]
    rb = [32, 64][(seed // 2) % 2]
    sb = [32, 64][(seed // 4) % 2]
    nr = int(rng.choice([0, 1, 5, 100, 4097, 20000, 70001]))
    ns = int(rng.choice([0, 1, 7, 100, 4096, 30011, 65537]))
    dom = int(rng.choice([1, 3, 64, 5000, 1 << 30]))
    kdt = np.int32 if kb == 32 else np.int64
    rk = (rng.integers(0, dom, nr) - dom // 2).astype(kdt)
    sk = (rng.integers(0, dom, ns) - dom // 2).astype(kdt)
    if nr * ns > 0 and nr * ns * 1.0 / max(dom, 1) > 5e6:  # keep |J| bounded
        sk = sk[: max(1, int(5e6 * dom / nr))]
        ns = len(sk)
    rp = rng.integers(-2**31, 2**31, nr).astype(np.int32 if rb == 32 else np.int64)
    sp = rng.integers(-2**31, 2**31, ns).astype(np.int32 if sb == 32 else np.int64)
    if rb == 64:
        rp = rp * 7919 + (1 << 40)
    j = joiner(DT[kb], DT[rb], DT[sb])
    want = oracle_res(rk, rp, sk, sp, materialize=True)
    n = want["count"]
    out_r = torch.empty(max(n, 1), dtype=DT[rb], device="cuda")
    out_s = torch.empty(max(n, 1), dtype=DT[sb], device="cuda")
    res = j.join(cuda(rk), cuda(rp), cuda(sk), cuda(sp), out_r, out_s)
    check(res, want)
    assert res.n_written == n
    a, b = sorted_pairs(out_r[:n], out_s[:n])
    assert np.array_equal(a, want["pairs"][0]) and np.array_equal(b, want["pairs"][1])


@pytest.mark.parametrize("cfg,nr,ns", [("c1", 1 << 20, 1 << 20), ("c2", 1 << 22, 1 << 22),
                                       ("c2", (1 << 22) + 12345, (1 << 22) + 12345),
                                       ("c3", 1 << 18, 1 << 21), ("c3", 100_003, 700_001),
                                       ("c5", 1 << 18, 1 << 20)])
def test_config_recipes_vs_oracle(cfg, nr, ns):
    wl = datagen.make(cfg, n_r=nr, n_s=ns)
    kdt = DT[wl.key_bits]
    want = oracle_res(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    j = joiner(kdt)
    res = j.join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload))
    check(res, want)
    assert res.match_count == ns  # closed form (P793-794)


@pytest.mark.parametrize("cfg,nr,ns", [("c1", 1 << 18, 1 << 18), ("c3", 1 << 16, 1 << 19),
                                       ("c5", 1 << 17, 1 << 19), ("c2", 100_003, 200_011)])
def test_declared_unique_build_side_vs_oracle(cfg, nr, ns):
    # HAPE_FLAG_R_UNIQUE (R is a primary key in every BASELINE recipe): the
    # probe stops at the first match; results must not change
    wl = datagen.make(cfg, n_r=nr, n_s=ns)
    kdt = DT[wl.key_bits]
    want = oracle_res(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)
    n = want["count"]
    out_r = torch.empty(n, dtype=kdt, device="cuda")
    out_s = torch.empty(n, dtype=kdt, device="cuda")
    res = joiner(kdt, r_unique=True).join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload),
                                          out_r, out_s)
    check(res, want)
    a, b = sorted_pairs(out_r, out_s)
    assert np.array_equal(a, want["pairs"][0]) and np.array_equal(b, want["pairs"][1])


def test_c1_full_with_pairs_vs_oracle():
    wl = datagen.make("c1")
    want = oracle_res(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)
    j = joiner(torch.int32)
    n = want["count"]
    out_r = torch.empty(n, dtype=torch.int32, device="cuda")
    out_s = torch.empty(n, dtype=torch.int32, device="cuda")
    res = j.join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload), out_r, out_s)
    check(res, want)
    a, b = sorted_pairs(out_r, out_s)
    assert np.array_equal(a, want["pairs"][0]) and np.array_equal(b, want["pairs"][1])


@pytest.mark.parametrize("passes,bits", [(1, (0, 0)), (1, (4, 0)), (1, (11, 0)), (2, (3, 5)),
                                         (2, (8, 8)), (2, (12, 2)), (2, (6, 12)), (2, (10, 10)),
                                         (2, (12, 12)), (1, (12, 0))])
@pytest.mark.parametrize("uq", [False, True])
def test_metamorphic_plans_identical(passes, bits, uq):
    # uq: the declared-unique probe (large co-partitions of the coarse plans
    # take the 512-consumer shape and R-chunking there)
    wl = datagen.make("c2", n_r=1 << 20, n_s=(1 << 20) + 3)
    ref = provenance.expected_from_workload(wl)
    j = joiner(torch.int32, radix_passes=passes, radix_bits=bits, r_unique=uq)
    res = j.join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload))
    check(res, ref)
    assert res.passes == passes


def test_duplicate_heavy_and_oversized_partitions():
    # R partitions far larger than the smem build capacity (R-chunking) and
    # huge S partitions (S-slices): all keys in a handful of values
    rng = np.random.default_rng(5)
    rk = rng.integers(0, 3, 20000).astype(np.int32)
    sk = rng.integers(0, 4, 50000).astype(np.int32)
    rp = rng.integers(-100, 100, 20000).astype(np.int32)
    sp = rng.integers(-100, 100, 50000).astype(np.int32)
    want = oracle_res(rk, rp, sk, sp)
    res = joiner(torch.int32).join(cuda(rk), cuda(rp), cuda(sk), cuda(sp))
    check(res, want)
    # all-equal keys: a*b
    a, b = 5000, 3000
    res = joiner(torch.int64).join(cuda(np.full(a, -7, np.int64)), cuda(np.arange(a)),
                                   cuda(np.full(b, -7, np.int64)), cuda(np.arange(b)))
    assert res.match_count == a * b
    assert res.sum_r_payload == (b * (a * (a - 1) // 2)) & M64


def test_extreme_keys():
    for kdt in (np.int32, np.int64):
        info = np.iinfo(kdt)
        vals = np.array([info.min, info.max, -1, 0, 1, info.min + 1, info.max - 1], kdt)
        rng = np.random.default_rng(3)
        rk = rng.choice(vals, 3000).astype(kdt)
        sk = rng.choice(vals, 5000).astype(kdt)
        rp = np.arange(3000).astype(kdt)
        sp = np.arange(5000).astype(kdt)
        want = oracle_res(rk, rp, sk, sp)
        res = joiner(torch.from_numpy(rk).dtype).join(cuda(rk), cuda(rp), cuda(sk), cuda(sp))
        check(res, want)


def test_empty_inputs():
    e32 = torch.empty(0, dtype=torch.int32, device="cuda")
    x = torch.arange(100, dtype=torch.int32, device="cuda")
    j = joiner(torch.int32)
    for args in ((e32, e32, x, x), (x, x, e32, e32), (e32, e32, e32, e32)):
        res = j.join(*args)
        assert res.as_tuple() == (0, 0, 0, 0)


def test_output_capacity_protocol():
    wl = datagen.make("c1", n_r=1 << 16, n_s=1 << 16)
    want = provenance.expected_from_workload(wl)
    j = joiner(torch.int32)
    out_r = torch.empty(1000, dtype=torch.int32, device="cuda")
    out_s = torch.empty(1000, dtype=torch.int32, device="cuda")
    args = (cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload))
    with pytest.raises(HapeError) as ei:
        j.join(*args, out_r, out_s)
    assert ei.value.status == _lib.HAPE_ERR_OUTPUT_CAPACITY
    res = j.join(*args, out_r, out_s, raise_on_capacity=False)
    check(res, want)
    assert res.n_required == 1 << 16 and res.n_written == 1000
    # the written prefix is a sub-multiset of J: every pair is a real match
    rp = np.asarray(wl.R.payload)
    pairs_ok = set(zip(rp[wl.idx.astype(np.int64)].tolist(), wl.S.payload.tolist()))
    got = set(zip(out_r.cpu().tolist(), out_s.cpu().tolist()))
    assert got <= pairs_ok and len(got) == 1000


def test_host_resident_inputs_and_outputs():
    wl = datagen.make("c3", n_r=1 << 15, n_s=1 << 17)
    want = oracle_res(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=True)
    pin = lambda a: torch.from_numpy(np.ascontiguousarray(a)).pin_memory()
    n = want["count"]
    out_r = torch.empty(n, dtype=torch.int64).pin_memory()
    out_s = torch.empty(n, dtype=torch.int64).pin_memory()
    res = joiner(torch.int64).join(pin(wl.R.key), pin(wl.R.payload), pin(wl.S.key), pin(wl.S.payload),
                                   out_r, out_s)
    check(res, want)
    a, b = sorted_pairs(out_r, out_s)
    assert np.array_equal(a, want["pairs"][0]) and np.array_equal(b, want["pairs"][1])
    assert res.stage_ms["h2d"] > 0


def test_invalid_args():
    j = joiner(torch.int32)
    x = torch.arange(10, dtype=torch.int32, device="cuda")
    R = _lib.hape_relation(None, None, 10, 0)
    S = _lib.hape_relation(x.data_ptr(), x.data_ptr(), 10, 0)
    res = _lib.hape_join_result()
    assert _lib.hape_radix_join(j.handle, R, S, None, res) == _lib.HAPE_ERR_INVALID_ARG
    R = _lib.hape_relation(x.data_ptr() + 1, x.data_ptr(), 9, 0)  # misaligned
    assert _lib.hape_radix_join(j.handle, R, S, None, res) == _lib.HAPE_ERR_INVALID_ARG
    R = _lib.hape_relation(x.data_ptr(), x.data_ptr(), 10, 7)     # bad mem kind
    assert _lib.hape_radix_join(j.handle, R, S, None, res) == _lib.HAPE_ERR_INVALID_ARG
    assert "mem" in _lib.hape_last_error(j.handle)


# ---- stage invariants (a6-a9) through the debug entry point -----------------
@pytest.mark.parametrize("passes,bits,kb", [(1, (9, 0), 32), (2, (8, 8), 32), (2, (5, 7), 64),
                                            (1, (12, 0), 64)])
def test_partition_invariants(passes, bits, kb):
    n = (1 << 20) + 777
    rng = np.random.default_rng(11)
    kdt = np.int32 if kb == 32 else np.int64
    keys = rng.integers(np.iinfo(kdt).min, np.iinfo(kdt).max, n, dtype=kdt)
    pays = np.arange(n).astype(kdt)
    j = joiner(DT[kb], radix_passes=passes, radix_bits=bits)
    ok, op, ob, plan = j.debug_partition(cuda(keys), cuda(pays))
    ok, op, ob = ok.cpu().numpy(), op.cpu().numpy(), ob.cpu().numpy()
    b1, b2 = bits
    Q = 1 << (b1 + (b2 if passes == 2 else 0))
    # bounds monotone, start at 0, end at N; histogram sums to N
    assert ob[0] == 0 and ob[-1] == n and np.all(np.diff(ob) >= 0) and len(ob) == Q + 1
    # permutation: payload column is a permutation of 0..n-1 and pairs stay together
    assert np.array_equal(np.sort(op), pays)
    assert np.array_equal(ok, keys[op.astype(np.int64)])
    # every tuple in partition q has partition_id(key) == q
    pid = partition.partition_id(ok, b1, b2 if passes == 2 else 0)
    expect = np.repeat(np.arange(Q), np.diff(ob))
    assert np.array_equal(pid, expect)
    # per-partition counts equal np.bincount of the partition function
    assert np.array_equal(np.diff(ob), np.bincount(partition.partition_id(keys, b1, b2 if passes == 2 else 0),
                                                   minlength=Q))


def test_identity_partitions_equal_size():
    # P802-804: "we select the keys so that all produced partitions have
    # exactly the same size" -- dense keys + identity partition function
    n = 1 << 21
    keys = np.random.default_rng(2).permutation(n).astype(np.int32)
    j = joiner(torch.int32, radix_passes=2, radix_bits=(6, 5), identity=True)
    ok, op, ob, _ = j.debug_partition(cuda(keys), cuda(keys))
    assert np.all(np.diff(ob.cpu().numpy()) == n >> 11)
    wl = datagen.make("c1", n_r=n, n_s=n)
    res = j.join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload))
    check(res, provenance.expected_from_workload(wl))


# ---- BASELINE full sizes, in the launch configuration bench.py times --------
@pytest.mark.slow
def test_c2_full_size_vs_oracle():
    # configs[1]: |R|=|S|=2^27 int32, 2-pass; the oracle's sort-merge (~15 s)
    # and the generator provenance both check the device result
    wl = datagen.make("c2", backend="torch", device="cuda")
    j = RadixJoin(key_dtype=torch.int32, max_r=1 << 27, max_s=1 << 27, r_unique=True)  # as bench.py
    res = j.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    rk, rp, sk, sp = (x.cpu().numpy() for x in (wl.R.key, wl.R.payload, wl.S.key, wl.S.payload))
    want = oracle_res(rk, rp, sk, sp)
    check(res, want)
    assert res.passes == 2 and res.bits == (8, 8)
    prov = provenance.expected_pkfk(rp[wl.idx.cpu().numpy()], sp)
    assert prov == want


@pytest.mark.slow
def test_c3_full_size_pairs_vs_provenance():
    # configs[2]: |R|=2^27, |S|=2^30 int64, 2^30 materialised pairs.  Count,
    # sums and checksum vs the provenance closed forms (oracle/provenance.py);
    # the pair multiset vs provenance by a sorted compare on the device.
    wl = datagen.make("c3", backend="torch", device="cuda")
    n = wl.S.key.shape[0]
    out_r = torch.empty(n, dtype=torch.int64, device="cuda")
    out_s = torch.empty(n, dtype=torch.int64, device="cuda")
    j = RadixJoin(key_dtype=torch.int64, max_r=1 << 27, max_s=1 << 30, r_unique=True)
    res = j.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, out_r, out_s)
    exp_r = wl.R.payload[wl.idx]
    want = provenance.expected_pkfk(exp_r.cpu().numpy(), wl.S.payload.cpu().numpy())
    check(res, want)
    assert res.n_written == n
    # every S payload is unique (sm() is a bijection), so sorting by s orders both sides
    o_got = torch.argsort(out_s)
    o_exp = torch.argsort(wl.S.payload)
    assert torch.equal(out_s[o_got], wl.S.payload[o_exp])
    assert torch.equal(out_r[o_got], exp_r[o_exp])


@pytest.mark.parametrize("theta", [0.5, 1.0])
def test_zipf_skew_vs_oracle(theta):
    # C5's skew recipe at one-GPU scale: the hottest key spans many S slices
    wl = datagen.make("c5", n_r=1 << 20, n_s=1 << 22, theta=theta)
    want = oracle_res(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    res = joiner(torch.int32).join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload))
    check(res, want)
    if theta == 1.0:
        assert res.n_items > res.n_partitions  # the hot co-partitions were split into S slices


# ---- the joint pass-1/pass-2 histogram (k_hist_joint) and the claiming pass 2
def test_joint_histogram_row_spill_partitions():
    # 2^24 tuples, 3/4 of them one key: every SM's 16-bit counters for that
    # key's row would pass 65535, so the row-spill path runs; the partition
    # invariants (bounds = bincount of the partition function, permutation)
    # must still hold exactly
    n = 1 << 24
    rng = np.random.default_rng(5)
    keys = rng.integers(-2**31, 2**31, n, dtype=np.int64).astype(np.int32)
    keys[rng.random(n) < 0.75] = 12345
    pays = np.arange(n, dtype=np.int32)
    j = joiner(torch.int32, radix_passes=2, radix_bits=(8, 8))
    ok, op, ob, plan = j.debug_partition(cuda(keys), cuda(pays))
    ok, op, ob = ok.cpu().numpy(), op.cpu().numpy(), ob.cpu().numpy()
    pid = partition.partition_id(keys, 8, 8)
    assert np.array_equal(np.diff(ob), np.bincount(pid, minlength=1 << 16))
    assert np.array_equal(np.sort(op), pays)
    assert np.array_equal(ok, keys[op.astype(np.int64)])
    assert np.array_equal(partition.partition_id(ok, 8, 8), np.repeat(np.arange(1 << 16), np.diff(ob)))


def test_joint_histogram_both_halves_of_one_word_wrap():
    # two hot keys whose joint buckets q (even) and q+1 share one 32-bit
    # counter word: the low half wraps and carries into the high half, which
    # wraps too -- the carry fix-up (ovf[q+1] adjustments) must net out exactly
    n = 1 << 24
    rng = np.random.default_rng(9)
    cand = rng.integers(-2**31, 2**31, 200000, dtype=np.int64).astype(np.int32)
    pid = partition.partition_id(cand, 8, 8)
    first = {}
    for k, q in zip(cand.tolist(), pid.tolist()):
        first.setdefault(int(q), k)
    q0 = next(q for q in sorted(first) if q % 2 == 0 and q + 1 in first)
    ka, kb = first[q0], first[q0 + 1]
    keys = rng.integers(-2**31, 2**31, n, dtype=np.int64).astype(np.int32)
    u = rng.random(n)
    keys[u < 0.45] = ka
    keys[(u >= 0.45) & (u < 0.9)] = kb
    pays = np.arange(n, dtype=np.int32)
    j = joiner(torch.int32, radix_passes=2, radix_bits=(8, 8))
    ok, op, ob, plan = j.debug_partition(cuda(keys), cuda(pays))
    ok, op, ob = ok.cpu().numpy(), op.cpu().numpy(), ob.cpu().numpy()
    pid = partition.partition_id(keys, 8, 8)
    assert np.array_equal(np.diff(ob), np.bincount(pid, minlength=1 << 16))
    assert np.array_equal(np.sort(op), pays)
    assert np.array_equal(ok, keys[op.astype(np.int64)])


def test_joint_histogram_skewed_join_vs_oracle():
    # the same skew through the join (one S tuple of the hot key: count = its
    # R multiplicity, the R co-partition is joined in chunks)
    n = 1 << 22
    rng = np.random.default_rng(6)
    rk = rng.integers(-2**31, 2**31, n, dtype=np.int64).astype(np.int32)
    rk[rng.random(n) < 0.6] = -7
    rp = rng.integers(-2**31, 2**31, n, dtype=np.int64).astype(np.int32)
    head = rk[:100000]
    sk = np.concatenate([head[head != -7], np.array([-7], np.int32)])
    sp = rng.integers(-2**31, 2**31, len(sk), dtype=np.int64).astype(np.int32)
    want = oracle_res(rk, rp, sk, sp)
    res = joiner(torch.int32, radix_passes=2, radix_bits=(8, 8)).join(cuda(rk), cuda(rp), cuda(sk), cuda(sp))
    check(res, want)


@pytest.mark.parametrize("identity", [False, True])
def test_open_addressing_refill_cases(identity):
    """k_join_oa's free-slot test is "the slot's key is in another
    co-partition".  Key 0 is the initial fill key (h(0) = 0: co-partition 0)
    and consecutive stages of ONE co-partition (R chunks of an oversized R
    side, and > grid S slices of a hot S side on one CTA) must refill."""
    rng = np.random.default_rng(99)
    hot = 1 << 23
    rk = np.concatenate([np.zeros(3, np.int32), np.full(7000, 1, np.int32), rng.integers(2, 50, 40000).astype(np.int32)])
    sk = np.concatenate([np.zeros(hot, np.int32), np.full(1000, 1, np.int32), rng.integers(0, 60, 5000).astype(np.int32)])
    rp = rng.integers(-2**31, 2**31, len(rk)).astype(np.int32)
    sp = rng.integers(-2**31, 2**31, len(sk)).astype(np.int32)
    want = oracle_res(rk, rp, sk, sp)
    res = joiner(torch.int32, identity=identity).join(cuda(rk), cuda(rp), cuda(sk), cuda(sp))
    check(res, want)
    assert res.n_items > 444
    # the same through the open-addressing form (child process: env read once)
    import subprocess, sys, os
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    np.savez("/tmp/_oa_refill.npz", rk=rk, rp=rp, sk=sk, sp=sp)
    code = (
        "import numpy as np, torch\n"
        "from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin\n"
        "z = np.load('/tmp/_oa_refill.npz'); d = lambda a: torch.from_numpy(z[a]).cuda()\n"
        f"j = RadixJoin(key_dtype=torch.int32, identity={identity})\n"
        "r = j.join(d('rk'), d('rp'), d('sk'), d('sp'))\n"
        "print(r.match_count, r.sum_r_payload, r.sum_s_payload, r.pair_checksum)\n")
    r = subprocess.run([sys.executable, "-c", code], cwd=root, capture_output=True, text=True, timeout=600,
                       env=dict(os.environ, HAPE_JN_OA="1", PYTHONPATH=root))
    assert r.returncode == 0, r.stderr
    assert r.stdout.split() == [str(want[k]) for k in ("count", "sum_r", "sum_s", "checksum")]


@pytest.mark.parametrize("env", [dict(HAPE_JOINT="0"), dict(HAPE_JOINT="0", HAPE_CLAIM="0"),
                                 dict(HAPE_HJ_TMA="1"), dict(HAPE_SC="3"), dict(HAPE_SC_WIDE="0"),
                                 dict(HAPE_JN_OA="1"), dict(HAPE_JN_SU="2"), dict(HAPE_JN_SU="0"),
                                 dict(HAPE_SC_AGG="1"), dict(HAPE_SC_AGG="2"),
                                 dict(HAPE_JN_EPOCH_PERIOD="1"), dict(HAPE_JN_EPOCH_PERIOD="3"),
                                 dict(HAPE_JN_LAY="1"), dict(HAPE_JN_LAY="0"), dict(HAPE_JN_LAY="2"),
                                 dict(HAPE_JN_LAY="1", HAPE_JN_SU="0"), dict(HAPE_JN_LAY="2", HAPE_JN_SU="0"),
                                 dict(HAPE_JN_LAY="1", HAPE_JN_EPOCH_PERIOD="1"),
                                 dict(HAPE_JN_NC="512"), dict(HAPE_JN_NC="256")])
def test_alternative_kernel_forms_vs_oracle(env):
    # the retained alternatives, each read once per process (child process):
    # HAPE_JOINT=0 the per-pass totals + claiming scatters (the path of plans
    # with bits[0]+bits[1] > 16), HAPE_CLAIM=0 per-CTA offset scatters,
    # HAPE_JN_OA=1 the open-addressing build+probe, HAPE_JN_SU the staged-S /
    # direct build+probe forms, HAPE_SC_AGG the warp-aggregated rankings,
    # HAPE_JN_EPOCH_PERIOD the chain-head epoch wrap (reset every 1 / 3 stages),
    # HAPE_JN_LAY the direct build+probe's table layouts forced (0 AoS
    # tuples + next[], 1 key|next nodes -- the bag default, 2 dense keys[]),
    # HAPE_JN_NC the unique direct form's 512- / 256-consumer shapes
    import subprocess
    import sys
    import os
    code = r'''
import numpy as np, torch, datagen, oracle
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin
for cfg, nr, ns, kdt, bits, uq in (("c2", 1 << 20, (1 << 20) + 333, torch.int32, (8, 8), False),
                                   ("c2", 1 << 20, (1 << 20) + 333, torch.int32, (8, 8), True),
                                   ("c3", 1 << 18, 1 << 20, torch.int64, (8, 8), False),
                                   ("dup", 9000, 12000, torch.int32, (9, 9), False)):
    wl = datagen.make(cfg, n_r=nr, n_s=ns, **(dict(dup_domain=300) if cfg == "dup" else {}))
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
    with RadixJoin(key_dtype=kdt, radix_passes=2, radix_bits=bits, r_unique=uq) as j:
        r = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
    got = dict(count=r.match_count, sum_r=r.sum_r_payload, sum_s=r.sum_s_payload, checksum=r.pair_checksum)
    assert got == {k: want[k] for k in got}, (cfg, got, want)
print("ok")
'''
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    e = dict(os.environ, PYTHONPATH=root, **env)
    r = subprocess.run([sys.executable, "-c", code], cwd=root, env=e, capture_output=True, text=True, timeout=600)
    assert r.returncode == 0 and "ok" in r.stdout, r.stdout + r.stderr


def test_separate_pass2_histogram_path_vs_oracle():
    # HAPE_JOINT=0 forces the separate pass-2 histogram + offset scatter (the
    # path plans with bits[0]+bits[1] > 16 take); read once per process, so it
    # runs in a child process
    import subprocess
    import sys
    import os
    code = r'''
import numpy as np, torch, datagen, oracle
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin
for cfg, nr, ns, kdt in (("c2", 1 << 20, (1 << 20) + 333, torch.int32), ("c3", 1 << 18, 1 << 20, torch.int64)):
    wl = datagen.make(cfg, n_r=nr, n_s=ns)
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
    with RadixJoin(key_dtype=kdt, radix_passes=2, radix_bits=(8, 8)) as j:
        r = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
    got = dict(count=r.match_count, sum_r=r.sum_r_payload, sum_s=r.sum_s_payload, checksum=r.pair_checksum)
    assert got == {k: want[k] for k in got}, (cfg, got, want)
print("ok")
'''
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, HAPE_JOINT="0", PYTHONPATH=root)
    r = subprocess.run([sys.executable, "-c", code], cwd=root, env=env, capture_output=True, text=True, timeout=600)
    assert r.returncode == 0 and "ok" in r.stdout, r.stdout + r.stderr


# ---- the paper's single-scan linked-buffer pass 1 (HAPE_FLAG_LINKED, NEXT-2) --
@pytest.mark.parametrize("bits", [(8, 8), (3, 5), (10, 10), (12, 4), (6, 12)])
@pytest.mark.parametrize("cfg", ["c2", "c3", "dup", "c5"])
def test_linked_pass1_vs_oracle(cfg, bits):
    n = {"c2": 1 << 20, "c3": 1 << 18, "dup": 20000, "c5": 1 << 19}[cfg]
    kw = dict(dup_domain=300) if cfg == "dup" else (dict(theta=1.0) if cfg == "c5" else {})
    wl = datagen.make(cfg, n_r=n, n_s=2 * n + 77, **kw)
    kdt = DT[wl.key_bits]
    want = oracle_res(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload, materialize=cfg != "c5")
    j = joiner(kdt, radix_passes=2, radix_bits=bits, linked=True)
    out = None
    if cfg != "c5":
        out = (torch.empty(max(want["count"], 1), dtype=kdt, device="cuda"),
               torch.empty(max(want["count"], 1), dtype=kdt, device="cuda"))
    res = j.join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload), *(out or (None, None)))
    check(res, want)
    if out is not None:
        a, b = sorted_pairs(out[0][:want["count"]], out[1][:want["count"]])
        assert np.array_equal(a, want["pairs"][0]) and np.array_equal(b, want["pairs"][1])
    # repeated call (graph replay, directory reset inside the graph)
    res2 = j.join(cuda(wl.R.key), cuda(wl.R.payload), cuda(wl.S.key), cuda(wl.S.payload), *(out or (None, None)))
    assert res2.as_tuple() == res.as_tuple()


@pytest.mark.parametrize("bits,kb", [((8, 8), 32), ((5, 7), 64), ((11, 9), 32)])
def test_linked_partition_invariants(bits, kb):
    n = (1 << 20) + 777
    rng = np.random.default_rng(13)
    kdt = np.int32 if kb == 32 else np.int64
    keys = rng.integers(np.iinfo(kdt).min, np.iinfo(kdt).max, n, dtype=kdt)
    keys[: n // 5] = keys[0]                      # a hot key: one chain far longer than the others
    pays = np.arange(n).astype(kdt)
    j = joiner(DT[kb], radix_passes=2, radix_bits=bits, linked=True)
    ok, op, ob, plan = j.debug_partition(cuda(keys), cuda(pays))
    ok, op, ob = ok.cpu().numpy(), op.cpu().numpy(), ob.cpu().numpy()
    b1, b2 = bits
    Q = 1 << (b1 + b2)
    assert ob[0] == 0 and ob[-1] == n and np.all(np.diff(ob) >= 0) and len(ob) == Q + 1
    assert np.array_equal(np.sort(op), pays)
    assert np.array_equal(ok, keys[op.astype(np.int64)])
    pid = partition.partition_id(ok, b1, b2)
    assert np.array_equal(pid, np.repeat(np.arange(Q), np.diff(ob)))


def test_linked_graph_replay_after_workspace_regrowth():
    """The cached CUDA graph of a linked join must not outlive the buffer
    directory it captured: a larger debug partition on the same handle
    regrows the directory, and the next join with the old pointers/sizes
    must re-capture (graph key includes the directory)."""
    j = RadixJoin(key_dtype=torch.int32, radix_passes=2, radix_bits=(8, 8), linked=True)
    wl = datagen.make("c2", n_r=1 << 18, n_s=1 << 18)
    args = [cuda(a) for a in (wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)]
    want = provenance.expected_from_workload(wl)
    check(j.join(*args), want)
    big = datagen.make("c2", n_r=1 << 21, n_s=1 << 21)
    j.debug_partition(cuda(big.R.key), cuda(big.R.payload))
    torch.cuda.empty_cache()
    check(j.join(*args), want)
    check(j.join(*args), want)
    j.close()
