"""Seeded, counter-based synthetic (key, payload) relations.

This module is the ONE piece shared by the oracle side (tests, ``oracle/``
checks, bench ``cpu_baseline``) and the CUDA side (tests, bench).  It holds
none of the join's arithmetic: no partition function, no hash table, no
checksum.  It only decides *which* tuples exist, and records the provenance
``idx[j]`` (the R row whose key S row j copies) so that expected results can
be derived without running a join.

Workload shapes follow the paper's radix-join experiments:
  * two tables, each a key column and a payload column, an equi-join on the
    key followed by sum/count over each payload (PAPER.md P789-793, §6.2);
  * "Both tables have exactly the same keys" (P793-794) -> the dense PK-FK
    recipes ``c1``/``c2``/``c4`` below;
  * table sizes 1-128 M tuples in GPU memory (P862-864), 256 M-2 G for
    co-processing (P875-876);
  * BASELINE.json ``configs`` fixes the five shapes (c1..c5).

Generator definition:
  sm(x)       = splitmix64 output for state x: fmix64(x + 0x9E3779B97F4A7C15)
  perm_w(i;s) = 3 rounds of  x = (x*a_r + c_r) mod 2^w ; x ^= x >> ceil(w/2)
                with a_r = sm(s+r) | 1, c_r = sm(s+r+256); a bijection of
                [0, 2^w).  For n not a power of two, cycle-walk into [0, n).
  seeds       : sub(cfg, stream) = sm(0x48415045 + 16*cfg + stream);
                stream 0 = R keys, 1 = S index map, 2 = R payloads,
                3 = S payloads.
  payloads    : low bits of sm(sub ^ row) (independent of the key).

Every formula is written once against a tiny array-ops shim so that it runs
on numpy uint64 arrays (host) and on torch int64 tensors (any device, e.g. to
generate 2^30-row relations directly in HBM).  Both backends produce the same
bits; ``tests/test_datagen.py`` pins that.
"""
from __future__ import annotations

import dataclasses
import math
from typing import Optional

import numpy as np

GOLDEN = 0x9E3779B97F4A7C15
BASE_SEED = 0x48415045  # "HAPE"
_M64 = (1 << 64) - 1

CONFIG_IDS = {"c1": 1, "c2": 2, "c3": 3, "c4": 4, "c5": 5, "dup": 6, "ragged": 7}


# --------------------------------------------------------------------------
# scalar (python int) helpers -- used for seeds
# --------------------------------------------------------------------------
def sm_scalar(x: int) -> int:
    z = (x + GOLDEN) & _M64
    z = ((z ^ (z >> 30)) * 0xBF58476D1CE4E5B9) & _M64
    z = ((z ^ (z >> 27)) * 0x94D049BB133111EB) & _M64
    return z ^ (z >> 31)


def sub_seed(config: str, stream: int) -> int:
    return sm_scalar(BASE_SEED + 16 * CONFIG_IDS[config] + stream)


# --------------------------------------------------------------------------
# array backends: numpy uint64 / torch int64 (two's complement wrap)
# --------------------------------------------------------------------------
class _NP:
    name = "numpy"

    @staticmethod
    def const(c):
        return np.uint64(c & _M64)

    @staticmethod
    def arange(lo, hi, device=None):
        return np.arange(lo, hi, dtype=np.uint64)

    @staticmethod
    def lsr(x, k):
        return x >> np.uint64(k)

    @staticmethod
    def mask(x, w):
        return x & np.uint64((1 << w) - 1) if w < 64 else x


class _TORCH:
    name = "torch"

    @staticmethod
    def const(c):
        c &= _M64
        return c - (1 << 64) if c >= (1 << 63) else c

    @staticmethod
    def arange(lo, hi, device=None):
        import torch
        return torch.arange(lo, hi, dtype=torch.int64, device=device)

    @staticmethod
    def lsr(x, k):
        # logical shift right on int64 bit patterns
        if k == 0:
            return x
        return (x >> k) & ((1 << (64 - k)) - 1)

    @staticmethod
    def mask(x, w):
        return x & ((1 << w) - 1) if w < 63 else (x if w == 64 else x & ((1 << w) - 1))


def _ops(backend):
    return _TORCH if backend == "torch" else _NP


def sm(x, ops=_NP):
    """splitmix64 output for state(s) x (array)."""
    z = x + ops.const(GOLDEN)
    z = (z ^ ops.lsr(z, 30)) * ops.const(0xBF58476D1CE4E5B9)
    z = (z ^ ops.lsr(z, 27)) * ops.const(0x94D049BB133111EB)
    return z ^ ops.lsr(z, 31)


def _perm_pow2(x, w, seed, ops=_NP):
    sh = (w + 1) // 2
    for r in range(3):
        a = (sm_scalar(seed + r) | 1) & ((1 << w) - 1)
        c = sm_scalar(seed + r + 256) & ((1 << w) - 1)
        x = ops.mask(x * ops.const(a) + ops.const(c), w)
        x = x ^ ops.lsr(x, sh)
    return x


def perm(x, n: int, seed: int, ops=_NP):
    """Seeded bijection of [0, n) applied to the array x (values in [0, n))."""
    if n <= 1:
        return x * 0
    w = max(1, math.ceil(math.log2(n)))
    y = _perm_pow2(x, w, seed, ops)
    if n == (1 << w):
        return y
    # cycle-walking keeps it a bijection of [0, n)
    while True:
        bad = y >= ops.const(n) if ops is _NP else (y >= n)
        if not bool(bad.any()):
            return y
        y2 = _perm_pow2(y, w, seed, ops)
        if ops is _NP:
            y = np.where(bad, y2, y)
        else:
            import torch
            y = torch.where(bad, y2, y)


def _cast(x, dtype_bits: int, ops):
    """Reinterpret the low dtype_bits of uint64/int64 array x as a signed int."""
    if ops is _NP:
        if dtype_bits == 32:
            return (x & np.uint64(0xFFFFFFFF)).astype(np.uint32).view(np.int32)
        return x.view(np.int64)
    import torch
    if dtype_bits == 32:
        lo = x & 0xFFFFFFFF
        return torch.where(lo >= (1 << 31), lo - (1 << 32), lo).to(torch.int32)
    return x


# --------------------------------------------------------------------------
# workloads
# --------------------------------------------------------------------------
@dataclasses.dataclass
class Relation:
    key: object        # np.ndarray or torch.Tensor (int32 / int64)
    payload: object

    @property
    def n(self) -> int:
        return int(self.key.shape[0])


@dataclasses.dataclass
class Workload:
    name: str
    R: Relation
    S: Relation
    idx: Optional[object]   # provenance: S row j copies R row idx[j] (global R row id)
    n_r_global: int
    n_s_global: int
    key_bits: int
    pay_bits: int
    kind: str               # "pkfk-dense" | "fk-uniform" | "zipf" | "dup"


SHAPES = {
    # name: (n_r, n_s, key_bits, pay_bits, kind)
    "c1": (1 << 20, 1 << 20, 32, 32, "pkfk-dense"),
    "c2": (1 << 27, 1 << 27, 32, 32, "pkfk-dense"),
    "c3": (1 << 27, 1 << 30, 64, 64, "fk-uniform"),
    "c4": (1 << 31, 1 << 31, 32, 32, "pkfk-dense"),
    "c5": (1 << 28, 1 << 30, 32, 32, "zipf"),
}


def _rows(n: int, rank: int, world: int):
    return (n * rank) // world, (n * (rank + 1)) // world


def make(config: str, n_r: Optional[int] = None, n_s: Optional[int] = None,
         rank: int = 0, world: int = 1, backend: str = "numpy",
         device=None, key_bits: Optional[int] = None,
         pay_bits: Optional[int] = None, theta: float = 1.0,
         dup_domain: Optional[int] = None) -> Workload:
    """Generate rank `rank`'s contiguous row shard of config `config`.

    `n_r`/`n_s` override the config's sizes (the recipe is unchanged), which
    is how tests run the BASELINE recipes at oracle-friendly sizes with
    ragged tails.  `backend` is "numpy" (host) or "torch" (any device)."""
    shape = SHAPES.get(config)
    if config == "dup":
        shape = (1 << 12, 1 << 12, 32, 32, "dup")
    if config == "ragged":
        shape = (1000, 1000, 32, 32, "pkfk-dense")
    if shape is None:
        raise ValueError(f"unknown config {config}")
    NR = n_r if n_r is not None else shape[0]
    NS = n_s if n_s is not None else shape[1]
    kb = key_bits or shape[2]
    pb = pay_bits or shape[3]
    kind = shape[4]
    ops = _ops(backend)
    s0, s1, s2, s3 = (sub_seed(config, k) for k in range(4))

    r_lo, r_hi = _rows(NR, rank, world)
    s_lo, s_hi = _rows(NS, rank, world)
    i = ops.arange(r_lo, r_hi, device)
    j = ops.arange(s_lo, s_hi, device)

    def r_key_of(rows):
        if kind in ("pkfk-dense", "zipf"):
            return perm(rows, NR, s0, ops)              # dense key set [0, NR)
        if kind == "fk-uniform":
            return sm(rows ^ ops.const(s0), ops)         # unique 64-bit keys
        if kind == "dup":
            D = dup_domain or 64
            return _signed_small(sm(rows ^ ops.const(s0), ops), D, ops)
        raise AssertionError(kind)

    rk = r_key_of(i)
    if kind == "pkfk-dense":
        if NS == NR:
            idx = perm(j, NR, s1, ops)                   # same key set, other order
        else:
            idx = _uniform_idx(j, NR, s1, ops)
    elif kind == "fk-uniform":
        idx = _uniform_idx(j, NR, s1, ops)
    elif kind == "zipf":
        idx = _zipf_idx(j, NR, theta, s1, ops)
    elif kind == "dup":
        idx = None
    if kind == "dup":
        D = dup_domain or 64
        sk = _signed_small(sm(j ^ ops.const(s1), ops), D, ops)
    else:
        sk = r_key_of(idx)
    rp = sm(i ^ ops.const(s2), ops)
    sp = sm(j ^ ops.const(s3), ops)
    R = Relation(_cast(rk, kb, ops), _cast(rp, pb, ops))
    S = Relation(_cast(sk, kb, ops), _cast(sp, pb, ops))
    return Workload(config, R, S, idx, NR, NS, kb, pb, kind)


def _uniform_idx(j, n, seed, ops):
    """idx_j = floor(hi32(sm(seed + j)) * n / 2^32), uniform with replacement."""
    hi = ops.lsr(sm(j + ops.const(seed), ops), 32)
    if n <= (1 << 32):
        return ops.lsr(hi * ops.const(n), 32)
    raise ValueError("n too large for _uniform_idx")


def _signed_small(x, D, ops):
    """Map a uint64 draw to [-D/2, D/2) (duplicate-heavy keys incl. negatives)."""
    v = x % ops.const(D) if ops is _NP else _torch_umod(x, D)
    if ops is _NP:
        return (v.view(np.int64) - np.int64(D // 2)).view(np.uint64)
    return v - D // 2


def _torch_umod(x, D):
    # unsigned 64-bit modulo for int64 bit patterns (D < 2^31)
    hi = (x >> 32) & 0xFFFFFFFF
    lo = x & 0xFFFFFFFF
    return ((hi % D) * ((1 << 32) % D) + lo) % D


def _zipf_idx(j, n, theta, seed, ops):
    """Zipf(theta) rank r in [1, n] by inverse CDF of the continuous
    approximation H(x) = (x^(1-theta) - 1)/(1-theta) (theta != 1) or ln x,
    with the first 2^16 ranks tabulated exactly; returns r - 1.  Deterministic
    in (j, seed).  Used for the C5 skew recipe (BASELINE.json configs[4])."""
    u_raw = ops.lsr(sm(j + ops.const(seed), ops), 11)   # 53-bit uniform
    if ops is _NP:
        u = u_raw.astype(np.float64) / float(1 << 53)
        xp = np
    else:
        import torch
        u = u_raw.to(torch.float64) / float(1 << 53)
        xp = torch
    T = min(n, 1 << 16)
    ks = np.arange(1, T + 1, dtype=np.float64)
    head = np.cumsum(ks ** (-theta))

    def Hc(x):  # continuous tail mass from T+0.5 to x+0.5
        a, b = T + 0.5, x + 0.5
        if theta == 1.0:
            return math.log(b / a)
        return (b ** (1 - theta) - a ** (1 - theta)) / (1 - theta)

    tail_total = Hc(n) if n > T else 0.0
    total = head[-1] + tail_total
    target = u * total
    if ops is _NP:
        r_head = np.searchsorted(head, target, side="right")  # 0-based rank
        t = np.maximum(target - head[-1], 0.0)
    else:
        import torch
        head_t = torch.as_tensor(head, device=u.device)
        r_head = torch.searchsorted(head_t, target, right=True)
        t = torch.clamp(target - head[-1], min=0.0)
    a = T + 0.5
    if theta == 1.0:
        x = a * xp.exp(t) - 0.5
    else:
        x = (t * (1 - theta) + a ** (1 - theta)) ** (1.0 / (1 - theta)) - 0.5
    if ops is _NP:
        r_tail = np.clip(np.floor(x), T, n - 1).astype(np.uint64)
        return np.where(r_head < T, r_head.astype(np.uint64), r_tail)
    import torch
    r_tail = torch.clamp(torch.floor(x), T, n - 1).to(torch.int64)
    return torch.where(r_head < T, r_head.to(torch.int64), r_tail)
