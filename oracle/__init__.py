"""CPU oracle for the HAPE radix-join hot path -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.  The
product path (``paper_conf_cidr_chrysogelossa19_b200``) never imports it and
shares no code with it (no kernels, headers, helpers, constant tables).

Contents
  join(...)        -- oracle.c: single-threaded sort-merge computing the plain
                      definition of the §6.2 micro-benchmark result
                      (PAPER.md P789-794), see oracle.c's header.
  join_sharded(...) -- the same oracle on T host threads:
                      R and S split by key into T shards (equal keys share a
                      shard), one oracle.c join per shard, sums mod 2^64.
  mix / fmix64     -- numpy re-statement of the pair-checksum term (DESIGN.md
                      reading R10); pinned by published splitmix64 vectors.
  partition.py     -- the partition function h and its bit fields (DESIGN.md
                      R1/R3), for the stage-invariant tests.
  provenance.py    -- expected results for PK-FK workloads derived from the
                      generator's provenance (no join), SURVEY §8.c.4.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from typing import Optional

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_lib = None


def build(force: bool = False) -> str:
    """Compile oracle.c with gcc (plain C, -O2, single-threaded)."""
    src = os.path.join(_HERE, "oracle.c")
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(src):
        tmp = _LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-shared", "-fPIC", "-o", tmp, src])
        os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def _load():
    global _lib
    if _lib is None:
        build()
        lib = ctypes.CDLL(_LIB_PATH)
        lib.oracle_join.restype = ctypes.c_int
        lib.oracle_join.argtypes = [
            ctypes.c_int,
            ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int, ctypes.c_uint64,
            ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int, ctypes.c_uint64,
            ctypes.POINTER(ctypes.c_uint64),
            ctypes.c_void_p, ctypes.c_void_p, ctypes.c_uint64,
            ctypes.POINTER(ctypes.c_uint64)]
        lib.oracle_mix.restype = ctypes.c_uint64
        lib.oracle_mix.argtypes = [ctypes.c_int64, ctypes.c_int64]
        lib.oracle_fmix64_export.restype = ctypes.c_uint64
        lib.oracle_fmix64_export.argtypes = [ctypes.c_uint64]
        _lib = lib
    return _lib


def _np(a):
    if hasattr(a, "detach"):  # torch tensor
        a = a.detach().cpu().numpy()
    return np.ascontiguousarray(a)


def join(rk, rp, sk, sp, materialize: bool = False) -> dict:
    """Run the C sort-merge oracle.  Inputs: 1-D int32/int64 arrays (numpy or
    torch; copied to host).  Returns dict(count, sum_r, sum_s, checksum[, pairs])
    with u64 python ints; pairs = (p_r, p_s) int64 arrays sorted
    lexicographically."""
    lib = _load()
    rk, rp, sk, sp = (_np(x) for x in (rk, rp, sk, sp))
    assert rk.dtype == sk.dtype and rk.dtype in (np.int32, np.int64)
    for x in (rp, sp):
        assert x.dtype in (np.int32, np.int64)
    assert rk.shape == rp.shape and sk.shape == sp.shape
    out = (ctypes.c_uint64 * 4)()
    npairs = ctypes.c_uint64(0)
    pr = ps = None
    cap = 0
    if materialize:
        # first pass: count only
        rc = lib.oracle_join(rk.itemsize, rk.ctypes.data, rp.ctypes.data, rp.itemsize, rk.size,
                             sk.ctypes.data, sp.ctypes.data, sp.itemsize, sk.size,
                             out, None, None, 0, ctypes.byref(npairs))
        if rc != 0:
            raise MemoryError("oracle_join failed")
        cap = int(npairs.value)
        pr = np.empty(max(cap, 1), np.int64)
        ps = np.empty(max(cap, 1), np.int64)
    rc = lib.oracle_join(rk.itemsize, rk.ctypes.data, rp.ctypes.data, rp.itemsize, rk.size,
                         sk.ctypes.data, sp.ctypes.data, sp.itemsize, sk.size,
                         out, pr.ctypes.data if materialize else None,
                         ps.ctypes.data if materialize else None, cap, ctypes.byref(npairs))
    if rc != 0:
        raise MemoryError("oracle_join failed")
    res = dict(count=int(out[0]), sum_r=int(out[1]), sum_s=int(out[2]), checksum=int(out[3]))
    if materialize:
        res["pairs"] = (pr[:cap], ps[:cap])
    return res


def mix_scalar(p: int, q: int) -> int:
    """pair-checksum term via the C oracle (scalar)."""
    return int(_load().oracle_mix(int(p), int(q)))


def fmix64_scalar(x: int) -> int:
    return int(_load().oracle_fmix64_export(x & ((1 << 64) - 1)))


# ---- numpy re-statement (vectorised) ------------------------------------
_U = np.uint64


def fmix64(x: np.ndarray) -> np.ndarray:
    """splitmix64 finaliser on uint64 arrays."""
    x = x.astype(np.uint64, copy=True)
    x ^= x >> _U(30); x *= _U(0xBF58476D1CE4E5B9)
    x ^= x >> _U(27); x *= _U(0x94D049BB133111EB)
    x ^= x >> _U(31)
    return x


def mix(p: np.ndarray, q: np.ndarray) -> np.ndarray:
    """mix(p, q) = fmix64((u64)p * 0x9E3779B97F4A7C15 + (u64)q),
    p and q sign-extended to 64 bits first (R10)."""
    pu = np.asarray(p).astype(np.int64).view(np.uint64)
    qu = np.asarray(q).astype(np.int64).view(np.uint64)
    with np.errstate(over="ignore"):
        return fmix64(pu * _U(0x9E3779B97F4A7C15) + qu)


def u64sum(x: np.ndarray) -> int:
    """sum mod 2^64 of a uint64 (or sign-extended int) array."""
    x = np.asarray(x)
    if x.dtype != np.uint64:
        x = x.astype(np.int64).view(np.uint64)
    return int(np.add.reduce(x, dtype=np.uint64))


def threads_used() -> int:
    return 1


def host_cores() -> int:
    try:
        return len(os.sched_getaffinity(0))
    except Exception:
        return os.cpu_count() or 1


def join_sharded(rk, rp, sk, sp, threads: int = 0) -> dict:
    """SURVEY §8.d.6's T-core variant of the oracle (count and sums only):
    shard s gets the tuples whose key k has (k mod T) == s -- a plain
    function of the key, so equal keys meet in one shard and the shard
    results add up to the whole join -- and each shard runs join() on its
    own thread (the C call releases the GIL).  T = host cores by default."""
    from concurrent.futures import ThreadPoolExecutor
    T = threads or host_cores()
    rk, rp, sk, sp = (_np(x) for x in (rk, rp, sk, sp))

    def shard(i):
        # every thread selects its own shard (numpy releases the GIL on the
        # array passes, so the selection runs in parallel too)
        if T == 1:
            return join(rk, rp, sk, sp)
        mr = (rk.astype(np.int64) % T) == i
        ms = (sk.astype(np.int64) % T) == i
        return join(rk[mr], rp[mr], sk[ms], sp[ms])

    with ThreadPoolExecutor(max_workers=T) as ex:
        parts = list(ex.map(shard, range(T)))
    M = (1 << 64) - 1
    return dict(count=sum(p["count"] for p in parts), sum_r=sum(p["sum_r"] for p in parts) & M,
                sum_s=sum(p["sum_s"] for p in parts) & M, checksum=sum(p["checksum"] for p in parts) & M,
                threads=T)
