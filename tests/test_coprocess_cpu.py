"""CPU checks of the co-processing join's host step (hape_host_partition,
PAPER.md §5 P717-737: "a first partitioning step locally to the input").

The step is integer and stable, so it is compared bit-exactly with the
oracle's definition of the owner bits (oracle/partition.py: the top
fanout_bits bits of h, R14) applied by a stable sort.
"""
import ctypes

import numpy as np
import pytest
import torch

from oracle import partition as opart
from paper_conf_cidr_chrysogelossa19_b200 import HapeError, _lib, host_partition


def _expected(k, p, fb, identity=False):
    d = opart.destination(k, 1 << fb, identity) if fb else np.zeros(len(k), np.int64)
    o = np.argsort(d, kind="stable")
    b = np.concatenate([[0], np.cumsum(np.bincount(d, minlength=1 << fb))]).astype(np.int64)
    return k[o], p[o], b


@pytest.mark.parametrize("kdt,pdt", [(np.int32, np.int32), (np.int32, np.int64), (np.int64, np.int32),
                                     (np.int64, np.int64)])
@pytest.mark.parametrize("fb", [0, 1, 4, 10])
@pytest.mark.parametrize("threads", [1, 3, 0])
def test_host_partition_matches_oracle(kdt, pdt, fb, threads):
    rng = np.random.default_rng(fb * 31 + threads + (kdt == np.int64) * 7 + (pdt == np.int64) * 3)
    n = 200_003
    k = rng.integers(np.iinfo(kdt).min, np.iinfo(kdt).max, size=n, dtype=kdt)
    p = rng.integers(-2**31, 2**31, size=n).astype(pdt)
    ok, op, b = host_partition(torch.from_numpy(k), torch.from_numpy(p), fb, threads=threads)
    ek, ep, eb = _expected(k, p, fb)
    assert np.array_equal(ok.numpy(), ek) and np.array_equal(op.numpy(), ep)
    assert np.array_equal(b.numpy(), eb)


@pytest.mark.parametrize("n", [0, 1, 5, 65537])
def test_host_partition_small_and_ragged(n):
    rng = np.random.default_rng(n)
    k = rng.integers(-50, 50, size=n).astype(np.int32)  # heavy duplicates: equal keys stay together
    p = np.arange(n, dtype=np.int32)
    ok, op, b = host_partition(torch.from_numpy(k), torch.from_numpy(p), 3, threads=4)
    ek, ep, eb = _expected(k, p, 3)
    assert np.array_equal(ok.numpy(), ek) and np.array_equal(op.numpy(), ep) and np.array_equal(b.numpy(), eb)


def test_host_partition_identity_reads_top_key_bits():
    k = np.arange(1 << 12, dtype=np.int64) << 52  # identity h: the top 12 bits are the row index
    p = np.arange(1 << 12, dtype=np.int64)
    ok, op, b = host_partition(torch.from_numpy(k), torch.from_numpy(p), 4, identity=True)
    assert np.array_equal(np.diff(b.numpy()), np.full(16, 256))  # dense keys: equal partitions (P802-804)
    ek, ep, eb = _expected(k, p, 4, identity=True)
    assert np.array_equal(ok.numpy(), ek) and np.array_equal(b.numpy(), eb)


def test_host_partition_rejects_bad_args():
    k = torch.zeros(8, dtype=torch.int32)
    with pytest.raises(HapeError):
        host_partition(k, k.clone(), 17)
    rel = _lib.hape_relation(k.data_ptr(), k.data_ptr(), 8, _lib.HAPE_MEM_DEVICE)
    b = (ctypes.c_uint64 * 3)()
    assert _lib.hape_host_partition(rel, 0, 0, 0, 1, 0, k.data_ptr(), k.data_ptr(), b) == _lib.HAPE_ERR_INVALID_ARG
    rel = _lib.hape_relation(k.data_ptr(), None, 8, _lib.HAPE_MEM_HOST)
    assert _lib.hape_host_partition(rel, 0, 0, 0, 1, 0, k.data_ptr(), k.data_ptr(), b) == _lib.HAPE_ERR_INVALID_ARG


def test_coprocess_rejects_without_gpu_work():
    """Argument errors surface before any device work (NULL handle / result)."""
    assert _lib.lib.hape_coprocess_join(None, None, None, None, None, None) == _lib.HAPE_ERR_INVALID_ARG


@pytest.mark.parametrize("shift", [1, 3, 5])
def test_host_partition_unaligned_outputs(shift):
    """Output columns that do not start on a 64-byte line (the write-combining
    path's slot arithmetic) give the same stable partition."""
    rng = np.random.default_rng(shift)
    n = 100_001
    k = rng.integers(-2**31, 2**31, size=n).astype(np.int32)
    p = rng.integers(-2**40, 2**40, size=n).astype(np.int64)
    ok = np.zeros(n + 16, np.int32)
    op = np.zeros(n + 16, np.int64)
    rel = _lib.hape_relation(k.ctypes.data, p.ctypes.data, n, _lib.HAPE_MEM_HOST)
    b = (ctypes.c_uint64 * 9)()
    st = _lib.hape_host_partition(rel, _lib.HAPE_INT32, _lib.HAPE_INT64, _lib.HAPE_PART_HASH, 3, 6,
                                  ok.ctypes.data + 4 * shift, op.ctypes.data + 8 * shift, b)
    assert st == _lib.HAPE_OK
    ek, ep, eb = _expected(k, p, 3)
    assert np.array_equal(ok[shift:shift + n], ek) and np.array_equal(op[shift:shift + n], ep)
    assert not ok[:shift].any() and not ok[shift + n:].any() and not op[shift + n:].any()
    assert np.array_equal(np.array(list(b)), eb)


@pytest.mark.parametrize("n", [1, 3, 9, 40])
def test_host_partition_unaligned_tiny(n):
    k = np.arange(n, dtype=np.int64) * 977 - 5
    p = np.arange(n, dtype=np.int64)
    ok = np.zeros(n + 8, np.int64)
    op = np.zeros(n + 8, np.int64)
    rel = _lib.hape_relation(k.ctypes.data, p.ctypes.data, n, _lib.HAPE_MEM_HOST)
    b = (ctypes.c_uint64 * 5)()
    assert _lib.hape_host_partition(rel, _lib.HAPE_INT64, _lib.HAPE_INT64, _lib.HAPE_PART_HASH, 2, 2,
                                    ok.ctypes.data + 40, op.ctypes.data + 24, b) == _lib.HAPE_OK
    ek, ep, _ = _expected(k, p, 2)
    assert np.array_equal(ok[5:5 + n], ek) and np.array_equal(op[3:3 + n], ep)
