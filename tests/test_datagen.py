"""Input generator checks (-m "not gpu"): determinism, bijectivity, backend
agreement (numpy host vs torch), recipe shapes of BASELINE.json configs."""
import numpy as np
import pytest
import torch

import datagen
from oracle import partition


@pytest.mark.parametrize("n", [1, 2, 3, 1000, 1 << 12, (1 << 12) + 5])
def test_perm_is_bijection(n):
    x = datagen.perm(np.arange(n, dtype=np.uint64), n, 12345)
    assert np.array_equal(np.sort(x), np.arange(n, dtype=np.uint64))


@pytest.mark.parametrize("cfg,nr,ns", [("c1", 1 << 12, 1 << 12), ("c1", 1001, 1001),
                                       ("c3", 1 << 10, 1 << 12), ("c5", 1 << 10, 1 << 12),
                                       ("dup", 300, 500)])
def test_numpy_torch_backends_agree(cfg, nr, ns):
    a = datagen.make(cfg, n_r=nr, n_s=ns)
    b = datagen.make(cfg, n_r=nr, n_s=ns, backend="torch")
    for x, y in ((a.R.key, b.R.key), (a.R.payload, b.R.payload), (a.S.key, b.S.key),
                 (a.S.payload, b.S.payload)):
        assert x.dtype == y.numpy().dtype
        assert np.array_equal(x, y.numpy())
    if a.idx is not None:
        assert np.array_equal(a.idx.astype(np.int64), b.idx.numpy())


def test_dense_pkfk_same_key_set():
    wl = datagen.make("c1", n_r=1 << 14, n_s=1 << 14)
    assert np.array_equal(np.sort(wl.R.key), np.arange(1 << 14, dtype=np.int32))
    assert np.array_equal(np.sort(wl.S.key), np.arange(1 << 14, dtype=np.int32))
    assert np.array_equal(wl.S.key, wl.R.key[wl.idx.astype(np.int64)])


def test_sharding_concatenates_to_global():
    full = datagen.make("c1", n_r=1 << 12, n_s=1 << 12)
    parts = [datagen.make("c1", n_r=1 << 12, n_s=1 << 12, rank=r, world=4) for r in range(4)]
    assert np.array_equal(np.concatenate([p.R.key for p in parts]), full.R.key)
    assert np.array_equal(np.concatenate([p.S.payload for p in parts]), full.S.payload)
    assert np.array_equal(np.concatenate([p.idx for p in parts]), full.idx)


def test_c3_keys_unique_and_signed():
    wl = datagen.make("c3", n_r=1 << 14, n_s=1 << 15)
    assert wl.R.key.dtype == np.int64
    assert len(np.unique(wl.R.key)) == 1 << 14
    assert (wl.R.key < 0).any() and (wl.R.key > 0).any()
    assert wl.idx.max() < (1 << 14)


def test_zipf_skew_monotone():
    lo = datagen.make("c5", n_r=1 << 16, n_s=1 << 18, theta=0.5)
    hi = datagen.make("c5", n_r=1 << 16, n_s=1 << 18, theta=1.0)
    top = lambda w: np.bincount(w.idx.astype(np.int64)).max()
    assert top(hi) > 10 * top(lo)
    # rank 0 is the most frequent under theta = 1
    c = np.bincount(hi.idx.astype(np.int64))
    assert c.argmax() == 0


def test_hash_is_bijective_on_sample():
    x = np.arange(-(1 << 19), 1 << 19, dtype=np.int32)
    assert len(np.unique(partition.fmix32(x))) == len(x)
    y = np.arange(1 << 18, dtype=np.int64) * 0x1_0000_0001
    assert len(np.unique(partition.fmix64(y))) == len(y)
