"""C-ABI checks that need no GPU (-m "not gpu"): the library builds and loads,
exports every function include/hape.h declares, and its host-only logic
(status strings, argument validation, the all-to-allv exchange plan) is
right.  No compute call is made here."""
import ctypes
import os
import re
import subprocess

import numpy as np
import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def lib():
    from paper_conf_cidr_chrysogelossa19_b200 import build
    build.build()
    from paper_conf_cidr_chrysogelossa19_b200 import _lib
    return _lib


def declared_functions():
    hdr = open(os.path.join(ROOT, "include", "hape.h")).read()
    hdr = re.sub(r"/\*.*?\*/", "", hdr, flags=re.S)
    return sorted(set(re.findall(r"\b(hape_[a-z0-9_]+)\s*\(", hdr)))


def test_every_declared_symbol_is_exported(lib):
    names = declared_functions()
    assert len(names) >= 12
    out = subprocess.run(["nm", "-D", "--defined-only", lib.LIB_PATH], capture_output=True, text=True).stdout
    exported = set(l.split()[-1] for l in out.splitlines() if " T " in l)
    missing = [n for n in names if n not in exported]
    assert not missing, missing
    assert set(names) == set(lib.EXPORTED)
    for n in names:
        assert hasattr(lib.lib, n)


def test_sm100a_code_present(lib):
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", lib.LIB_PATH],
                         capture_output=True, text=True).stdout
    assert "sm_100a" in out


def test_status_strings(lib):
    assert lib.hape_status_string(0) == "HAPE_OK"
    assert lib.hape_status_string(4) == "HAPE_ERR_OUTPUT_CAPACITY"
    assert lib.hape_status_string(99) == "HAPE_ERR_UNKNOWN"
    assert "sm_100a" in lib.hape_version()


def test_create_rejects_bad_config_without_touching_cuda(lib):
    for field, val in (("key_type", 7), ("radix_passes", 3), ("part_fn", 5), ("world_size", 3),
                       ("world_size", 128), ("device", -1), ("flags", 4)):
        cfg = lib.hape_join_config()
        setattr(cfg, field, val)
        st, h = lib.hape_join_create(cfg)
        assert st == lib.HAPE_ERR_INVALID_ARG, field
        assert not h.value
    cfg = lib.hape_join_config()
    cfg.world_size, cfg.rank = 2, 0  # no communicator
    assert lib.hape_join_create(cfg)[0] == lib.HAPE_ERR_INVALID_ARG
    cfg = lib.hape_join_config()
    cfg.radix_bits[0] = 13
    assert lib.hape_join_create(cfg)[0] == lib.HAPE_ERR_INVALID_ARG


def test_null_handle_paths(lib):
    assert lib.hape_join_destroy(None) == lib.HAPE_OK
    res = lib.hape_join_result()
    R = lib.hape_relation()
    assert lib.lib.hape_radix_join(None, ctypes.byref(R), ctypes.byref(R), None, ctypes.byref(res)) == \
        lib.HAPE_ERR_INVALID_ARG
    assert lib.lib.hape_join_plan(None, 1, 1, None) == lib.HAPE_ERR_INVALID_ARG


@pytest.mark.parametrize("G", [1, 2, 4, 8])
def test_exchange_plan_matches_definition(lib, G):
    rng = np.random.default_rng(G)
    counts = rng.integers(0, 1000, (G, G))
    for me in range(G):
        st, so, ro, rt = lib.hape_exchange_plan(G, me, counts.reshape(-1).tolist())
        assert st == lib.HAPE_OK
        assert so == np.concatenate([[0], np.cumsum(counts[me])[:-1]]).tolist()
        assert ro == np.concatenate([[0], np.cumsum(counts[:, me])[:-1]]).tolist()
        assert rt == int(counts[:, me].sum())
    assert lib.hape_exchange_plan(G, G, counts.reshape(-1).tolist())[0] == lib.HAPE_ERR_INVALID_ARG


@pytest.mark.parametrize("G", [1, 2, 3, 8, 64])
def test_peer_plan_tiles_every_receive_buffer(lib, G):
    """hape_peer_plan (the fused exchange's addressing): the G sources'
    segments tile each destination's receive buffer [0, total) exactly, in
    rank order, and the capacity is the largest receive total."""
    rng = np.random.default_rng(100 + G)
    counts = rng.integers(0, 1000, (G, G))
    counts[0, :] = 0                                  # a rank that sends nothing
    offs = []
    for me in range(G):
        st, wo, rt, cap = lib.hape_peer_plan(G, me, counts.reshape(-1).tolist())
        assert st == lib.HAPE_OK
        assert rt == int(counts[:, me].sum()) and cap == int(counts.sum(axis=0).max())
        offs.append(wo)
    for d in range(G):
        cover = np.zeros(int(counts[:, d].sum()), np.int64)
        for src in range(G):
            o, c = offs[src][d], int(counts[src, d])
            assert o == int(counts[:src, d].sum())
            cover[o:o + c] += 1
        assert (cover == 1).all()
    assert lib.hape_peer_plan(G, G, counts.reshape(-1).tolist())[0] == lib.HAPE_ERR_INVALID_ARG
