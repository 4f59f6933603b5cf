"""The device-partition + NCCL exchange path (a2-a5) on one GPU: a 1-rank
communicator makes hape_radix_join route every tuple through the destination
partition kernels, the count all-gather, the grouped send/recv and the
allreduce, then join what it received.  Parity vs the oracle, bit-exact."""
import numpy as np
import pytest
import torch

import datagen
import oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin, _lib


@pytest.fixture(scope="module")
def comm():
    uid = _lib.hape_nccl_unique_id()
    st, c = _lib.hape_nccl_comm_init(uid, 1, 0, 0)
    assert st == _lib.HAPE_OK
    yield c
    _lib.hape_nccl_comm_destroy(c)


@pytest.mark.parametrize("cfg,nr,ns", [("c1", 1 << 18, (1 << 18) + 7), ("c3", 1 << 16, 1 << 18),
                                       ("dup", 5000, 7000)])
def test_one_rank_exchange_vs_oracle(comm, cfg, nr, ns):
    kw = dict(dup_domain=50) if cfg == "dup" else {}
    wl = datagen.make(cfg, n_r=nr, n_s=ns, **kw)
    kdt = torch.int32 if wl.key_bits == 32 else torch.int64
    want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
    with RadixJoin(key_dtype=kdt, world_size=1, rank=0, nccl_comm=comm) as j:
        res = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
    got = dict(count=res.match_count, sum_r=res.sum_r_payload, sum_s=res.sum_s_payload,
               checksum=res.pair_checksum)
    assert got == want
    assert res.local_match_count == res.match_count
    assert res.r_local == nr and res.s_local == ns
    assert res.stage_ms["devpart"] > 0 and res.stage_ms["exchange"] > 0
    assert res.exchange_path == 2    # the fused peer scatter (own buffer as the one peer)
    # repeated calls reuse the mapped receive buffers
    res2 = None
    with RadixJoin(key_dtype=kdt, world_size=1, rank=0, nccl_comm=comm) as j:
        for _ in range(2):
            res2 = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
    assert res2.as_tuple() == res.as_tuple()


def test_one_rank_exchange_nccl_form(comm):
    """HAPE_XCHG=nccl: the send-buffer + ncclSend/ncclRecv form (child process)."""
    import os, subprocess, sys
    code = r'''
import numpy as np, torch, datagen, oracle
from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin, _lib
uid = _lib.hape_nccl_unique_id(); st, c = _lib.hape_nccl_comm_init(uid, 1, 0, 0)
wl = datagen.make("dup", n_r=5000, n_s=7000, dup_domain=50)
want = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
with RadixJoin(key_dtype=torch.int32, world_size=1, rank=0, nccl_comm=c) as j:
    r = j.join(d(wl.R.key), d(wl.R.payload), d(wl.S.key), d(wl.S.payload))
assert r.exchange_path == 1, r.exchange_path
assert (r.match_count, r.sum_r_payload, r.sum_s_payload, r.pair_checksum) == (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
_lib.hape_nccl_comm_destroy(c)
print("ok")
'''
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, "-c", code], cwd=root, capture_output=True, text=True, timeout=600,
                       env=dict(os.environ, HAPE_XCHG="nccl", PYTHONPATH=root))
    assert r.returncode == 0 and "ok" in r.stdout, r.stdout + r.stderr
