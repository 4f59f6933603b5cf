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
