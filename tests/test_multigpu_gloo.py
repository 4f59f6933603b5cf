"""The N>1 path on CPU (world_size 2 and 4, gloo): the library's host-side
exchange plan (NCCL send/recv form: hape_exchange_plan; fused peer-scatter
form: hape_peer_plan, each rank writing its segment into every destination's
receive buffer at its own offset) drives an all-to-allv of hash-routed
shards, every rank joins
what it received with the oracle, and the summed rank results must equal the
oracle on the whole input -- the co-location argument of DESIGN.md R14
(destination = top log2(G) bits of h, so equal keys meet on one rank).  The
device kernels of the same path run on the GPU in test_gpu_exchange.py."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import datagen
import oracle
from oracle import partition

M64 = (1 << 64) - 1


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _route(keys, pays, world, rank, lib):
    dest = partition.destination(keys, world)
    counts = np.bincount(dest, minlength=world).astype(np.int64)
    mat = torch.zeros(world, world, dtype=torch.int64)
    gathered = [torch.zeros(world, dtype=torch.int64) for _ in range(world)]
    dist.all_gather(gathered, torch.from_numpy(counts))
    mat = torch.stack(gathered).numpy()
    st, soff, roff, rtot = lib.hape_exchange_plan(world, rank, mat.reshape(-1).tolist())
    assert st == 0
    order = np.argsort(dest, kind="stable")
    assert soff == np.concatenate([[0], np.cumsum(counts)[:-1]]).tolist()
    out = []
    for col in (keys, pays):
        send = torch.from_numpy(np.ascontiguousarray(col[order]).astype(np.int64))
        recv = torch.empty(rtot, dtype=torch.int64)
        dist.all_to_all_single(recv, send, output_split_sizes=mat[:, rank].tolist(),
                               input_split_sizes=mat[rank].tolist())
        out.append(recv.numpy().astype(col.dtype))
    # every received tuple is owned by this rank; segments sit at roff
    assert (partition.destination(out[0], world) == rank).all()
    assert roff[-1] + mat[world - 1, rank] == rtot
    return out


def _route_peer(keys, pays, world, rank, lib):
    """The fused form's addressing: rank r writes its destination-d segment
    at hape_peer_plan's write_off[d] inside d's receive buffer, sized to the
    common capacity.  Simulated with gloo: the segments travel with their
    offsets, the destination places them and checks they tile [0, total)."""
    dest = partition.destination(keys, world)
    counts = np.bincount(dest, minlength=world).astype(np.int64)
    gathered = [torch.zeros(world, dtype=torch.int64) for _ in range(world)]
    dist.all_gather(gathered, torch.from_numpy(counts))
    mat = torch.stack(gathered).numpy()
    st, woff, rtot, cap = lib.hape_peer_plan(world, rank, mat.reshape(-1).tolist())
    assert st == 0
    assert rtot == int(mat[:, rank].sum()) and cap == int(mat.sum(axis=0).max()) and rtot <= cap
    caps = [torch.zeros(1, dtype=torch.int64) for _ in range(world)]
    dist.all_gather(caps, torch.tensor([cap]))
    assert len({int(c) for c in caps}) == 1          # every rank sizes its buffer alike
    order = np.argsort(dest, kind="stable")
    # offsets travel to the destinations (one per source)
    offs_in = torch.empty(world, dtype=torch.int64)
    dist.all_to_all_single(offs_in, torch.tensor(woff, dtype=torch.int64))
    out = []
    for col in (keys, pays):
        send = torch.from_numpy(np.ascontiguousarray(col[order]).astype(np.int64))
        recv = torch.empty(rtot, dtype=torch.int64)
        dist.all_to_all_single(recv, send, output_split_sizes=mat[:, rank].tolist(),
                               input_split_sizes=mat[rank].tolist())
        buf = np.full(cap, np.iinfo(np.int64).min, np.int64)
        filled = np.zeros(cap, np.int64)
        pos = 0
        for src in range(world):
            c = int(mat[src, rank])
            o = int(offs_in[src])
            buf[o:o + c] = recv.numpy()[pos:pos + c]
            filled[o:o + c] += 1
            pos += c
        # the sources' segments tile [0, rtot) exactly: no overlap, no gap
        assert (filled[:rtot] == 1).all() and (filled[rtot:] == 0).all()
        out.append(buf[:rtot].astype(col.dtype))
    assert (partition.destination(out[0], world) == rank).all()
    return out


def _worker(rank, world, port, cfg, n, q, peer=False):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    from paper_conf_cidr_chrysogelossa19_b200 import _lib
    kw = dict(dup_domain=97) if cfg == "dup" else {}
    wl = datagen.make(cfg, n_r=n, n_s=n + 333, rank=rank, world=world, **kw)
    route = _route_peer if peer else _route
    rk, rp = route(np.asarray(wl.R.key), np.asarray(wl.R.payload), world, rank, _lib)
    sk, sp = route(np.asarray(wl.S.key), np.asarray(wl.S.payload), world, rank, _lib)
    loc = oracle.join(rk, rp, sk, sp)
    vals = torch.tensor([loc["count"], loc["sum_r"], loc["sum_s"], loc["checksum"]], dtype=torch.float64)
    parts = [torch.zeros(4, dtype=torch.float64) for _ in range(world)]
    # gather exact integers as 4 x 16-bit limbs (no float rounding)
    limbs = torch.tensor([[(v >> (16 * i)) & 0xFFFF for i in range(4)] for v in
                          (loc["count"], loc["sum_r"], loc["sum_s"], loc["checksum"])], dtype=torch.int64)
    allv = [torch.zeros_like(limbs) for _ in range(world)]
    dist.all_gather(allv, limbs)
    if rank == 0:
        tot = [0, 0, 0, 0]
        for t in allv:
            for f in range(4):
                tot[f] = (tot[f] + sum(int(t[f][i]) << (16 * i) for i in range(4))) & M64
        q.put(tot)
    dist.destroy_process_group()


@pytest.mark.parametrize("world,cfg,peer", [(2, "c1", False), (4, "c1", False), (2, "dup", False),
                                            (2, "c3", False), (2, "c1", True), (4, "c1", True),
                                            (4, "dup", True), (2, "c3", True)])
def test_sharded_join_equals_global_oracle(world, cfg, peer):
    n = 1 << 13
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, cfg, n, q, peer)) for r in range(world)]
    for p in procs:
        p.start()
    tot = q.get(timeout=240)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    kw = dict(dup_domain=97) if cfg == "dup" else {}
    g = datagen.make(cfg, n_r=n, n_s=n + 333, **kw)
    want = oracle.join(g.R.key, g.R.payload, g.S.key, g.S.payload)
    assert tot == [want["count"], want["sum_r"], want["sum_s"], want["checksum"]]
