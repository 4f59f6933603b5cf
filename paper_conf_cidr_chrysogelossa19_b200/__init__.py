"""HAPE radix hash equi-join, B200-native (sm_100a) -- thin Python front end.

The product is libhape.so (csrc/, C ABI in include/hape.h).  This module only
marshals torch tensors into the ABI structs: it never computes any part of the
join and has no fallback path.

    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin
    j = RadixJoin(key_dtype=torch.int32)
    res = j.join(rk, rp, sk, sp)            # CUDA tensors (or pinned host tensors)
    res.match_count, res.sum_r_payload, res.sum_s_payload, res.pair_checksum
"""
from __future__ import annotations

import ctypes
import dataclasses
from typing import Optional

from . import _lib
from ._lib import (HAPE_INT32, HAPE_INT64, HAPE_MEM_DEVICE, HAPE_MEM_HOST, HAPE_OK,
                   HAPE_ERR_OUTPUT_CAPACITY, HAPE_PART_HASH, HAPE_PART_IDENTITY, STAGES,
                   hape_join_config, hape_join_create, hape_join_destroy, hape_join_plan,
                   hape_join_result, hape_last_error, hape_output, hape_radix_join,
                   hape_nonpartitioned_join, hape_coprocess_join, hape_coprocess_config,
                   hape_host_partition,
                   hape_relation, hape_status_string, hape_debug_partition, hape_version,
                   hape_join_stream, hape_debug_route, hape_debug_loopback_join)

__all__ = ["RadixJoin", "JoinResult", "HapeError", "hape_version", "hape_join_create",
           "hape_radix_join", "hape_nonpartitioned_join", "hape_coprocess_join", "hape_join_destroy",
           "hape_join_stream", "hape_debug_route", "hape_debug_loopback_join", "host_partition", "STAGES"]


class HapeError(RuntimeError):
    def __init__(self, status: int, detail: str):
        super().__init__(f"{hape_status_string(status)}: {detail}")
        self.status = status


@dataclasses.dataclass
class JoinResult:
    status: int
    match_count: int
    sum_r_payload: int
    sum_s_payload: int
    pair_checksum: int
    local_match_count: int
    local_sum_r: int
    local_sum_s: int
    local_pair_checksum: int
    n_written: int
    n_required: int
    r_local: int
    s_local: int
    passes: int
    bits: tuple
    n_partitions: int
    n_items: int
    kernel_launches: int
    stage_ms: dict
    exchange_path: int = 0

    def as_tuple(self):
        return (self.match_count, self.sum_r_payload, self.sum_s_payload, self.pair_checksum)


def _dt(torch_dtype) -> int:
    import torch
    if torch_dtype == torch.int32:
        return HAPE_INT32
    if torch_dtype == torch.int64:
        return HAPE_INT64
    raise TypeError(f"unsupported dtype {torch_dtype} (int32 / int64 only)")


def _rel(key, pay, key_type=None, pay_type=None, device=None) -> hape_relation:
    if key.dim() != 1 or pay.dim() != 1 or key.shape[0] != pay.shape[0]:
        raise ValueError("key/payload must be 1-D columns of equal length")
    if not key.is_contiguous() or not pay.is_contiguous():
        raise ValueError("columns must be contiguous")
    if key.device != pay.device:
        raise ValueError("key and payload must live on the same device")
    if key_type is not None and _dt(key.dtype) != key_type:
        raise ValueError(f"key dtype {key.dtype} does not match the handle's key type")
    if pay_type is not None and _dt(pay.dtype) != pay_type:
        raise ValueError(f"payload dtype {pay.dtype} does not match the handle's payload type")
    if key.is_cuda and device is not None and key.device.index != device:
        raise ValueError(f"columns live on {key.device}, the handle on cuda:{device}")
    mem = HAPE_MEM_DEVICE if key.is_cuda else HAPE_MEM_HOST
    return hape_relation(key.data_ptr() if key.numel() else None,
                         pay.data_ptr() if pay.numel() else None, key.shape[0], mem)


def _result(st, res) -> "JoinResult":
    return JoinResult(
        status=st, match_count=res.match_count, sum_r_payload=res.sum_r_payload,
        sum_s_payload=res.sum_s_payload, pair_checksum=res.pair_checksum,
        local_match_count=res.local_match_count, local_sum_r=res.local_sum_r,
        local_sum_s=res.local_sum_s, local_pair_checksum=res.local_pair_checksum,
        n_written=res.n_written, n_required=res.n_required, r_local=res.r_local,
        s_local=res.s_local, passes=res.passes, bits=(res.bits[0], res.bits[1]),
        n_partitions=res.n_partitions, n_items=res.n_items,
        kernel_launches=res.kernel_launches,
        stage_ms={name: float(res.stage_ms[i]) for i, name in enumerate(STAGES)},
        exchange_path=res.exchange_path)


class RadixJoin:
    """Owns one hape_join handle (one per process and device)."""

    def __init__(self, key_dtype=None, r_payload_dtype=None, s_payload_dtype=None, device: int = 0,
                 radix_passes: int = 0, radix_bits=(0, 0), identity: bool = False,
                 max_r: int = 0, max_s: int = 0, world_size: int = 1, rank: int = 0,
                 nccl_comm=None, stream=None, r_unique: bool = False, linked: bool = False):
        import torch
        key_dtype = key_dtype or torch.int32
        cfg = hape_join_config()
        cfg.device = device
        cfg.key_type = _dt(key_dtype)
        cfg.r_payload_type = _dt(r_payload_dtype or key_dtype)
        cfg.s_payload_type = _dt(s_payload_dtype or key_dtype)
        cfg.radix_passes = radix_passes
        cfg.radix_bits[0], cfg.radix_bits[1] = radix_bits
        cfg.part_fn = HAPE_PART_IDENTITY if identity else HAPE_PART_HASH
        cfg.max_r, cfg.max_s = max_r, max_s
        cfg.world_size, cfg.rank = world_size, rank
        cfg.flags = (_lib.HAPE_FLAG_R_UNIQUE if r_unique else 0) | (_lib.HAPE_FLAG_LINKED if linked else 0)
        cfg.nccl_comm = nccl_comm.value if isinstance(nccl_comm, ctypes.c_void_p) else nccl_comm
        # the library enqueues on the caller's stream (inputs must be ready on
        # it): default to torch's current stream on the device
        if stream is None:
            stream = torch.cuda.current_stream(device)
        cfg.stream = stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream)
        self.cfg = cfg
        st, h = hape_join_create(cfg)
        if st != HAPE_OK:
            raise HapeError(st, "hape_join_create failed")
        self._h = h
        # the stream the library really enqueues on (a NULL stream -- torch's
        # legacy default stream -- makes the handle create its own)
        st, self._stream_handle = hape_join_stream(h)
        if st != HAPE_OK:
            raise HapeError(st, "hape_join_stream failed")

    def close(self):
        if getattr(self, "_h", None) is not None and self._h.value:
            hape_join_destroy(self._h)
            self._h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    @property
    def handle(self):
        return self._h

    def plan(self, n_r: int, n_s: int):
        st, p = hape_join_plan(self._h, n_r, n_s)
        if st != HAPE_OK:
            raise HapeError(st, hape_last_error(self._h))
        return p

    def _order_inputs(self):
        """Order the library's stream after torch's current stream: inputs
        produced there must be complete before the join's kernels read them
        (the ABI leaves ordering to the caller, include/hape.h)."""
        import torch
        dev = self.cfg.device
        cur = torch.cuda.current_stream(dev)
        if cur.cuda_stream != self._stream_handle:
            if getattr(self, "_ext", None) is None:
                self._ext = torch.cuda.ExternalStream(self._stream_handle, device=dev)
                self._ev = torch.cuda.Event()
            self._ev.record(cur)
            self._ext.wait_event(self._ev)

    @property
    def stream(self):
        """The library's stream as a torch stream object."""
        import torch
        return torch.cuda.ExternalStream(self._stream_handle, device=self.cfg.device)

    def join(self, rk, rp, sk, sp, out_r=None, out_s=None, raise_on_capacity: bool = True) -> JoinResult:
        """hape_radix_join: the partitioned radix hash join (the product path)."""
        return self._call(hape_radix_join, rk, rp, sk, sp, out_r, out_s, raise_on_capacity)

    def join_nonpartitioned(self, rk, rp, sk, sp, out_r=None, out_s=None,
                            raise_on_capacity: bool = True) -> JoinResult:
        """hape_nonpartitioned_join: one HBM hash table over R (Fig. 6's
        non-partitioned GPU join, kept for the comparison)."""
        return self._call(hape_nonpartitioned_join, rk, rp, sk, sp, out_r, out_s, raise_on_capacity)

    def coprocess_join(self, rk, rp, sk, sp, out_r=None, out_s=None, device_budget: int = 0,
                       fanout_bits: int = 0, host_threads: int = 0,
                       raise_on_capacity: bool = True) -> JoinResult:
        """hape_coprocess_join: out-of-HBM co-processing of host-resident R and S
        (CPU tensors, pinned for full PCIe speed): CPU-side co-partitioning, one
        transfer per co-partition pair, the device radix join per pair (PAPER.md
        §5, P717-737; Fig. 7).  stage_ms['host_part'] is the host step."""
        cp = hape_coprocess_config(int(device_budget), int(fanout_bits), int(host_threads))
        fn = lambda h, R, S, out, res: hape_coprocess_join(h, R, S, cp, out, res)  # noqa: E731
        return self._call(fn, rk, rp, sk, sp, out_r, out_s, raise_on_capacity)

    def _rels(self, rk, rp, sk, sp):
        c = self.cfg
        R = _rel(rk, rp, c.key_type, c.r_payload_type, c.device)
        S = _rel(sk, sp, c.key_type, c.s_payload_type, c.device)
        return R, S

    def _out(self, out_r, out_s):
        if out_r is None and out_s is None:
            return None
        c = self.cfg
        if out_r is None or out_s is None or out_r.dim() != 1 or out_s.dim() != 1 \
                or out_r.shape[0] != out_s.shape[0]:
            raise ValueError("out_r / out_s must be given together as 1-D tensors of equal length")
        if not out_r.is_contiguous() or not out_s.is_contiguous():
            raise ValueError("out_r / out_s must be contiguous")
        if out_r.device != out_s.device:
            raise ValueError("out_r / out_s must live on the same device")
        if _dt(out_r.dtype) != c.r_payload_type or _dt(out_s.dtype) != c.s_payload_type:
            raise ValueError("out_r / out_s dtypes must match the R / S payload types")
        if out_r.is_cuda and out_r.device.index != c.device:
            raise ValueError(f"outputs live on {out_r.device}, the handle on cuda:{c.device}")
        return hape_output(out_r.data_ptr(), out_s.data_ptr(), out_r.shape[0],
                           HAPE_MEM_DEVICE if out_r.is_cuda else HAPE_MEM_HOST)

    def _call(self, fn, rk, rp, sk, sp, out_r, out_s, raise_on_capacity) -> JoinResult:
        R, S = self._rels(rk, rp, sk, sp)
        out = self._out(out_r, out_s)
        self._order_inputs()
        res = hape_join_result()
        st = fn(self._h, R, S, out, res)
        if st != HAPE_OK and not (st == HAPE_ERR_OUTPUT_CAPACITY and not raise_on_capacity):
            raise HapeError(st, hape_last_error(self._h))
        return _result(st, res)

    def loopback_join(self, r_shards, s_shards, out_r=None, out_s=None, raise_on_capacity: bool = True,
                      peer: bool = False):
        """hape_debug_loopback_join: len(r_shards) simulated ranks on this GPU
        (every device step of the G>1 path; device copies stand in for NCCL,
        or, with peer=True, the fused peer-scatter exchange into one receive
        buffer per simulated rank).
        r_shards / s_shards: lists of (key, payload) CUDA tensor pairs.
        Returns (total JoinResult, [per-destination JoinResult])."""
        G = len(r_shards)
        if len(s_shards) != G:
            raise ValueError("one R and one S shard per simulated rank")
        rels = [self._rels(rk, rp, sk, sp) for (rk, rp), (sk, sp) in zip(r_shards, s_shards)]
        out = self._out(out_r, out_s)
        self._order_inputs()
        per = (hape_join_result * G)()
        tot = hape_join_result()
        st = hape_debug_loopback_join(self._h, G, int(peer), [r for r, _ in rels], [s for _, s in rels], out, per,
                                      tot)
        if st != HAPE_OK and not (st == HAPE_ERR_OUTPUT_CAPACITY and not raise_on_capacity):
            raise HapeError(st, hape_last_error(self._h))
        return _result(st, tot), [_result(st, per[d]) for d in range(G)]

    def debug_route(self, key, pay, fanout: int, is_s: bool = False):
        """hape_debug_route: the destination partition with fan-out `fanout`;
        returns (keys, payloads, bounds[int64 of fanout+1])."""
        import torch
        c = self.cfg
        rel = _rel(key, pay, c.key_type, c.s_payload_type if is_s else c.r_payload_type, c.device)
        self._order_inputs()
        dev = torch.device("cuda", c.device)
        ok = torch.empty_like(key, device=dev)
        op = torch.empty_like(pay, device=dev)
        ob = torch.empty(fanout + 1, dtype=torch.int32, device=dev)
        st = hape_debug_route(self._h, rel, int(is_s), int(fanout), ok.data_ptr(), op.data_ptr(), ob.data_ptr())
        if st != HAPE_OK:
            raise HapeError(st, hape_last_error(self._h))
        return ok, op, ob.to(torch.int64) & 0xFFFFFFFF

    def debug_partition(self, key, pay, is_s: bool = False, plan=None):
        """Run the planned radix passes on one relation; returns
        (partitioned keys, partitioned payloads, bounds[int64], plan)."""
        import torch
        c = self.cfg
        rel = _rel(key, pay, c.key_type, c.s_payload_type if is_s else c.r_payload_type, c.device)
        self._order_inputs()
        dev = torch.device("cuda", self.cfg.device)
        ok = torch.empty_like(key, device=dev)
        op = torch.empty_like(pay, device=dev)
        p = plan or self.plan(key.shape[0], key.shape[0])
        Q = 1 << (p.bits[0] + (p.bits[1] if p.passes == 2 else 0))
        ob = torch.empty(Q + 1, dtype=torch.int32, device=dev)
        st, pout = hape_debug_partition(self._h, rel, int(is_s), p, ok.data_ptr(), op.data_ptr(),
                                        ob.data_ptr())
        if st != HAPE_OK:
            raise HapeError(st, hape_last_error(self._h))
        return ok, op, ob.to(torch.int64) & 0xFFFFFFFF, pout


def host_partition(key, pay, fanout_bits: int, identity: bool = False, threads: int = 0):
    """hape_host_partition (the co-processing join's CPU step) on CPU tensors:
    returns (keys, payloads, bounds[int64 of 2^fanout_bits + 1])."""
    import torch
    if key.is_cuda or pay.is_cuda:
        raise ValueError("host_partition takes CPU tensors")
    key, pay = key.contiguous(), pay.contiguous()
    rel = _rel(key, pay)
    ok = torch.empty_like(key)
    op = torch.empty_like(pay)
    F = 1 << int(fanout_bits)
    b = (ctypes.c_uint64 * (F + 1))()
    st = hape_host_partition(rel, _dt(key.dtype), _dt(pay.dtype),
                             HAPE_PART_IDENTITY if identity else HAPE_PART_HASH, int(fanout_bits), int(threads),
                             ok.data_ptr() if ok.numel() else None, op.data_ptr() if op.numel() else None, b)
    if st != HAPE_OK:
        raise HapeError(st, "hape_host_partition failed")
    return ok, op, torch.tensor(list(b), dtype=torch.int64)
