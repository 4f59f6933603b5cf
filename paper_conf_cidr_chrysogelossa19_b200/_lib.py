"""ctypes binding of include/hape.h -- argument marshalling only.

Function names are the C names.  Every step of the join runs in libhape.so's
sm_100a kernels; there is no Python or CPU fallback: if the library cannot be
loaded, importing the binding raises.
"""
from __future__ import annotations

import ctypes
import os

_PKG = os.path.dirname(os.path.abspath(__file__))
# HAPE_LIB: an A/B variant built by build.py --out (tuning only)
LIB_PATH = os.environ.get("HAPE_LIB") or os.path.join(_PKG, "libhape.so")

HAPE_OK = 0
HAPE_ERR_INVALID_ARG = 1
HAPE_ERR_CUDA = 2
HAPE_ERR_OOM = 3
HAPE_ERR_OUTPUT_CAPACITY = 4
HAPE_ERR_NCCL = 5
HAPE_ERR_UNSUPPORTED = 6

HAPE_INT32 = 0
HAPE_INT64 = 1
HAPE_PART_HASH = 0
HAPE_PART_IDENTITY = 1
HAPE_MEM_DEVICE = 0
HAPE_MEM_HOST = 1
HAPE_FLAG_R_UNIQUE = 1
HAPE_FLAG_LINKED = 2

STAGES = ["h2d", "devpart", "exchange", "hist1", "scan1", "scatter1", "hist2", "scan2",
          "scatter2", "worklist", "build_probe", "np_build", "np_probe", "finalize", "host_part", "total"]
HAPE_NSTAGES = len(STAGES)

EXPORTED = ["hape_version", "hape_status_string", "hape_join_create", "hape_radix_join",
            "hape_join_destroy", "hape_last_error", "hape_join_plan", "hape_debug_partition",
            "hape_nccl_unique_id", "hape_nccl_comm_init", "hape_nccl_comm_destroy",
            "hape_exchange_plan", "hape_nonpartitioned_join", "hape_coprocess_join",
            "hape_host_partition", "hape_join_stream", "hape_debug_route", "hape_debug_loopback_join",
            "hape_peer_plan"]


class hape_join_config(ctypes.Structure):
    _fields_ = [("device", ctypes.c_int), ("key_type", ctypes.c_int),
                ("r_payload_type", ctypes.c_int), ("s_payload_type", ctypes.c_int),
                ("radix_passes", ctypes.c_int), ("radix_bits", ctypes.c_int * 2),
                ("part_fn", ctypes.c_int), ("max_r", ctypes.c_uint64), ("max_s", ctypes.c_uint64),
                ("world_size", ctypes.c_int), ("rank", ctypes.c_int),
                ("nccl_comm", ctypes.c_void_p), ("stream", ctypes.c_void_p), ("flags", ctypes.c_int)]


class hape_relation(ctypes.Structure):
    _fields_ = [("key", ctypes.c_void_p), ("payload", ctypes.c_void_p), ("n", ctypes.c_uint64),
                ("mem", ctypes.c_int)]


class hape_output(ctypes.Structure):
    _fields_ = [("r_payload", ctypes.c_void_p), ("s_payload", ctypes.c_void_p),
                ("capacity", ctypes.c_uint64), ("mem", ctypes.c_int)]


class hape_join_result(ctypes.Structure):
    _fields_ = [("match_count", ctypes.c_uint64), ("sum_r_payload", ctypes.c_uint64),
                ("sum_s_payload", ctypes.c_uint64), ("pair_checksum", ctypes.c_uint64),
                ("local_match_count", ctypes.c_uint64), ("local_sum_r", ctypes.c_uint64),
                ("local_sum_s", ctypes.c_uint64), ("local_pair_checksum", ctypes.c_uint64),
                ("n_written", ctypes.c_uint64), ("n_required", ctypes.c_uint64),
                ("r_local", ctypes.c_uint64), ("s_local", ctypes.c_uint64),
                ("passes", ctypes.c_uint32), ("bits", ctypes.c_uint32 * 2),
                ("n_partitions", ctypes.c_uint32), ("n_items", ctypes.c_uint32),
                ("kernel_launches", ctypes.c_uint32), ("stage_ms", ctypes.c_float * HAPE_NSTAGES),
                ("exchange_path", ctypes.c_uint32)]


class hape_coprocess_config(ctypes.Structure):
    _fields_ = [("device_budget", ctypes.c_uint64), ("fanout_bits", ctypes.c_uint32),
                ("host_threads", ctypes.c_int)]


class hape_plan(ctypes.Structure):
    _fields_ = [("passes", ctypes.c_uint32), ("bits", ctypes.c_uint32 * 2),
                ("slot_bits", ctypes.c_uint32), ("slot_shift", ctypes.c_uint32),
                ("dest_bits", ctypes.c_uint32), ("ctas_per_seg", ctypes.c_uint32 * 2),
                ("build_cap", ctypes.c_uint32), ("probe_slice", ctypes.c_uint32),
                ("join_ctas", ctypes.c_uint32)]


def _load() -> ctypes.CDLL:
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"{LIB_PATH} is missing: run __graft_entry__.build() "
                          "(python __graft_entry__.py); there is no fallback")
    lib = ctypes.CDLL(LIB_PATH)
    P = ctypes.POINTER
    vp = ctypes.c_void_p
    lib.hape_version.restype = ctypes.c_char_p
    lib.hape_version.argtypes = []
    lib.hape_status_string.restype = ctypes.c_char_p
    lib.hape_status_string.argtypes = [ctypes.c_int]
    lib.hape_join_create.restype = ctypes.c_int
    lib.hape_join_create.argtypes = [P(hape_join_config), P(vp)]
    lib.hape_radix_join.restype = ctypes.c_int
    lib.hape_radix_join.argtypes = [vp, P(hape_relation), P(hape_relation), P(hape_output),
                                    P(hape_join_result)]
    lib.hape_nonpartitioned_join.restype = ctypes.c_int
    lib.hape_nonpartitioned_join.argtypes = [vp, P(hape_relation), P(hape_relation), P(hape_output),
                                             P(hape_join_result)]
    lib.hape_coprocess_join.restype = ctypes.c_int
    lib.hape_coprocess_join.argtypes = [vp, P(hape_relation), P(hape_relation), P(hape_coprocess_config),
                                        P(hape_output), P(hape_join_result)]
    lib.hape_host_partition.restype = ctypes.c_int
    lib.hape_host_partition.argtypes = [P(hape_relation), ctypes.c_int, ctypes.c_int, ctypes.c_int,
                                        ctypes.c_uint32, ctypes.c_int, vp, vp, P(ctypes.c_uint64)]
    lib.hape_join_destroy.restype = ctypes.c_int
    lib.hape_join_destroy.argtypes = [vp]
    lib.hape_last_error.restype = ctypes.c_char_p
    lib.hape_last_error.argtypes = [vp]
    lib.hape_join_plan.restype = ctypes.c_int
    lib.hape_join_plan.argtypes = [vp, ctypes.c_uint64, ctypes.c_uint64, P(hape_plan)]
    lib.hape_debug_partition.restype = ctypes.c_int
    lib.hape_debug_partition.argtypes = [vp, P(hape_relation), ctypes.c_int, P(hape_plan), vp, vp,
                                         vp, P(hape_plan)]
    lib.hape_nccl_unique_id.restype = ctypes.c_int
    lib.hape_nccl_unique_id.argtypes = [vp]
    lib.hape_nccl_comm_init.restype = ctypes.c_int
    lib.hape_nccl_comm_init.argtypes = [vp, ctypes.c_int, ctypes.c_int, ctypes.c_int, P(vp)]
    lib.hape_nccl_comm_destroy.restype = ctypes.c_int
    lib.hape_nccl_comm_destroy.argtypes = [vp]
    lib.hape_exchange_plan.restype = ctypes.c_int
    lib.hape_exchange_plan.argtypes = [ctypes.c_int, ctypes.c_int, P(ctypes.c_uint64),
                                       P(ctypes.c_uint64), P(ctypes.c_uint64), P(ctypes.c_uint64)]
    lib.hape_peer_plan.restype = ctypes.c_int
    lib.hape_peer_plan.argtypes = [ctypes.c_int, ctypes.c_int, P(ctypes.c_uint64), P(ctypes.c_uint64),
                                   P(ctypes.c_uint64), P(ctypes.c_uint64)]
    lib.hape_join_stream.restype = ctypes.c_int
    lib.hape_join_stream.argtypes = [vp, P(vp)]
    lib.hape_debug_route.restype = ctypes.c_int
    lib.hape_debug_route.argtypes = [vp, P(hape_relation), ctypes.c_int, ctypes.c_int, vp, vp, vp]
    lib.hape_debug_loopback_join.restype = ctypes.c_int
    lib.hape_debug_loopback_join.argtypes = [vp, ctypes.c_int, ctypes.c_int, P(hape_relation), P(hape_relation),
                                             P(hape_output), P(hape_join_result), P(hape_join_result)]
    return lib


lib = _load()


# -- same names as the C ABI ------------------------------------------------
def hape_version() -> str:
    return lib.hape_version().decode()


def hape_status_string(s: int) -> str:
    return lib.hape_status_string(s).decode()


def hape_join_create(cfg: hape_join_config):
    h = ctypes.c_void_p()
    st = lib.hape_join_create(ctypes.byref(cfg), ctypes.byref(h))
    return st, h


def hape_radix_join(h, R: hape_relation, S: hape_relation, out, res: hape_join_result) -> int:
    return lib.hape_radix_join(h, ctypes.byref(R), ctypes.byref(S),
                               ctypes.byref(out) if out is not None else None, ctypes.byref(res))


def hape_nonpartitioned_join(h, R: hape_relation, S: hape_relation, out, res: hape_join_result) -> int:
    return lib.hape_nonpartitioned_join(h, ctypes.byref(R), ctypes.byref(S),
                                        ctypes.byref(out) if out is not None else None, ctypes.byref(res))


def hape_coprocess_join(h, R: hape_relation, S: hape_relation, cp, out, res: hape_join_result) -> int:
    return lib.hape_coprocess_join(h, ctypes.byref(R), ctypes.byref(S),
                                   ctypes.byref(cp) if cp is not None else None,
                                   ctypes.byref(out) if out is not None else None, ctypes.byref(res))


def hape_host_partition(rel: hape_relation, key_type: int, payload_type: int, part_fn: int,
                        fanout_bits: int, threads: int, out_keys: int, out_payloads: int, out_bounds) -> int:
    return lib.hape_host_partition(ctypes.byref(rel), key_type, payload_type, part_fn, fanout_bits, threads,
                                   out_keys, out_payloads, out_bounds)


def hape_join_destroy(h) -> int:
    return lib.hape_join_destroy(h)


def hape_last_error(h) -> str:
    r = lib.hape_last_error(h)
    return r.decode() if r else ""


def hape_join_plan(h, n_r: int, n_s: int):
    p = hape_plan()
    st = lib.hape_join_plan(h, n_r, n_s, ctypes.byref(p))
    return st, p


def hape_debug_partition(h, rel: hape_relation, is_s: int, plan_in, out_keys: int,
                         out_payloads: int, out_bounds: int):
    p = hape_plan()
    st = lib.hape_debug_partition(h, ctypes.byref(rel), is_s,
                                  ctypes.byref(plan_in) if plan_in is not None else None,
                                  out_keys, out_payloads, out_bounds, ctypes.byref(p))
    return st, p


def hape_nccl_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    st = lib.hape_nccl_unique_id(buf)
    if st != HAPE_OK:
        raise RuntimeError(hape_status_string(st))
    return buf.raw


def hape_nccl_comm_init(uid: bytes, world: int, rank: int, device: int):
    comm = ctypes.c_void_p()
    buf = ctypes.create_string_buffer(uid, 128)
    st = lib.hape_nccl_comm_init(buf, world, rank, device, ctypes.byref(comm))
    return st, comm


def hape_nccl_comm_destroy(comm) -> int:
    return lib.hape_nccl_comm_destroy(comm)


def hape_exchange_plan(world: int, rank: int, counts):
    G = world
    c = (ctypes.c_uint64 * (G * G))(*[int(x) for x in counts])
    so = (ctypes.c_uint64 * G)()
    ro = (ctypes.c_uint64 * G)()
    rt = ctypes.c_uint64()
    st = lib.hape_exchange_plan(G, rank, c, so, ro, ctypes.byref(rt))
    return st, list(so), list(ro), int(rt.value)


def hape_join_stream(h):
    s = ctypes.c_void_p()
    st = lib.hape_join_stream(h, ctypes.byref(s))
    return st, int(s.value or 0)


def hape_debug_route(h, rel: hape_relation, is_s: int, fanout: int, out_keys: int, out_payloads: int,
                     out_bounds: int) -> int:
    return lib.hape_debug_route(h, ctypes.byref(rel), is_s, fanout, out_keys, out_payloads, out_bounds)


def hape_debug_loopback_join(h, world: int, peer: int, R_shards, S_shards, out, per_dest,
                             total: hape_join_result) -> int:
    Ra = (hape_relation * world)(*R_shards)
    Sa = (hape_relation * world)(*S_shards)
    return lib.hape_debug_loopback_join(h, world, peer, Ra, Sa, ctypes.byref(out) if out is not None else None,
                                        per_dest, ctypes.byref(total))


def hape_peer_plan(world: int, rank: int, counts):
    G = world
    c = (ctypes.c_uint64 * (G * G))(*[int(x) for x in counts])
    wo = (ctypes.c_uint64 * G)()
    rt = ctypes.c_uint64()
    cap = ctypes.c_uint64()
    st = lib.hape_peer_plan(G, rank, c, wo, ctypes.byref(rt), ctypes.byref(cap))
    return st, list(wo), int(rt.value), int(cap.value)
