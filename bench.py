#!/usr/bin/env python
"""Benchmark of the B200 radix hash equi-join (BASELINE.json metric).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config c2] [--impl ours|reference]

A step is one hape_radix_join call over the whole workload: both radix passes
over R and S (hist -> scan -> scatter), the work list, the smem build+probe
with the fused count/sum/checksum aggregation and the result read-back.  At
N=1 the workload is BASELINE.json configs[1] (|R|=|S|=2^27 int32, 2-pass);
under torchrun (N>1) the same c2 workload scales weakly: every rank holds a
2^27-row shard of R and of S of a global 2^27*N-row relation, routed by the
NCCL exchange.  `--config c4` runs BASELINE configs[3] (2^31 x 2^31, strong
scaling: the global job split over the ranks).  At N=1 the line also carries
`legs`: the other BASELINE configs on the one GPU (C1, C3, C4 = 2^31 x 2^31,
C2 with the bag-semantics probe, C5 at theta 0.5/0.75/0.9/1.0), each with
its own stage roofline.

Prints ONE JSON line on rank 0.  `value` is device-resident throughput
(|R|+|S|)/s; `e2e` repeats the measurement through the same C-ABI call with
pinned HOST buffers (H2D inside the timed region); `roofline` is the dominant
kernel's algorithmic bytes / its CUDA-event time (stage events recorded on the
launching stream inside libhape) against MEASURED_PEAKS.json; `cpu_baseline`
is the CPU oracle (test infrastructure, never tuned) timed on a bounded sample
of the same recipe on this host.
"""
from __future__ import annotations

import argparse
import json
import os
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "radix-join (|R|+|S|) tuples/sec at 1/2/4/8 B200; % of HBM roofline"
UNIT = "tuples/s"
FALLBACK_HBM_GBS = 6650.0

CONFIG_TEXT = {
    "c1": "|R|=|S|=2^20 int32 key/payload, unique PK-FK uniform keys (BASELINE configs[0])",
    "c2": "|R|=|S|=2^27 int32 key/payload, unique uniform keys, 2-pass radix (BASELINE configs[1])",
    "c3": "|R|=2^27, |S|=2^30 int64 key/payload FK join, materialised pairs (BASELINE configs[2])",
    "c4": "|R|=|S|=2^31 int32, hash-shuffled via NCCL all-to-all and co-partitioned join (BASELINE configs[3])",
    "c5": "|R|=2^28, |S|=2^30 int32 with Zipf-skewed probe keys (BASELINE configs[4])",
}


def load_peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs, torch copy)"
    except Exception:
        return FALLBACK_HBM_GBS, "fallback (B200_PROFILING.md)"


# --------------------------------------------------------------------------
class ClockSampler:
    """nvidia-smi clocks + throttle reasons sampled during the timed region."""

    FIELDS = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,"
              "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
              "clocks_event_reasons.sw_power_cap")

    def __init__(self, index: int):
        self.index = index
        self.proc = None
        self.lines = []

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.FIELDS}",
                 "--format=csv,noheader,nounits", "-lms", "100"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def stop(self):
        if self.proc is None:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        time.sleep(0.25)
        self.proc.terminate()
        try:
            self.proc.wait(timeout=2)
        except Exception:
            self.proc.kill()
        sm, mx, reasons = [], [], set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for ln in self.lines:
            parts = [x.strip() for x in ln.split(",")]
            if len(parts) < 6:
                continue
            try:
                sm.append(float(parts[0]))
                mx.append(float(parts[1]))
            except ValueError:
                continue
            for nm, v in zip(names, parts[2:6]):
                if v.lower().startswith("active"):
                    reasons.add(nm)
        sm.sort()
        return {"sm_mhz": sm[len(sm) // 2] if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": sorted(reasons), "samples": len(sm)}


# --------------------------------------------------------------------------
def cpu_oracle_sample(log2n: int):
    """Time the CPU oracle (as it stands) on the c2 recipe at |R|=|S|=2^log2n:
    on all host cores (key-sharded, one single-thread sort-
    merge per shard and thread) and on one core."""
    import datagen
    import oracle
    wl = datagen.make("c2", n_r=1 << log2n, n_s=1 << log2n)
    oracle.build()
    n = 2 << log2n
    t0 = time.perf_counter()
    res = oracle.join_sharded(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    dt_t = time.perf_counter() - t0
    assert res["count"] == 1 << log2n
    t0 = time.perf_counter()
    res1 = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
    dt = time.perf_counter() - t0
    assert res1["count"] == 1 << log2n
    return dict(value=n / dt_t, unit=UNIT, cores=res["threads"], kind="oracle",
                sample=f"c2 recipe at |R|=|S|=2^{log2n} int32: key-sharded over {res['threads']} threads, "
                       f"one single-thread sort-merge per shard (incl. the host sharding), {dt_t:.2f} s",
                seconds=dt_t,
                single_core={"value": n / dt, "cores": oracle.threads_used(), "seconds": round(dt, 3),
                             "sample": "the same sample, one thread"})


def run_reference(args):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return 0
    if args.config == "auto":
        args.config = "c2"
    import numpy as np
    import datagen
    import oracle
    log2n = args.ref_log2n
    wl = datagen.make(args.config if args.config in ("c1", "c2", "c4") else "c2", n_r=1 << log2n, n_s=1 << log2n)
    oracle.build()
    times = []
    for i in range(args.warmup + args.steps):
        t0 = time.perf_counter()
        res = oracle.join(wl.R.key, wl.R.payload, wl.S.key, wl.S.payload)
        dt = time.perf_counter() - t0
        if i >= args.warmup:
            times.append(dt)
    assert res["count"] == 1 << log2n
    ms = 1000 * sum(times) / len(times)
    n = 2 << log2n
    v = n / (ms / 1000)
    line = {"metric": METRIC, "value": v, "unit": UNIT, "impl": "reference", "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True,
            "scaling": "strong" if args.config == "c4" else "weak", "vs_baseline": None, "dtype": "int32",
            "data": "synthetic",
            "config": {"workload": f"{args.config}: CPU oracle on a bounded sample |R|=|S|=2^{log2n} of the same recipe"},
            "cpu_baseline": {"value": v, "unit": UNIT, "cores": oracle.threads_used(), "kind": "oracle",
                             "sample": f"c2 recipe at |R|=|S|=2^{log2n} int32, single-thread sort-merge"},
            "e2e": {"value": v, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)
    return 0


# --------------------------------------------------------------------------
def gen_shard(cfg, n_r, n_s, rank, world, theta=1.0, chunk=1 << 27):
    """This rank's row shard of config `cfg`, generated on the device in
    row chunks of <= `chunk` tuples (the torch temporaries of one chunk stay
    a few GiB even for the 2^31-row C4 relations).  Sub-shards compose
    exactly: rows [N*i//W, N*(i+1)//W) = the union of the k sub-chunks of
    rank*k+j over world W*k."""
    import torch
    import datagen
    lo_r, hi_r = (n_r * rank) // world, (n_r * (rank + 1)) // world
    lo_s, hi_s = (n_s * rank) // world, (n_s * (rank + 1)) // world
    k = max(1, -(-max(hi_r - lo_r, hi_s - lo_s) // chunk))
    kw = dict(theta=theta) if cfg == "c5" else {}
    first = datagen.make(cfg, n_r=n_r, n_s=n_s, rank=rank * k, world=world * k, backend="torch", device="cuda", **kw)
    if k == 1:
        return first, [x.contiguous() for x in (first.R.key, first.R.payload, first.S.key, first.S.payload)]
    cols = [torch.empty(hi_r - lo_r, dtype=first.R.key.dtype, device="cuda"),
            torch.empty(hi_r - lo_r, dtype=first.R.payload.dtype, device="cuda"),
            torch.empty(hi_s - lo_s, dtype=first.S.key.dtype, device="cuda"),
            torch.empty(hi_s - lo_s, dtype=first.S.payload.dtype, device="cuda")]
    pr = ps = 0
    for j in range(k):
        wl = first if j == 0 else datagen.make(cfg, n_r=n_r, n_s=n_s, rank=rank * k + j, world=world * k,
                                               backend="torch", device="cuda", **kw)
        a, b = wl.R.n, wl.S.n
        cols[0][pr:pr + a] = wl.R.key
        cols[1][pr:pr + a] = wl.R.payload
        cols[2][ps:ps + b] = wl.S.key
        cols[3][ps:ps + b] = wl.S.payload
        pr, ps = pr + a, ps + b
        del wl
    assert pr == hi_r - lo_r and ps == hi_s - lo_s
    return first, cols


def alg_bytes(res, kw, prw, psw, materialize, joint):
    """Algorithmic bytes per stage of one call."""
    nr, ns = res.r_local, res.s_local
    tr, ts = kw + prw, kw + psw
    alg = {"hist1": kw * (nr + ns), "scatter1": 2 * (tr * nr + ts * ns),
           "hist2": kw * (nr + ns), "scatter2": 2 * (tr * nr + ts * ns),
           "build_probe": tr * nr + ts * ns + ((prw + psw) * res.n_written if materialize else 0)}
    if joint:
        alg.pop("hist2")
    if res.passes < 2:
        alg.pop("hist2", None)
        alg.pop("scatter2")
    return alg


KERNEL_NAME = {"hist1": "k_hist pass 1 (R+S)", "scatter1": "k_scatter pass 1 (R+S)",
               "hist2": "k_hist pass 2 (R+S)", "scatter2": "k_scatter pass 2 (R+S)",
               "build_probe": "k_build_probe", "devpart": "device partition (hist+scan+scatter)"}


def is_joint(res, linked=False):
    return (not linked and res.passes == 2 and 6 <= res.bits[0] + res.bits[1] <= 16
            and os.environ.get("HAPE_JOINT", "1") != "0")


def roofline_of(res, stage_avg, ms, kw, prw, psw, materialize, peak, extra=None, linked=False):
    joint = is_joint(res, linked)
    alg = alg_bytes(res, kw, prw, psw, materialize, joint)
    if linked:
        # pass 1 without a histogram: stage hist1 is the buffer-directory reset
        alg.pop("hist1", None)
    alg.update(extra or {})
    per_stage = {}
    for k in alg:
        if stage_avg.get(k, 0) > 0:
            gbs = alg[k] / (stage_avg[k] / 1000.0) / 1e9
            per_stage[k] = {"ms": round(stage_avg[k], 4), "alg_bytes": alg[k], "GB/s": round(gbs, 1),
                            "frac": round(gbs / peak, 3)}
    dom = max(per_stage, key=lambda k: per_stage[k]["ms"])
    names = dict(KERNEL_NAME)
    if joint:
        names["hist1"] = "k_hist_joint (pass-1 and pass-2 buckets, R+S)"
        names["scatter1"] = "k_scatter pass 1, claiming (R+S)"
        names["scatter2"] = "k_scatter pass 2, claiming (R+S)"
    alg_total = sum(alg.values())
    return {"bound": "hbm", "achieved": per_stage[dom]["GB/s"], "peak": peak, "unit": "GB/s",
            "frac": round(per_stage[dom]["GB/s"] / peak, 4), "kernel": names[dom], "dominant_stage": dom,
            "step": {"alg_bytes": alg_total, "GB/s": round(alg_total / (ms / 1000) / 1e9, 1),
                     "frac": round(alg_total / (ms / 1000) / 1e9 / peak, 4)},
            "stages": per_stage}


def time_calls(fn, steps, stream):
    """CUDA events on the library's stream around `steps` calls; returns
    (ms per call, summed stage_ms, launches, last result)."""
    import torch
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    stage_sum, launches, res = {}, 0, None
    e0.record(stream)
    for _ in range(steps):
        res = fn()
        launches += res.kernel_launches
        for k, v in res.stage_ms.items():
            stage_sum[k] = stage_sum.get(k, 0.0) + v
    e1.record(stream)
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / steps, {k: v / steps for k, v in stage_sum.items()}, launches, res


def run_leg(name, cfg, args, peak, n_r=None, n_s=None, theta=1.0, r_unique=True, materialize=None, steps=None,
            linked=False):
    """One extra single-GPU workload (a bench 'leg'): generate, warm up, time."""
    import torch
    import datagen
    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin
    base = datagen.SHAPES[cfg]
    n_r = n_r or base[0]
    n_s = n_s or base[1]
    t0 = time.perf_counter()
    wl, (rk, rp, sk, sp) = gen_shard(cfg, n_r, n_s, 0, 1, theta=theta)
    gen_s = time.perf_counter() - t0
    mat = (cfg == "c3") if materialize is None else materialize
    out_r = out_s = None
    if mat:
        out_r = torch.empty(n_s, dtype=rp.dtype, device="cuda")
        out_s = torch.empty(n_s, dtype=sp.dtype, device="cuda")
    j = RadixJoin(key_dtype=rk.dtype, r_payload_dtype=rp.dtype, s_payload_dtype=sp.dtype,
                  max_r=n_r, max_s=n_s, r_unique=r_unique, linked=linked, stream=torch.cuda.current_stream())
    for _ in range(args.warmup):
        res = j.join(rk, rp, sk, sp, out_r, out_s)
    torch.cuda.synchronize()
    k = steps or args.leg_steps
    ms, st, launches, res = time_calls(lambda: j.join(rk, rp, sk, sp, out_r, out_s), k, j.stream)
    kw, prw, psw = rk.element_size(), rp.element_size(), sp.element_size()
    roof = roofline_of(res, st, ms, kw, prw, psw, mat, peak, linked=linked)
    leg = {"workload": f"{cfg}: {CONFIG_TEXT.get(cfg, cfg)}" + (f"; theta={theta}" if cfg == "c5" else "")
           + ("" if r_unique else "; bag-semantics probe (R not declared unique)")
           + ("; pass 1 = single-scan linked-buffer partitioning (P593-597)" if linked else ""),
           "n_r": n_r, "n_s": n_s, "steps": k, "ms_per_step": round(ms, 4), "value": (n_r + n_s) / (ms / 1000.0),
           "unit": UNIT, "passes": res.passes, "bits": list(res.bits), "n_items": res.n_items,
           "match_count": res.match_count, "r_unique_declared": r_unique, "materialize": mat,
           "gpu_launches": launches, "gen_s": round(gen_s, 2), "roofline": roof}
    if cfg in ("c1", "c2", "c4") and n_s == n_r:
        leg["count_ok"] = res.match_count == n_s   # PK-FK same key set: |J| = |S| (P793-794)
    if cfg in ("c3", "c5"):
        leg["count_ok"] = res.match_count == n_s   # FK: every S key is in R
    j.close()
    del rk, rp, sk, sp, out_r, out_s, wl
    torch.cuda.empty_cache()
    return leg


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--config", default="auto", choices=["auto", "c1", "c2", "c3", "c4", "c5"],
                    help="auto: c2 (BASELINE configs[1]) at every N: one GPU runs |R|=|S|=2^27, N ranks "
                         "each hold a 2^27-row shard of R and of S of a global 2^27*N relation (weak scaling)")
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--ref-log2n", type=int, default=22)
    ap.add_argument("--cpu-log2n", type=int, default=24)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--verify", action="store_true", help="check the result against generator provenance")
    ap.add_argument("--bits", default="0,0", help="radix bits per pass (0 = auto; tuning only)")
    ap.add_argument("--passes", type=int, default=0, help="radix passes (0 = auto; tuning only)")
    ap.add_argument("--no-mat", action="store_true", help="c3 without materialised pairs (diagnostics)")
    ap.add_argument("--bag", action="store_true",
                    help="do not declare R's keys unique (HAPE_FLAG_R_UNIQUE): full bag-semantics probe")
    ap.add_argument("--theta", type=float, default=1.0, help="c5 Zipf skew")
    ap.add_argument("--legs", default="default",
                    help="extra single-GPU workloads at N=1, comma list of c1,c3,c4,c4rG (C4's per-rank "
                         "share at G ranks),c2bag,c2linked,c4linked,c5 (or c5:THETA); 'default' = all; 'none'")
    ap.add_argument("--leg-steps", type=int, default=5)
    ap.add_argument("--partitioner", default="hist", choices=["hist", "linked"],
                    help="pass 1: histogram -> prefix sum -> scatter (default), or the paper's single-scan "
                         "linked-buffer partitioning (HAPE_FLAG_LINKED; A/B, SURVEY NEXT-2)")
    ap.add_argument("--no-ablation", action="store_true",
                    help="skip the non-partitioned GPU join comparison (PAPER.md Fig. 6)")
    ap.add_argument("--no-coprocess", action="store_true",
                    help="skip the out-of-HBM co-processing measurement (hape_coprocess_join, PAPER.md Fig. 7)")
    ap.add_argument("--cp-fanout", type=int, default=3,
                    help="co-processing: host fan-out bits (F = 2^bits co-partition pairs, each one transfer)")
    ap.add_argument("--exchange", action="store_true",
                    help="at N=1, run the device-partition + NCCL exchange path through a 1-rank communicator")
    args = ap.parse_args()
    if args.impl == "reference":
        return run_reference(args)

    import torch
    import torch.distributed as dist
    import datagen
    from paper_conf_cidr_chrysogelossa19_b200 import RadixJoin, _lib

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    # one non-default stream for everything: the generator's kernels, the
    # library's kernels and the timing events are ordered on it
    stream = torch.cuda.Stream()
    torch.cuda.set_stream(stream)
    if world > 1:
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    args.warmup = max(args.warmup, 3)
    peak, peak_src = load_peaks()

    cfg = args.config
    if cfg == "auto":
        cfg = "c2"
    base = datagen.SHAPES[cfg]
    # c4 is a fixed global job (2^31 per relation) split over the ranks
    # (strong scaling); the other configs give every rank a full-size shard
    # of a global relation N times larger (weak scaling)
    strong = cfg == "c4"
    n_r, n_s = (base[0], base[1]) if strong else (base[0] * world, base[1] * world)
    wl, (rk, rp, sk, sp) = gen_shard(cfg, n_r, n_s, rank, world, theta=args.theta)
    kdt, pdt = rk.dtype, rp.dtype
    nr_loc, ns_loc = rk.shape[0], sk.shape[0]
    materialize = cfg == "c3" and not args.no_mat

    comm = None
    if world > 1 or args.exchange:
        uid = [_lib.hape_nccl_unique_id() if rank == 0 else None]
        if world > 1:
            dist.broadcast_object_list(uid, src=0)
        st, comm = _lib.hape_nccl_comm_init(uid[0], world, rank, local)
        assert st == 0, f"nccl comm init failed: {st}"
    j = RadixJoin(key_dtype=kdt, r_payload_dtype=pdt, s_payload_dtype=pdt, device=local,
                  max_r=nr_loc, max_s=ns_loc, world_size=world, rank=rank,
                  radix_passes=args.passes, radix_bits=tuple(int(x) for x in args.bits.split(",")),
                  r_unique=not args.bag, nccl_comm=comm, stream=stream, linked=args.partitioner == "linked")
    assert j.stream.cuda_stream == stream.cuda_stream
    out_r = out_s = None
    if materialize:
        cap = int(ns_loc * 1.1) if world > 1 else ns_loc
        out_r = torch.empty(cap, dtype=pdt, device="cuda")
        out_s = torch.empty(cap, dtype=pdt, device="cuda")

    def barrier():
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()

    def max_over_ranks(x: float) -> float:
        if world == 1:
            return x
        t = torch.tensor([x], dtype=torch.float64, device="cuda")
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return float(t.item())

    # ---- device-resident timed region
    for _ in range(args.warmup):
        res = j.join(rk, rp, sk, sp, out_r, out_s)
    verify = None
    if args.verify and world == 1:
        from oracle import provenance
        want = provenance.expected_pkfk(wl.R.payload[wl.idx].cpu().numpy(), wl.S.payload.cpu().numpy()) \
            if wl.idx is not None and n_r == wl.R.n else None
        if want is not None:
            verify = (res.match_count, res.sum_r_payload, res.sum_s_payload, res.pair_checksum) == \
                (want["count"], want["sum_r"], want["sum_s"], want["checksum"])
    clocks = ClockSampler(local)
    barrier()
    clocks.start()
    time.sleep(0.3)
    barrier()
    ms_loc, stage_avg, launches, res = time_calls(lambda: j.join(rk, rp, sk, sp, out_r, out_s), args.steps, stream)
    barrier()
    clk = clocks.stop()
    ms = max_over_ranks(ms_loc)
    total_tuples = n_r + n_s
    value = total_tuples / (ms / 1000.0)

    # ---- roofline of the dominant kernel stage (algorithmic bytes)
    kw, pw = rk.element_size(), rp.element_size()
    t = kw + pw
    extra = {}
    fused = res.exchange_path == 2
    if world > 1 or args.exchange:
        # NCCL form: destination hist + scatter into a send buffer; fused form:
        # the destination totals only (the scatter is the exchange stage)
        extra["devpart"] = (kw if fused else kw + 2 * t) * (nr_loc + ns_loc)
    roofline = roofline_of(res, stage_avg, ms, kw, pw, pw, materialize, peak, extra,
                           linked=args.partitioner == "linked")
    roofline["peak_source"] = peak_src
    traffic = None
    try:
        tj = json.load(open(os.path.join(ROOT, "profiles", "ncu_traffic.json")))
        traffic = tj.get(cfg, {}).get(roofline["dominant_stage"])
    except Exception:
        pass
    roofline["traffic"] = traffic
    if stage_avg.get("exchange", 0) > 0:
        xb = t * (nr_loc + ns_loc)  # every local tuple leaves through the exchange (incl. the self segment)
        xs = stage_avg["exchange"] / 1000.0
        remote = xb * (world - 1) // max(world, 1)
        roofline["stages"]["exchange"] = {
            "ms": round(stage_avg["exchange"], 4), "bytes_sent": xb, "GB/s": round(xb / xs / 1e9, 1),
            "remote_bytes": remote, "remote_GB/s": round(remote / xs / 1e9, 1),
            "nvlink_frac": round(remote / xs / 1e9 / 900.0, 3) if world > 1 else None,
            "form": "fused peer scatter (destination partition writes into the peers' receive buffers)"
            if fused else "NCCL send/recv of a device-partitioned send buffer",
            "bound": "nvlink 900 GB/s/dir per GPU (remote part); HBM 2t B/tuple (read + write)"}
        roofline["exchange_path"] = res.exchange_path
        if world > 1:
            # the NVLink reference the exchange stage is read against (SURVEY
            # §8.d.3): one NCCL all-to-all of the same bytes per rank, CUDA
            # events on this stream, max over ranks
            buf = out = None
            try:
                # the same size on every rank (ragged shards differ by a row)
                per = t * (n_r + n_s) // world
                buf = torch.empty(per // 4 // world * world, dtype=torch.int32, device="cuda")
                out = torch.empty_like(buf)
            except Exception:
                buf = out = None
            # every rank runs the collective, or none does
            okf = torch.tensor([1 if buf is not None else 0], dtype=torch.int32, device="cuda")
            dist.all_reduce(okf, op=dist.ReduceOp.MIN)
            try:
                if int(okf.item()) != 1:
                    raise RuntimeError("all-to-all reference buffers not allocated on every rank")
                for _ in range(2):
                    dist.all_to_all_single(out, buf)
                barrier()
                a0, a1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a0.record(stream)
                for _ in range(3):
                    dist.all_to_all_single(out, buf)
                a1.record(stream)
                barrier()
                a_ms = max_over_ranks(a0.elapsed_time(a1) / 3)
                nb = buf.numel() * 4
                roofline["stages"]["exchange"]["nccl_all_to_all_reference"] = {
                    "bytes_per_rank": nb, "ms": round(a_ms, 4),
                    "algbw_GB/s": round(nb / (a_ms / 1000.0) / 1e9, 1),
                    "busbw_GB/s": round(nb * (world - 1) / world / (a_ms / 1000.0) / 1e9, 1)}
                del buf, out
            except Exception as ex:  # never lose the line to the reference measurement
                roofline["stages"]["exchange"]["nccl_all_to_all_reference"] = {"error": repr(ex)[:200]}

    # ---- end to end through the same C ABI call with pinned host buffers
    e2e = None
    coproc = None
    if not args.no_e2e:
        hk = [x.cpu().pin_memory() for x in (rk, rp, sk, sp)]
        ho = None
        if materialize:
            ho = [torch.empty(out_r.shape[0], dtype=pdt).pin_memory(), torch.empty(out_s.shape[0], dtype=pdt).pin_memory()]
        for _ in range(2):
            j.join(*hk, *(ho or (None, None)))
        barrier()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        n_e2e = max(1, min(args.steps, 5))
        d2h = 0
        for _ in range(n_e2e):
            r2 = j.join(*hk, *(ho or (None, None)))
            d2h += 48 + (r2.n_written * 2 * pw if materialize else 0)
        e1.record(stream)
        barrier()
        e_ms = max_over_ranks(e0.elapsed_time(e1) / n_e2e)
        h2d = sum(x.numel() * x.element_size() for x in hk)
        # host-link roofline of the e2e step: a plain pinned H2D copy of the
        # same byte count, timed here with CUDA events (no join work)
        pcie = None
        try:
            src = hk[0] if hk[0].numel() * hk[0].element_size() >= (256 << 20) else None
            if src is not None:
                dst = torch.empty(src.shape, dtype=src.dtype, device="cuda")
                for _ in range(2):
                    dst.copy_(src, non_blocking=True)
                torch.cuda.synchronize()
                e0.record(stream)
                for _ in range(3):
                    dst.copy_(src, non_blocking=True)
                e1.record(stream)
                torch.cuda.synchronize()
                bw = 3 * src.numel() * src.element_size() / (e0.elapsed_time(e1) / 1000.0)
                e0.record(stream)
                for _ in range(3):
                    src.copy_(dst, non_blocking=True)
                e1.record(stream)
                torch.cuda.synchronize()
                bw_d = 3 * src.numel() * src.element_size() / (e0.elapsed_time(e1) / 1000.0)
                del dst
                d2h_b = d2h // n_e2e
                # the call moves its inputs in and its result (and pairs) out in sequence
                bound = (h2d / bw + d2h_b / bw_d) * 1000.0
                pcie = {"h2d_GB/s_measured": round(bw / 1e9, 1), "d2h_GB/s_measured": round(bw_d / 1e9, 1),
                        "bound_ms": round(bound, 3), "frac": round(bound / e_ms, 3)}
        except Exception as ex:
            pcie = {"error": repr(ex)}
        e2e = {"value": total_tuples / (e_ms / 1000.0), "unit": UNIT, "ms_per_step": e_ms,
               "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": d2h // n_e2e,
               "h2d_stage_ms": r2.stage_ms.get("h2d"), "pcie_roofline": pcie}
        # ---- PAPER.md §5 / Fig. 7 co-processing on the same host-resident
        # inputs: CPU-side co-partitioning into F pairs, one transfer per pair
        # overlapping the previous pair's device join (hape_coprocess_join,
        # SURVEY §8.f NEXT-3).  Wall-clock timed: the call includes host work.
        if world == 1 and not args.exchange and not args.no_coprocess:
            for _ in range(2):
                rc = j.coprocess_join(*hk, *(ho or (None, None)), fanout_bits=args.cp_fanout)
            n_cp = 3
            t0 = time.perf_counter()
            agg = {}
            for _ in range(n_cp):
                rc = j.coprocess_join(*hk, *(ho or (None, None)), fanout_bits=args.cp_fanout)
                for k, v in rc.stage_ms.items():
                    agg[k] = agg.get(k, 0.0) + v / n_cp
            cp_ms = (time.perf_counter() - t0) * 1000.0 / n_cp
            # PCIe H2D bandwidth as this call measured it: its bytes over the
            # summed copy-stream transfer time of the co-partition pairs
            pcie_gbs = h2d / (agg["h2d"] / 1000.0) / 1e9 if agg.get("h2d") else None
            dev = sum(v for k, v in agg.items() if k not in ("h2d", "host_part", "total"))
            coproc = {
                "method": "hape_coprocess_join: CPU co-partitioning (host threads, pinned) + one H2D per pair + device radix join per pair",
                "fanout": rc.n_partitions, "host_threads": os.cpu_count(),
                "ms_per_step": round(cp_ms, 3), "value": total_tuples / (cp_ms / 1000.0), "unit": UNIT,
                "stages_ms": {"host_partition": round(agg.get("host_part", 0), 3),
                              "h2d (copy stream)": round(agg.get("h2d", 0), 3),
                              "device joins": round(dev, 3)},
                # host-link roofline: every input byte crosses PCIe once (the
                # point of the plan, P723-724); frac = that transfer time / step
                "pcie_roofline": {"bytes": h2d, "h2d_GB/s_measured": round(pcie_gbs, 1) if pcie_gbs else None,
                                  "frac": round((h2d / (pcie_gbs * 1e9) * 1000.0) / cp_ms, 3) if pcie_gbs else None},
                # the plan's serial bound: a two-phase host partition completes
                # every co-partition at the same moment, so no transfer can
                # start before the host step ends (out-of-HBM: the device
                # cannot stage pairs it cannot join yet); then every byte
                # crosses PCIe once and the last pair's join follows its copy
                "serial_bound": {
                    "host_partition_ms": round(agg.get("host_part", 0), 3),
                    "pcie_ms": round(h2d / (pcie_gbs * 1e9) * 1000.0, 3) if pcie_gbs else None,
                    "last_pair_join_ms": round(dev / max(1, rc.n_partitions), 3),
                    "frac": round((agg.get("host_part", 0) + h2d / (pcie_gbs * 1e9) * 1000.0
                                   + dev / max(1, rc.n_partitions)) / cp_ms, 3) if pcie_gbs else None,
                    "host_partition_GB/s": round(2 * h2d / (agg["host_part"] / 1000.0) / 1e9, 1)
                    if agg.get("host_part") else None},
                "same_result_as_radix": rc.as_tuple() == res.as_tuple()}
        del hk, ho

    # ---- PAPER.md Fig. 6's comparison on this hardware: the non-partitioned
    # GPU hash join (one HBM table over R; hape_nonpartitioned_join) on the
    # same resident inputs, same result
    nonpart = None
    if world == 1 and not args.exchange and not args.no_ablation:
        for _ in range(2):
            rn = j.join_nonpartitioned(rk, rp, sk, sp, out_r, out_s)
        barrier()
        np_ms, _, _, rn = time_calls(lambda: j.join_nonpartitioned(rk, rp, sk, sp, out_r, out_s),
                                     max(1, min(args.steps, 5)), stream)
        nonpart = {"method": "non-partitioned GPU hash join (hape_nonpartitioned_join, PAPER.md Fig. 6 baseline)",
                   "ms_per_step": round(np_ms, 4), "value": total_tuples / (np_ms / 1000.0), "unit": UNIT,
                   "radix_speedup": round(np_ms / ms, 3),
                   "stages_ms": {"build (clear + insert)": round(rn.stage_ms["np_build"], 4),
                                 "probe": round(rn.stage_ms["np_probe"], 4)},
                   "same_result_as_radix": rn.as_tuple() == res.as_tuple()}

    j.close()
    del rk, rp, sk, sp, out_r, out_s
    torch.cuda.empty_cache()

    # ---- the other BASELINE configs on this one GPU (extra keys of the line)
    legs = {}
    if world == 1 and args.legs != "none":
        spec = args.legs if args.legs != "default" else \
            "c1,c3,c4,c4r2,c4r4,c4r8,c2bag,c2linked,c4linked,c5:0.5,c5:0.75,c5:0.9,c5:1.0"
        for item in [x for x in spec.split(",") if x]:
            try:
                if item == "c2bag":
                    legs[item] = run_leg(item, "c2", args, peak, r_unique=False)
                elif item in ("c2linked", "c4linked"):
                    legs[item] = run_leg(item, item[:2], args, peak, linked=True)
                elif item.startswith("c4r"):
                    # the local join one rank runs after the exchange at G = 2/4/8
                    # (2^31 / G tuples of R and of S, the C4 recipe)
                    g = int(item[3:])
                    legs[item] = run_leg(item, "c4", args, peak, n_r=(1 << 31) // g, n_s=(1 << 31) // g)
                elif item.startswith("c5"):
                    th = float(item.split(":")[1]) if ":" in item else 1.0
                    legs[f"c5_theta{th}"] = run_leg(item, "c5", args, peak, theta=th)
                else:
                    legs[item] = run_leg(item, item, args, peak, steps=args.leg_steps if item != "c1" else 50)
            except Exception as ex:  # never lose the main line to a leg
                legs[item] = {"error": repr(ex)[:400]}
                torch.cuda.empty_cache()
        if "c5_theta1.0" in legs and "c5_theta0.5" in legs and "ms_per_step" in legs["c5_theta1.0"] \
                and "ms_per_step" in legs.get("c5_theta0.5", {}):
            legs["c5_skew_ratio_theta1_vs_0.5"] = round(legs["c5_theta1.0"]["ms_per_step"]
                                                        / legs["c5_theta0.5"]["ms_per_step"], 3)

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        try:
            cpu = cpu_oracle_sample(args.cpu_log2n)
        except Exception as ex:  # never lose the GPU line to the CPU leg
            cpu = {"error": repr(ex)}

    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True,
            "scaling": "strong" if strong else "weak",
            "vs_baseline": None, "dtype": "int32" if kdt == torch.int32 else "int64",
            "data": "synthetic (datagen counter-based recipe, generated on device)",
            "config": {"workload": f"{cfg}: {CONFIG_TEXT[cfg]}"
                       + ((f"; split over {world} ranks" if strong else f"; {world} ranks x shard") if world > 1 else "")
                       + ("; through the 1-rank NCCL exchange path" if (args.exchange and world == 1) else ""),
                       "n_r": n_r, "n_s": n_s, "per_rank_r": nr_loc, "per_rank_s": ns_loc,
                       "passes": res.passes, "bits": list(res.bits), "n_items": res.n_items,
                       "r_unique_declared": not args.bag,
                       "partitioner": args.partitioner,
                       "materialize": materialize,
                       "l2": "inputs and workspace (>=2 GiB per step) exceed the 126 MB L2; no flush needed",
                       "parallelism": f"hash-sharded x{world}" if world > 1 else "1 GPU"},
            "gpu_launches": launches,
            "clocks": clk,
            "roofline": roofline,
            "e2e": e2e,
            "cpu_baseline": cpu,
        }
        if nonpart is not None:
            line["nonpartitioned_gpu"] = nonpart
        if coproc is not None:
            line["coprocess"] = coproc
        if legs:
            line["legs"] = legs
        if verify is not None:
            line["verified_vs_provenance"] = verify
        print(json.dumps(line), flush=True)
    if comm is not None:
        _lib.hape_nccl_comm_destroy(comm)
    if world > 1:
        dist.destroy_process_group()
    return 0


if __name__ == "__main__":
    sys.exit(main())
