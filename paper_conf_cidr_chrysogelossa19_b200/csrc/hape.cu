// hape.cu -- C ABI (include/hape.h) and host orchestration of the radix join.
//
// Stage sequence of one hape_radix_join call (e):
//   [H2D staging]                         host-resident inputs only
//   [device partition + exchange]         G>1: route by top log2(G) bits of h
//                                         (HetExchange hash router + mem-move,
//                                         PAPER.md P643-656, P717-737)
//   pass 1: hist -> scan -> scatter       (a6-a8; P572-598, Fig. 4)
//   pass 2: the same inside each pass-1 partition  (a9; P140-145, P589-593)
//   work list -> build+probe+aggregate    (a10-a12; P535-541, Fig. 3, P789-793)
//   result D2H (+ NCCL allreduce)         (a13)
// Every stage is one or two kernel launches on the handle's stream; the only
// host synchronisation points are the count exchange (G>1) and the result.
#include <cuda_runtime.h>
#include <nccl.h>

#include <algorithm>
#include <cstdarg>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <string>
#include <type_traits>
#include <vector>

#include "hape.h"
#include "kernels.cuh"
#include "join_oa.cuh"
#include "nonpart.cuh"

using namespace hape;

namespace {

struct DevBuf {
  void* p = nullptr;
  size_t bytes = 0;
};

constexpr uint32_t kTargetPerPartition = 2048;  // R tuples per co-partition (Fig. 5 range, P753-858)
constexpr uint32_t kMaxBitsPerPass = 12;
constexpr uint32_t kMaxSinglePassBits = 10;
constexpr uint32_t kChunk = 32768;              // tuples per partitioning CTA (upper bound)
// a partitioning CTA gets at least one full scatter tile (8-byte tuples):
// smaller chunks pay a partial tile and P total / claim atomics each
// (HAPE_MIN_CHUNK: A/B)
constexpr uint32_t kMinChunk = 6656;

inline uint32_t ceil_log2_u64(uint64_t x) {
  uint32_t b = 0;
  while ((1ull << b) < x) b++;
  return b;
}

}  // namespace

struct hape_join {
  hape_join_config cfg{};
  int dev = 0;
  int num_sms = 148;
  cudaStream_t stream = nullptr;
  bool own_stream = false;
  cudaStream_t copy_stream = nullptr;   // host-input S transfer (overlaps R's passes)
  cudaEvent_t ev_copy = nullptr;
  ncclComm_t comm = nullptr;
  std::string err;
  cudaEvent_t ev[HAPE_NSTAGES + 1] = {};
  bool ev_used[HAPE_NSTAGES] = {};
  uint32_t launches = 0;
  // workspace
  DevBuf stage[4];        // host-input staging: R key, R pay, S key, S pay
  DevBuf ping[2];         // pass-1 output tuples (R, S)
  DevBuf pong[2];         // pass-2 output tuples
  DevBuf send[2];         // G>1 device-partition output tuples
  DevBuf recv[2];         // G>1 exchange receive buffers
  DevBuf outst[2];        // host-output staging
  DevBuf small;           // histograms, bounds, work list, counters
  DevBuf route_ws;        // route(): per-CTA destination histograms + totals
  DevBuf xb;              // G>1: local + gathered destination bounds
  DevBuf np_table;        // hape_nonpartitioned_join: the HBM hash table
  unsigned long long* h_res = nullptr;  // pinned: acc[4], out_ctr, (n_items | item_ctr)
  // cached CUDA graph of the local join sequence (keyed by pointers + sizes)
  cudaGraphExec_t gexec = nullptr;
  uintptr_t gkey[18] = {};
  uint32_t g_launches = 0, g_join_ctas = 0;
  bool g_ev_used[HAPE_NSTAGES] = {};
  uint32_t* h_bounds = nullptr;         // pinned: gathered device-partition bounds
  size_t h_bounds_cap = 0;
  // hape_coprocess_join: pinned host co-partitions (R key, R pay, S key, S
  // pay), two device staging sets, copy events (start, end) per set
  void* hp[4] = {};
  size_t hp_cap[4] = {};
  DevBuf cpst[2][4];
  cudaEvent_t ev_h2d[2][2] = {};
  bool in_coprocess = false;            // join_impl: no CUDA-graph capture (sizes change per call)
  // G>1 peer exchange (exchange_p2p): receive buffers (IPC-exportable,
  // grown collectively), the peers' mapped receive buffers, the device
  // table of destination pointers per relation, pinned host scratch
  DevBuf prx[2];
  void* peer_rx[2][64] = {};            // opened IPC mappings (nullptr for self)
  DevBuf peer_tab;                      // [2][G] Tup* destinations
  DevBuf xipc;                          // IPC handle all-gather staging
  uint32_t* h_x = nullptr;              // pinned: [2][G] cursors
  bool p2p_failed = false;              // IPC unavailable: NCCL send/recv from then on
  // hape_debug_loopback_join (peer form): one receive buffer per simulated rank
  DevBuf lb_rx[2][64];
  DevBuf lbuf[2];                       // HAPE_FLAG_LINKED: buffer directory, owner, chain index
  uint32_t xchg_path = 0;               // last call: 0 none, 1 NCCL send/recv, 2 peer scatter
  bool peer_tab_dirty = false;          // peer_tab holds the loopback's table
};

// ---------------------------------------------------------------------------
// error plumbing
// ---------------------------------------------------------------------------
static hape_status fail(hape_join* h, hape_status s, const char* fmt, ...) {
  if (h) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    h->err = buf;
  }
  return s;
}

#define CK(h, call)                                                                      \
  do {                                                                                   \
    cudaError_t e_ = (call);                                                             \
    if (e_ != cudaSuccess) {                                                             \
      (void)cudaGetLastError();                                                          \
      return fail((h), e_ == cudaErrorMemoryAllocation ? HAPE_ERR_OOM : HAPE_ERR_CUDA,   \
                  "%s:%d %s: %s", __FILE__, __LINE__, #call, cudaGetErrorString(e_));    \
    }                                                                                    \
  } while (0)

#define CKN(h, call)                                                                     \
  do {                                                                                   \
    ncclResult_t r_ = (call);                                                            \
    if (r_ != ncclSuccess)                                                               \
      return fail((h), HAPE_ERR_NCCL, "%s:%d %s: %s", __FILE__, __LINE__, #call,         \
                  ncclGetErrorString(r_));                                               \
  } while (0)

#define CKS(call)                         \
  do {                                    \
    hape_status s_ = (call);              \
    if (s_ != HAPE_OK) return s_;         \
  } while (0)

#define CK_LAUNCH(h)                                                                     \
  do {                                                                                   \
    (h)->launches++;                                                                     \
    CK(h, cudaGetLastError());                                                           \
  } while (0)

static int env_int(const char* name, int dflt) {
  const char* e = getenv(name);
  return e ? atoi(e) : dflt;
}

static hape_status ensure(hape_join* h, DevBuf& b, size_t bytes) {
  if (bytes <= b.bytes) return HAPE_OK;
  if (b.p) {
    CK(h, cudaStreamSynchronize(h->stream));
    CK(h, cudaFree(b.p));
    b.p = nullptr;
    b.bytes = 0;
  }
  size_t want = (bytes + 4095) & ~(size_t)4095;
  cudaError_t e = cudaMalloc(&b.p, want);
  if (e != cudaSuccess) {
    (void)cudaGetLastError();
    b.p = nullptr;
    return fail(h, HAPE_ERR_OOM, "cudaMalloc(%zu) failed: %s", want, cudaGetErrorString(e));
  }
  b.bytes = want;
  return HAPE_OK;
}

static void mark(hape_join* h, int stage) {
  // inside a stream capture an "external" record becomes a real event-record
  // node of the graph (a plain record would only express a dependency)
  cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
  cudaStreamIsCapturing(h->stream, &cs);
  if (cs == cudaStreamCaptureStatusActive) cudaEventRecordWithFlags(h->ev[stage], h->stream, cudaEventRecordExternal);
  else cudaEventRecord(h->ev[stage], h->stream);
  h->ev_used[stage] = true;
}

// ---------------------------------------------------------------------------
// plan (a1): bits per pass, co-partition capacity, CTA shapes
// ---------------------------------------------------------------------------
static int key_width(const hape_join_config& c) { return c.key_type == HAPE_INT64 ? 8 : 4; }
static int pay_width(hape_dtype t) { return t == HAPE_INT64 ? 8 : 4; }

static uint32_t cps_for(const hape_join* h, uint64_t total, uint32_t nseg) {
  const uint64_t avg = nseg ? (total + nseg - 1) / nseg : total;
  static const uint64_t chunk = [] { const char* e = getenv("HAPE_CHUNK"); return e ? (uint64_t)atoll(e) : (uint64_t)kChunk; }();
  uint64_t c = (avg + chunk - 1) / chunk;
  const uint64_t want_ctas = (uint64_t)h->num_sms * 8;
  if (c * nseg < want_ctas) {
    uint64_t c2 = (want_ctas + nseg - 1) / nseg;
    static const uint64_t minc = [] { const char* e = getenv("HAPE_MIN_CHUNK"); return e ? (uint64_t)atoll(e) : (uint64_t)kMinChunk; }();
    uint64_t cmax = std::max<uint64_t>(1, (avg + minc - 1) / minc);
    c = std::max<uint64_t>(c, std::min(c2, cmax));
  }
  return (uint32_t)std::max<uint64_t>(1, std::min<uint64_t>(c, 1u << 20));
}

static hape_status make_plan(const hape_join* h, uint64_t n_r, uint64_t n_s, hape_plan* p) {
  const hape_join_config& c = h->cfg;
  memset(p, 0, sizeof *p);
  const uint32_t HW = key_width(c) * 8;
  const int world = c.world_size > 1 ? c.world_size : 1;
  p->dest_bits = ceil_log2_u64((uint64_t)world);
  uint32_t need = 0;
  while ((n_r >> need) > kTargetPerPartition) need++;
  // a 17-bit plan would lose the one-read joint histogram of both passes
  // (k_hist_joint counts at most 2^16 joint buckets); one bit less keeps it,
  // at ~4096 R tuples per co-partition -- worth it while S is not much larger
  // than R (measured: C4's 2^28-per-rank share 6.46 -> 6.24 ms; C5, |S| = 4|R|,
  // 16.61 -> 17.42 ms at theta 0.5: the larger co-partitions cost the probe
  // more than the histogram read saves).  HAPE_PLAN16=0: plain 17-bit plans.
  static const int plan16 = env_int("HAPE_PLAN16", 1);
  if (plan16 && need == 17 && n_s <= 2 * n_r && !c.radix_passes && !c.radix_bits[0]) need = 16;
  uint32_t passes = c.radix_passes ? (uint32_t)c.radix_passes : (need <= kMaxSinglePassBits ? 1u : 2u);
  uint32_t b1, b2;
  if (c.radix_bits[0] > 0) {
    b1 = (uint32_t)c.radix_bits[0];
    b2 = passes == 2 ? (uint32_t)std::max(0, c.radix_bits[1]) : 0u;
  } else if (passes == 1) {
    // at least 2 co-partitions: k_join_oa's free-slot test needs a
    // co-partition other than q to exist (join_oa.cuh)
    b1 = std::max(1u, std::min(need, kMaxBitsPerPass));
    b2 = 0;
  } else {
    b1 = std::min((need + 1) / 2, kMaxBitsPerPass);
    b2 = std::min(need - std::min(need, b1), kMaxBitsPerPass);
  }
  if (b1 > kMaxBitsPerPass || b2 > kMaxBitsPerPass) return HAPE_ERR_INVALID_ARG;
  if (b1 + b2 + p->dest_bits > HW) return HAPE_ERR_INVALID_ARG;
  p->passes = passes;
  p->bits[0] = b1;
  p->bits[1] = b2;
  const uint64_t Q = 1ull << (b1 + b2);
  const uint64_t expected = (n_r + Q - 1) / Q;
  // R chunk capacity: mean + 12.5% (+64) covers the hash spread of a uniform
  // co-partition (sigma = sqrt(mean)); larger co-partitions are chunked (R6)
  // R chunk capacity: mean + 12.5% (+64) covers the hash spread of a uniform
  // co-partition (sigma = sqrt(mean)); larger co-partitions are chunked (R6).
  // Heads: 2^sb >= ~2x the chunk (load factor ~0.5); HAPE_SLOT_EXTRA (tuning)
  // shifts the exponent.  Both shrink until the table fits ~2 CTAs per SM.
  int extra = 0;
  if (const char* e = getenv("HAPE_SLOT_EXTRA")) extra = atoi(e);
  const int prw = pay_width(c.r_payload_type), kwb = key_width(c);
  uint64_t cap = expected + expected / 8 + 64;
  cap = std::max<uint64_t>(256, std::min<uint64_t>(cap, JN_MAXCAP));
  cap = (cap + 127) & ~127ull;
  uint32_t sb = 0;
  while (true) {
    const int sbi = (int)ceil_log2_u64(std::min<uint64_t>(std::max<uint64_t>(expected, 1), cap)) + extra;
    sb = (uint32_t)std::max(6, std::min(sbi, 14));
    const size_t bytes = 2 * ((cap * kwb + 47) / 16 * 16 + (cap * prw + 47) / 16 * 16) + (cap * 2 + 15) / 16 * 16 +
                         (sizeof(JnHead) << sb);
    if (bytes <= 110 * 1024 || cap <= 256) break;
    cap -= 128;
  }
  p->build_cap = (uint32_t)cap;
  p->slot_shift = 0;  // slots use a multiplicative hash of the key (kernels.cuh jn_slot)
  p->slot_bits = sb;
  p->probe_slice = 16384;
  p->ctas_per_seg[0] = cps_for(h, n_r, 1);
  p->ctas_per_seg[1] = passes == 2 ? cps_for(h, n_r, 1u << b1) : 0;
  p->join_ctas = 0;  // filled at launch (occupancy)
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// kernel launchers (dtype dispatch)
// ---------------------------------------------------------------------------
// A relation as a partitioning pass sees it: SoA columns or AoS tuples.
struct Src {
  PartIn in;
  bool aos;
  uint32_t n;
  int pw;
};

static size_t tup_bytes(int kw, int pw) { return (kw + pw) <= 8 ? 8 : 16; }

// Workspace (AoS) tuples carry h(k) in their key field (kernels.cuh
// HAPE_STORE_H): passes over them take buckets from it directly (IDENT)
static bool ident_for(const hape_join* h, bool aos) {
  return (HAPE_STORE_H && aos) || h->cfg.part_fn == HAPE_PART_IDENTITY;
}

template <int KW, int PW, bool AOS>
static void hist_t(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, uint32_t* hist, uint32_t* rowsum) {
  const unsigned grid = m.nseg * m.cps;
  if (ident_for(h, AOS))
    k_hist<KW, PW, AOS, true><<<grid, HIST_THREADS, (size_t)P * 4, h->stream>>>(s.in, m, bf, P, hist, rowsum);
  else
    k_hist<KW, PW, AOS, false><<<grid, HIST_THREADS, (size_t)P * 4, h->stream>>>(s.in, m, bf, P, hist, rowsum);
}

static hape_status launch_hist(hape_join* h, int kw, const Src& s, SegMap m, BitField bf, uint32_t P, uint32_t* hist,
                               uint32_t* rowsum) {
  if (m.nseg * m.cps == 0) return HAPE_OK;
  const int pw = s.pw;
  if (s.aos) {
    if (kw == 4 && pw == 4) hist_t<4, 4, true>(h, s, m, bf, P, hist, rowsum);
    else if (kw == 4) hist_t<4, 8, true>(h, s, m, bf, P, hist, rowsum);
    else if (pw == 4) hist_t<8, 4, true>(h, s, m, bf, P, hist, rowsum);
    else hist_t<8, 8, true>(h, s, m, bf, P, hist, rowsum);
  } else {
    if (kw == 4) hist_t<4, 4, false>(h, s, m, bf, P, hist, rowsum);  // keys only: PW irrelevant
    else hist_t<8, 8, false>(h, s, m, bf, P, hist, rowsum);
  }
  CK_LAUNCH(h);
  return HAPE_OK;
}

// Two-pass plans with B1 + B2 <= 16 count both passes' buckets in one read of
// the keys (k_hist_joint) and run pass 2 as a claiming scatter.  HAPE_JOINT=0
// forces the separate pass-2 histogram (tests compare both forms).
// HAPE_FLAG_LINKED: two-pass plans run pass 1 as the paper's single-scan
// linked-buffer partitioning (no histogram before it; pass 2 reads the
// chains and counts its own buckets)
static bool use_linked(const hape_join* h, const hape_plan& pl) {
  return (h->cfg.flags & HAPE_FLAG_LINKED) && pl.passes == 2;
}

static bool use_joint(const hape_join* h, const hape_plan& pl) {
  static const int env = [] { const char* e = getenv("HAPE_JOINT"); return e ? atoi(e) : 1; }();
  return env != 0 && !use_linked(h, pl) && pl.passes == 2 && pl.bits[0] + pl.bits[1] <= 16 &&
         pl.bits[0] + pl.bits[1] >= 6 && pl.bits[1] >= 1;
}

// Plans the joint histogram cannot count (one pass, or B1 + B2 > 16) still
// claim their scatter runs: each pass counts only its bucket totals (k_hist
// without per-CTA rows), a one-CTA-per-row scan turns the totals into bounds
// and claim cursors, and the scatter claims runs from the cursors (the
// per-CTA offset form costs 0.38-0.49 of the HBM roofline at 2^20 buckets:
// runs of a few tuples per CTA chunk).  HAPE_CLAIM=0 keeps the per-CTA form.
static bool use_claim(const hape_join* h, const hape_plan& pl) {
  static const int env = [] { const char* e = getenv("HAPE_CLAIM"); return e ? atoi(e) : 1; }();
  return (env != 0 || use_linked(h, pl)) && !use_joint(h, pl);
}

static uint32_t joint_grid(const hape_join* h, uint32_t nchunks) {
  return std::max<uint32_t>(1, std::min<uint32_t>((uint32_t)h->num_sms, nchunks));
}

static size_t joint_smem(uint32_t P1, uint32_t P2, bool tma = false) {
  if (!tma) return (size_t)P1 * P2 * 2 + (size_t)P1 * 4;
  return hj_ring_off(P1 * P2 / 2, P1) + (size_t)HJ_NS * HJ_SB + 2 * HJ_NS * 8 + HJ_NS * 4 + 64;
}

// TMA-fed joint histogram where the ring fits beside the counters, only
// with HAPE_HJ_TMA=1: measured 0.452 vs 0.273 ms for C2 (the 64 KB ring
// gives each of the 992 consumer threads one 16-byte vector per stage, so
// the per-stage mbarrier round trip dominates; the register-batched form
// keeps 4 vectors per thread in flight with no synchronisation)
static bool hj_tma(uint32_t P1, uint32_t P2) {
  static const int env = env_int("HAPE_HJ_TMA", 0);
  return env != 0 && joint_smem(P1, P2, true) <= 200 * 1024;
}

// cudaFuncSetAttribute applies to the current device only: one bit per
// device ordinal and kernel instantiation (the caller's `mask` is a static
// of the instantiating template)
template <class F>
static hape_status smem_attr(hape_join* h, F kern, int bytes, uint64_t& mask) {
  const uint64_t bit = 1ull << (h->dev & 63);
  if (mask & bit) return HAPE_OK;
  CK(h, cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes));
  mask |= bit;
  return HAPE_OK;
}

template <int KW, int PW, bool AOS, bool IDENT>
static hape_status hist_joint_t(hape_join* h, const Src& s, SegMap m, BitField bf1, BitField bf2, uint32_t P1,
                                uint32_t P2, uint32_t* rowsum, uint16_t* part, uint32_t* ovf) {
  const uint32_t nch = m.nseg * m.cps;
  if (hj_tma(P1, P2)) {
    auto kern = k_hist_joint<KW, PW, AOS, IDENT, true>;
    static uint64_t attr_dev = 0;
    CKS(smem_attr(h, kern, 200 * 1024, attr_dev));
    kern<<<joint_grid(h, nch), HJ_THREADS, joint_smem(P1, P2, true), h->stream>>>(s.in, m, P1, P2, rowsum, part,
                                                                                ovf);
    return HAPE_OK;
  }
  auto kern = k_hist_joint<KW, PW, AOS, IDENT>;
  static uint64_t attr_dev = 0;
  CKS(smem_attr(h, kern, 200 * 1024, attr_dev));
  kern<<<joint_grid(h, nch), HJ_THREADS, joint_smem(P1, P2), h->stream>>>(s.in, m, P1, P2, rowsum, part,
                                                                        ovf);
  return HAPE_OK;
}

template <int KW, int PW, bool AOS>
static hape_status hist_joint_i(hape_join* h, const Src& s, SegMap m, BitField bf1, BitField bf2, uint32_t P1,
                                uint32_t P2, uint32_t* rowsum, uint16_t* part, uint32_t* ovf) {
  if (ident_for(h, AOS))
    return hist_joint_t<KW, PW, AOS, true>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
  return hist_joint_t<KW, PW, AOS, false>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
}

static hape_status launch_hist_joint(hape_join* h, int kw, const Src& s, SegMap m, BitField bf1, BitField bf2,
                                     uint32_t P1, uint32_t P2, uint32_t* rowsum, uint16_t* part, uint32_t* ovf) {
  if (m.nseg * m.cps == 0) return HAPE_OK;
  const int pw = s.pw;
  hape_status st;
  if (s.aos) {
    if (kw == 4 && pw == 4) st = hist_joint_i<4, 4, true>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
    else if (kw == 4) st = hist_joint_i<4, 8, true>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
    else if (pw == 4) st = hist_joint_i<8, 4, true>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
    else st = hist_joint_i<8, 8, true>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
  } else {
    if (kw == 4) st = hist_joint_i<4, 4, false>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
    else st = hist_joint_i<8, 8, false>(h, s, m, bf1, bf2, P1, P2, rowsum, part, ovf);
  }
  CKS(st);
  CK_LAUNCH(h);
  return HAPE_OK;
}

// nrel relations' joint reductions in one launch (grid.y = relation: R's
// and S's 2 x 256-row reductions fill the GPU together, C2 2 x 24 us -> one)
static hape_status launch_joint_reduce(hape_join* h, const JrArgs* a, int nrel, uint32_t P1, uint32_t P2) {
  JrArgs2 args{};
  for (int i = 0; i < nrel; i++) args.r[i] = a[i];
  k_joint_reduce<<<dim3(P1, (unsigned)nrel), JR_THREADS, 0, h->stream>>>(args, P1, P2);
  CK_LAUNCH(h);
  return HAPE_OK;
}

static hape_status launch_scan(hape_join* h, SegMap m, uint32_t P, uint32_t* hist, const uint32_t* rowsum,
                               uint32_t* bounds_out) {
  uint32_t rpc = std::max<uint32_t>(1, SCAN_TILE / m.cps);
  rpc = std::min(rpc, P);
  const uint32_t groups = (P + rpc - 1) / rpc;
  k_scan<<<m.nseg * groups, SCAN_THREADS, 0, h->stream>>>(hist, rowsum, m, P, rpc, bounds_out);
  CK_LAUNCH(h);
  return HAPE_OK;
}

// dynamic shared memory a scatter CTA may opt into (B200: 227 KB per block)
constexpr size_t kScatterSmemMax = 232448 - 1024;

template <int KW, int PW, bool AOS, class C, bool IDENT, bool CLAIM, bool LINKED = false>
static hape_status scatter_t(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, uint32_t* offs,
                             void* out, const LinkMap* lk = nullptr) {
  const size_t smem = ScLayout<KW, PW, AOS, C>::bytes(P, false, LINKED);
  static uint64_t attr_dev = 0;
  auto kern = k_scatter<KW, PW, AOS, C, IDENT, CLAIM, false, LINKED>;
  CKS(smem_attr(h, kern, (int)kScatterSmemMax, attr_dev));
  const unsigned grid = m.nseg * m.cps;
  if (grid == 0) return HAPE_OK;
  // warp-aggregated ranking: always for narrow fan-outs (the destination
  // route, P <= 64: lanes share buckets), else HAPE_SC_AGG=1
  // (wider fan-outs: HAPE_SC_AGG=1 match_any form, 2 the hot-bucket form)
  static const uint32_t agg_env = (uint32_t)env_int("HAPE_SC_AGG", 0);
  const uint32_t agg = P <= 64 ? 1u : agg_env;
  kern<<<grid, C::NT, smem, h->stream>>>(s.in, m, bf, P, offs, static_cast<Tup<KW, PW>*>(out), nullptr, agg,
                                         lk ? *lk : LinkMap{});
  CK_LAUNCH(h);
  return HAPE_OK;
}

// pass 1 of the linked-buffer partitioning (k_scatter LINKED): the shape
// the hist path would use where it fits with the chain arrays (wide tiles
// for >= 1024 buckets), else a smaller tile (runs <= one tile <= a buffer)
template <int KW, int PW, bool AOS, class C>
static hape_status scatter_linked_c(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, void* out,
                                    const LinkMap& lk) {
  if (ident_for(h, AOS))
    return scatter_t<KW, PW, AOS, C, true, true, true>(h, s, m, bf, P, lk.cnt, out, &lk);
  return scatter_t<KW, PW, AOS, C, false, true, true>(h, s, m, bf, P, lk.cnt, out, &lk);
}

template <int KW, int PW, bool AOS>
static hape_status scatter_linked_v(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, void* out,
                                    const LinkMap& lk) {
  using Cd = typename std::conditional<KW + PW <= 8, ScCfg<512, 13, 2, 2>, ScCfg<384, 9, 2, 2>>::type;
  using Cw = ScCfg<1024, 12, 2, 1>;
  using Cs = ScCfg<256, 8, 2, 1>;
  if (KW + PW <= 8 && P >= 1024 && ScLayout<KW, PW, AOS, Cw>::bytes(P, false, true) <= kScatterSmemMax)
    return scatter_linked_c<KW, PW, AOS, Cw>(h, s, m, bf, P, out, lk);
  if (ScLayout<KW, PW, AOS, Cd>::bytes(P, false, true) <= kScatterSmemMax)
    return scatter_linked_c<KW, PW, AOS, Cd>(h, s, m, bf, P, out, lk);
  return scatter_linked_c<KW, PW, AOS, Cs>(h, s, m, bf, P, out, lk);
}

static hape_status launch_scatter_linked(hape_join* h, int kw, const Src& s, SegMap m, BitField bf, uint32_t P,
                                         void* out, const LinkMap& lk) {
  const int pw = s.pw;
#define HAPE_SCL(AOS)                                                                  \
  if (kw == 4 && pw == 4) return scatter_linked_v<4, 4, AOS>(h, s, m, bf, P, out, lk); \
  if (kw == 4) return scatter_linked_v<4, 8, AOS>(h, s, m, bf, P, out, lk);            \
  if (pw == 4) return scatter_linked_v<8, 4, AOS>(h, s, m, bf, P, out, lk);            \
  return scatter_linked_v<8, 8, AOS>(h, s, m, bf, P, out, lk);
  if (s.aos) { HAPE_SCL(true) } else { HAPE_SCL(false) }
#undef HAPE_SCL
}

// linked-buffer geometry: buffers of eight default scatter tiles (pass 2
// reads whole tiles, one CTA per buffer: 2-tile buffers measured 48.5 vs
// 23.3 ms for C4's pass 2 -- per-CTA set-up), a dense directory row of kmax
// entries per pass-1 bucket
static uint32_t lb_buf(size_t tb) { return tb <= 8 ? 8u * 512u * 13u : 8u * 384u * 9u; }
static uint64_t lb_nbuf(uint64_t n, size_t tb, uint32_t P1) { return (n + lb_buf(tb) - 1) / lb_buf(tb) + P1; }
static uint64_t lb_kmax(uint64_t n, size_t tb) { return (n + lb_buf(tb) - 1) / lb_buf(tb) + 1; }
// linked pass 1: directory [P1][kmax] + owner [nbuf] + chain index [nbuf]
static size_t lb_ws_bytes(uint64_t n, size_t tb, uint32_t P1) {
  return (size_t)P1 * lb_kmax(n, tb) * 4 + 2 * lb_nbuf(n, tb, P1) * 4 + 64;
}

// scatter shape per tuple width (measured best of the ScCfg sweep);
// (the destination-table variant ScCfg<..., DST=true> is no longer dispatched)
template <int KW, int PW, bool AOS, bool IDENT, bool CLAIM>
static hape_status scatter_i(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, uint32_t* offs,
                             void* out) {
  static int v = [] { const char* e = getenv("HAPE_SC"); return e ? atoi(e) : 0; }();
  // measured (round 1): 8-byte tuples <512,13,2,2> (C2 scatters 1.09/1.03 ->
  // 0.96/0.93 ms vs <512,8,3,2>; <512,12,2,2> slower); 16-byte tuples
  // <384,9,2,2> (C3 7.95/7.04 -> 7.10/6.89 ms vs <256,8,2,3>).  The largest
  // tile two CTAs per SM can stage wins: longer bucket runs per tile
  // (P585-589: more staged tuples per partition -> longer runs -> better
  // store coalescing).  (The swept alternatives are no longer instantiated.)
  if constexpr (KW + PW <= 8) {
    // wide fan-outs (>= 1024 buckets): one CTA per SM staging twice the tile
    // (longer runs per bucket and tile); HAPE_SC=3 forces it, used for P >= 1024 unless HAPE_SC_WIDE=0
    // (measured C4 at N=1, 2 x 1024 buckets: scatters 25.0 / 23.3 -> 18.8 / 18.4 ms;
    // on 256 / 512 buckets it is slower: C2 0.94 -> 1.08 ms, C5 4.92 -> 5.43 ms)
    static int wide = [] { const char* e = getenv("HAPE_SC_WIDE"); return e ? atoi(e) : 1; }();
    using Cw = ScCfg<1024, 12, 2, 1>;
    if (v == 3 || (wide && P >= 1024 && ScLayout<KW, PW, AOS, Cw>::bytes(P) <= kScatterSmemMax))
      return scatter_t<KW, PW, AOS, Cw, IDENT, CLAIM>(h, s, m, bf, P, offs, out);
    return scatter_t<KW, PW, AOS, ScCfg<512, 13, 2, 2>, IDENT, CLAIM>(h, s, m, bf, P, offs, out);
  } else {
    return scatter_t<KW, PW, AOS, ScCfg<384, 9, 2, 2>, IDENT, CLAIM>(h, s, m, bf, P, offs, out);
  }
}

template <int KW, int PW, bool AOS>
static hape_status scatter_v(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, uint32_t* offs,
                             void* out, bool claim) {
  if (claim) {
    if (ident_for(h, AOS)) return scatter_i<KW, PW, AOS, true, true>(h, s, m, bf, P, offs, out);
    return scatter_i<KW, PW, AOS, false, true>(h, s, m, bf, P, offs, out);
  }
  if (ident_for(h, AOS)) return scatter_i<KW, PW, AOS, true, false>(h, s, m, bf, P, offs, out);
  return scatter_i<KW, PW, AOS, false, false>(h, s, m, bf, P, offs, out);
}

static hape_status launch_scatter(hape_join* h, int kw, const Src& s, SegMap m, BitField bf, uint32_t P,
                                  uint32_t* offs, void* out, bool claim = false) {
  const int pw = s.pw;
#define HAPE_SC_DISPATCH(AOS)                                                        \
  if (kw == 4 && pw == 4) return scatter_v<4, 4, AOS>(h, s, m, bf, P, offs, out, claim); \
  if (kw == 4) return scatter_v<4, 8, AOS>(h, s, m, bf, P, offs, out, claim);            \
  if (pw == 4) return scatter_v<8, 4, AOS>(h, s, m, bf, P, offs, out, claim);            \
  return scatter_v<8, 8, AOS>(h, s, m, bf, P, offs, out, claim);
  if (s.aos) { HAPE_SC_DISPATCH(true) } else { HAPE_SC_DISPATCH(false) }
#undef HAPE_SC_DISPATCH
}

// the fused destination partition + exchange scatter (k_scatter PEER): SoA
// caller columns in, claimed runs straight into each destination's buffer
template <int KW, int PW, bool IDENT>
static hape_status peer_scatter_t(hape_join* h, const Src& s, SegMap m, BitField bf, uint32_t P, uint32_t* offs,
                                  void* const* peers) {
  using C = ScCfg<512, 13, 2, 2>;
  using Cw = typename std::conditional<KW + PW <= 8, C, ScCfg<384, 9, 2, 2>>::type;
  auto kern = k_scatter<KW, PW, false, Cw, IDENT, true, true>;
  const size_t smem = ScLayout<KW, PW, false, Cw>::bytes(P, true);
  static uint64_t attr_dev = 0;
  CKS(smem_attr(h, kern, 220 * 1024, attr_dev));
  const unsigned grid = m.nseg * m.cps;
  if (grid == 0) return HAPE_OK;
  // few destinations: the lanes of a warp share buckets -- warp-aggregated
  // ranking (HAPE_SC_AGG_PEER=0 disables)
  static const uint32_t agg = (uint32_t)env_int("HAPE_SC_AGG_PEER", 1);
  kern<<<grid, Cw::NT, smem, h->stream>>>(s.in, m, bf, P, offs, nullptr,
                                         reinterpret_cast<Tup<KW, PW>* const*>(peers), agg, LinkMap{});
  CK_LAUNCH(h);
  return HAPE_OK;
}

static hape_status launch_peer_scatter(hape_join* h, int kw, const Src& s, SegMap m, BitField bf, uint32_t P,
                                       uint32_t* offs, void* const* peers) {
  if (s.aos) return fail(h, HAPE_ERR_UNSUPPORTED, "peer scatter reads SoA columns");
  const int pw = s.pw;
  const bool id = h->cfg.part_fn == HAPE_PART_IDENTITY;
#define HAPE_PS(KW, PW) return id ? peer_scatter_t<KW, PW, true>(h, s, m, bf, P, offs, peers) \
                                 : peer_scatter_t<KW, PW, false>(h, s, m, bf, P, offs, peers)
  if (kw == 4 && pw == 4) HAPE_PS(4, 4);
  if (kw == 4) HAPE_PS(4, 8);
  if (pw == 4) HAPE_PS(8, 4);
  HAPE_PS(8, 8);
#undef HAPE_PS
}

// Build+probe shape: SR kernels (SU > 0) stage S through a smem tile ring of
// SU*256-tuple tiles (the materialising and 16-byte-tuple forms, whose probe
// cannot keep a software-pipelined S batch in registers); the others read S
// straight from HBM with a register-pipelined batch.  HAPE_JN_SU=0/1/2/4
// forces the form, HAPE_JN_NRB / HAPE_JN_NSB the ring depths (tuning only).

template <int KW, int PRW, int PSW, bool MAT, int SU, int NC = 256, int LAY = JN_AOS>
static hape_status launch_join_t(hape_join* h, const JoinArgs& a_in, uint32_t* ctas_out) {
  constexpr bool SR = SU > 0;
  constexpr int JN_THREADS = NC + 32;
  auto kern = k_build_probe<KW, PRW, PSW, MAT, SU, NC, LAY>;
  JoinArgs a = a_in;
  static const int nrb_env = env_int("HAPE_JN_NRB", 0), nsb_env = env_int("HAPE_JN_NSB", 0);
  a.nsb = SR ? (uint32_t)std::min(8, std::max(2, nsb_env ? nsb_env : (SU >= 4 ? 3 : 2))) : 0u;
  a.nrb = (uint32_t)std::min(2, std::max(1, nrb_env ? nrb_env : 2));
  static uint64_t attr_dev = 0;
  CKS(smem_attr(h, kern, 200 * 1024, attr_dev));
  auto occ = [&](uint32_t sb, uint32_t nrb, int* per_sm) -> hape_status {
    const size_t smem = join_smem_bytes<KW, PRW, PSW, SU, NC, LAY>(a.cap, sb, nrb, a.nsb);
    *per_sm = 0;
    if (smem > 200 * 1024) return HAPE_OK;
    CK(h, cudaOccupancyMaxActiveBlocksPerMultiprocessor(per_sm, kern, JN_THREADS, smem));
    return HAPE_OK;
  };
  int per_sm = 0;
  CKS(occ(a.slot_bits, a.nrb, &per_sm));
  // a single R buffer when the second one would cost a CTA per SM (the
  // other resident CTAs cover the R load at a stage boundary).  The direct
  // form also takes a single R buffer when that buys a larger head array at
  // the same occupancy (C2: 2^12 heads instead of 2^11, 4 CTAs per SM either
  // way -- build+probe 0.742 -> 0.717 ms, profiles/r2/ab_build_probe_nrb.jsonl); shorter
  // chains are worth more than covering the R load of a stage boundary
  if (!nrb_env && a.nrb == 2) {
    int p1 = 0;
    CKS(occ(a.slot_bits, 1, &p1));
    if (p1 > per_sm) { a.nrb = 1; per_sm = p1; }
    else if (!SR && p1 == per_sm && a.slot_bits < 14) {
      int p2 = 0, p1b = 0;
      CKS(occ(a.slot_bits + 1, 2, &p2));
      CKS(occ(a.slot_bits + 1, 1, &p1b));
      if (p2 < per_sm && p1b == per_sm) a.nrb = 1;
    }
  }
  if (per_sm < 1)
    return fail(h, HAPE_ERR_UNSUPPORTED, "build+probe does not fit: smem %zu",
                join_smem_bytes<KW, PRW, PSW, SU, NC, LAY>(a.cap, a.slot_bits, a.nrb, a.nsb));
  // plan.slot_bits is the minimum table size: one more bit (shorter chains)
  // when the larger head array costs no occupancy (register-limited kernels)
  while (a.slot_bits < 14) {
    int per_sm2 = 0;
    CKS(occ(a.slot_bits + 1, a.nrb, &per_sm2));
    if (per_sm2 != per_sm) break;
    a.slot_bits = a.slot_bits + 1;
  }
  const size_t smem_used = join_smem_bytes<KW, PRW, PSW, SU, NC, LAY>(a.cap, a.slot_bits, a.nrb, a.nsb);
  const unsigned grid = (unsigned)(per_sm * h->num_sms);
  *ctas_out = grid;
  kern<<<grid, JN_THREADS, smem_used, h->stream>>>(a);
  CK_LAUNCH(h);
  return HAPE_OK;
}

template <int KW, int PRW, int PSW>
static hape_status launch_join_m(hape_join* h, const JoinArgs& a, bool mat, uint32_t* ctas) {
  // S tile tuples per thread of the SR form (0 = direct S loads); consumer
  // threads per CTA (SR: 512, direct: 256)
  // Measured (C3 build+probe): direct 14.1 ms; SR 256 threads, 1024-tuple
  // tiles 12.4; SR 512 threads, 1024-tuple tiles 10.7 ms.  C2 (8-byte tuples,
  // no pairs): direct 256 threads 0.74 ms, every SR / 512-thread form slower.
  // (the swept SU = 1 / 4 depths and the 512-thread direct form are no
  // longer instantiated; HAPE_JN_SU=2 forces the SR form, 0 the direct form)
  static const int su_env = env_int("HAPE_JN_SU", -1);
  const bool sr_form = su_env >= 0 ? su_env > 0 : (mat || KW + PSW > 8);
  if (sr_form) {
    if (mat) return launch_join_t<KW, PRW, PSW, true, 2, 512>(h, a, ctas);
    return launch_join_t<KW, PRW, PSW, false, 2, 512>(h, a, ctas);
  }
  // table layout (kernels.cuh JN_*): key|next nodes (one shared load per
  // chain hop) for bag semantics, whose probes walk every chain to its end
  // (C2 bag build+probe 1.023 -> 0.907 ms); a declared-unique build side
  // stops at the first match, where the 8-byte node loads cost more bank
  // conflicts than the hop saves (0.722 -> 1.020 ms).  HAPE_JN_LAY=0/1/2
  // forces the layout (A/B, tests)
  static const int lay_env = env_int("HAPE_JN_LAY", -1);
  const int lay = lay_env >= 0 ? lay_env : (a.r_unique == 0 ? JN_KN : JN_AOS);
  if (lay == JN_KN) {
    if (mat) return launch_join_t<KW, PRW, PSW, true, 0, 256, JN_KN>(h, a, ctas);
    return launch_join_t<KW, PRW, PSW, false, 0, 256, JN_KN>(h, a, ctas);
  }
  if (lay == JN_SK) {
    if (mat) return launch_join_t<KW, PRW, PSW, true, 0, 256, JN_SK>(h, a, ctas);
    return launch_join_t<KW, PRW, PSW, false, 0, 256, JN_SK>(h, a, ctas);
  }
  if (mat) return launch_join_t<KW, PRW, PSW, true, 0, 256>(h, a, ctas);
  // large co-partitions (R chunks beyond ~3 K tuples: 16-bit plans over
  // 2^28-tuple relations, C4's share at N = 8) run 512 consumer threads at 2
  // CTAs per SM with a 2^13-slot table, where the 256-thread form drops to 3
  // CTAs per SM at load factor 1 (C4/8 build+probe 1.466 -> 1.215 ms, 0.45 ->
  // 0.54 of HBM); so do probe-heavy joins (|S| >= 2|R|: C5's 4 S tuples per R
  // tuple, 3.82 -> 3.36 ms), where more probes share each build; 2 K-tuple
  // co-partitions with |S| = |R| stay on 256 (C2 0.643 vs 0.664 ms).
  // HAPE_JN_NC=256/512 forces the shape (A/B)
  static const int nc_env = env_int("HAPE_JN_NC", 0);
  if (KW + PSW <= 8 && (nc_env == 512 || (nc_env == 0 && (a.cap > 3072 || a.probe_heavy))))
    return launch_join_t<KW, PRW, PSW, false, 0, 512>(h, a, ctas);
  return launch_join_t<KW, PRW, PSW, false, 0, 256>(h, a, ctas);
}

// Open-addressing build+probe (join_oa.cuh).  Shape: 256 threads for
// 8-byte R tuples, 512 for 16-byte ones (the R chunk lives in registers:
// OA_CAPMAX / NC tuples per thread); NTAB = 2 tables (one barrier per stage)
// when two still fit 2+ CTAs per SM, else 1; U = 2 S tuples per thread per
// batch.  HAPE_OA_SB (extra slot bits) tunes the
// int32 form.  HAPE_JN_OA=1 selects it (default: the chained k_build_probe).
template <int KW, int PRW, int PSW, bool MAT, bool IDENT, int NC, int NTAB, int U>
static hape_status launch_oa_t(hape_join* h, const JoinArgs& a_in, uint32_t* ctas_out) {
  auto kern = k_join_oa<KW, PRW, PSW, MAT, IDENT, NC, NTAB, U>;
  JoinArgs a = a_in;
  constexpr uint32_t capmax = (uint32_t)((OA_CAPMAX + NC - 1) / NC) * NC;
  a.cap = std::min(a.cap, capmax);
  static const int sb_extra = env_int("HAPE_OA_SB", 0);
  const int sb = std::max(6, std::min(15, (int)ceil_log2_u64((uint64_t)a.cap + 1) + sb_extra));
  a.slot_bits = (uint32_t)sb;
  const size_t smem = oa_smem_bytes<KW, PRW, NC, NTAB>((uint32_t)sb);
  if (smem > 200 * 1024) return fail(h, HAPE_ERR_UNSUPPORTED, "open-addressing table does not fit: %zu B", smem);
  static uint64_t attr_dev = 0;
  CKS(smem_attr(h, kern, 200 * 1024, attr_dev));
  int per_sm = 0;
  CK(h, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, NC, smem));
  if (per_sm < 1) return fail(h, HAPE_ERR_UNSUPPORTED, "open-addressing build+probe does not fit");
  const unsigned grid = (unsigned)(per_sm * h->num_sms);
  *ctas_out = grid;
  kern<<<grid, NC, smem, h->stream>>>(a);
  CK_LAUNCH(h);
  return HAPE_OK;
}

template <int KW, int PRW, int PSW, bool MAT, bool IDENT>
static hape_status launch_oa_m(hape_join* h, const JoinArgs& a, uint32_t* ctas) {
  constexpr bool W8 = sizeof(Tup<KW, PRW>) == 8;
  constexpr int NC = W8 ? 256 : 512;
  // (measured shapes, C2: NTAB 1 3.81 / 2 4.03 ms, U 1 / 2 / 4 within 1 %;
  // only the default is instantiated)
  return launch_oa_t<KW, PRW, PSW, MAT, IDENT, NC, W8 ? 2 : 1, 2>(h, a, ctas);
}

template <int KW, int PRW, int PSW>
static hape_status launch_oa_w(hape_join* h, const JoinArgs& a, bool mat, uint32_t* ctas) {
  const bool ident = ident_for(h, true);  // the workspace tuples' key field holds h(k)
  if (mat) return ident ? launch_oa_m<KW, PRW, PSW, true, true>(h, a, ctas)
                        : launch_oa_m<KW, PRW, PSW, true, false>(h, a, ctas);
  return ident ? launch_oa_m<KW, PRW, PSW, false, true>(h, a, ctas)
               : launch_oa_m<KW, PRW, PSW, false, false>(h, a, ctas);
}

static hape_status launch_join(hape_join* h, int kw, int prw, int psw, const JoinArgs& a, bool mat,
                               uint32_t* ctas) {
  // (the open-addressing form measured 4.0 vs 0.73 ms for the C2
  // build+probe: linear probing pays the longest walk of 32 lanes per warp
  // step and a partition-hash free-slot test per visited slot)
  static const int oa = env_int("HAPE_JN_OA", 0);
  if (oa) {
    if (kw == 4) {
      if (prw == 4) return psw == 4 ? launch_oa_w<4, 4, 4>(h, a, mat, ctas) : launch_oa_w<4, 4, 8>(h, a, mat, ctas);
      return psw == 4 ? launch_oa_w<4, 8, 4>(h, a, mat, ctas) : launch_oa_w<4, 8, 8>(h, a, mat, ctas);
    }
    if (prw == 4) return psw == 4 ? launch_oa_w<8, 4, 4>(h, a, mat, ctas) : launch_oa_w<8, 4, 8>(h, a, mat, ctas);
    return psw == 4 ? launch_oa_w<8, 8, 4>(h, a, mat, ctas) : launch_oa_w<8, 8, 8>(h, a, mat, ctas);
  }
  if (kw == 4) {
    if (prw == 4) return psw == 4 ? launch_join_m<4, 4, 4>(h, a, mat, ctas) : launch_join_m<4, 4, 8>(h, a, mat, ctas);
    return psw == 4 ? launch_join_m<4, 8, 4>(h, a, mat, ctas) : launch_join_m<4, 8, 8>(h, a, mat, ctas);
  }
  if (prw == 4) return psw == 4 ? launch_join_m<8, 4, 4>(h, a, mat, ctas) : launch_join_m<8, 4, 8>(h, a, mat, ctas);
  return psw == 4 ? launch_join_m<8, 8, 4>(h, a, mat, ctas) : launch_join_m<8, 8, 8>(h, a, mat, ctas);
}

static hape_status launch_unpack(hape_join* h, int kw, int pw, const void* t, uint32_t n, void* k, void* p) {
  if (!n) return HAPE_OK;
  const unsigned grid = std::min<unsigned>((n + 255) / 256, 4096);
  // workspace tuples hold h(k): hand the key back (HAPE_STORE_H)
  const uint32_t um = (HAPE_STORE_H && h->cfg.part_fn == HAPE_PART_HASH) ? 1u : 0u;
  if (kw == 4 && pw == 4) k_unpack<4, 4><<<grid, 256, 0, h->stream>>>((const Tup<4, 4>*)t, n, (uint32_t*)k, (uint32_t*)p, um);
  else if (kw == 4) k_unpack<4, 8><<<grid, 256, 0, h->stream>>>((const Tup<4, 8>*)t, n, (uint32_t*)k, (uint64_t*)p, um);
  else if (pw == 4) k_unpack<8, 4><<<grid, 256, 0, h->stream>>>((const Tup<8, 4>*)t, n, (uint64_t*)k, (uint32_t*)p, um);
  else k_unpack<8, 8><<<grid, 256, 0, h->stream>>>((const Tup<8, 8>*)t, n, (uint64_t*)k, (uint64_t*)p, um);
  CK_LAUNCH(h);
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// small-buffer carve-up for one call
// ---------------------------------------------------------------------------
struct Carve {
  size_t off = 0;
  size_t take(size_t bytes) {
    size_t o = (off + 255) & ~(size_t)255;
    off = o + bytes;
    return o;
  }
};

struct SideLayout {            // per relation
  uint32_t cps1 = 0, cps2 = 0;
  size_t hist1 = 0, rowsum1 = 0, bounds1 = 0, hist2 = 0, rowsum2 = 0, bounds2 = 0;
  // joint path: hist2 holds the claim cursors [Q], rowsum2 the spill counts
  // [Q] (zeroed), part the per-CTA 16-bit joint histograms [nparts][Q]
  size_t part = 0;
  uint32_t nparts = 0;
  size_t lpool = 0;          // linked pass 1: buffers handed out (zeroed)
};

struct CallLayout {
  size_t zero_lo = 0, zero_hi = 0;
  size_t acc = 0, out_ctr = 0, ctrs = 0, items = 0;
  SideLayout side[2];
  size_t total = 0;
  uint32_t n_items_cap = 0;
};

static CallLayout layout_for(const hape_join* h, const hape_plan& pl, uint64_t n_r, uint64_t n_s) {
  CallLayout L;
  Carve cv;
  const uint64_t P1 = 1ull << pl.bits[0], P2 = pl.passes == 2 ? (1ull << pl.bits[1]) : 1ull;
  const uint64_t Q = P1 * P2;
  // zeroed region first: acc[4] u64, out_ctr u64, ctrs (n_items, item_ctr), rowsums
  L.acc = cv.take(4 * 8);
  L.zero_lo = L.acc;
  L.out_ctr = cv.take(8);
  L.ctrs = cv.take(8);
  const uint64_t ns[2] = {n_r, n_s};
  for (int s = 0; s < 2; s++) {
    L.side[s].rowsum1 = cv.take(P1 * 4);   // (linked pass 1: the buckets' claim counters)
    if (pl.passes == 2) L.side[s].rowsum2 = cv.take(Q * 4);
    if (use_linked(h, pl)) L.side[s].lpool = cv.take(8);
  }
  L.zero_hi = cv.off;
  for (int s = 0; s < 2; s++) {
    SideLayout& S = L.side[s];
    S.cps1 = cps_for(h, ns[s], 1);
    S.hist1 = cv.take(P1 * (use_joint(h, pl) || use_claim(h, pl) ? 1 : S.cps1) * 4);  // joint / claim: pass-1 cursors
    S.bounds1 = cv.take((P1 + 1) * 4);
    if (pl.passes == 2 && use_joint(h, pl)) {
      S.cps2 = cps_for(h, ns[s], (uint32_t)P1);
      S.hist2 = cv.take(Q * 4);
      S.bounds2 = cv.take((Q + 1) * 4);
      S.nparts = joint_grid(h, (uint32_t)std::min<uint64_t>(ns[s] / 1024 + 1, 1u << 20));
      S.part = cv.take((size_t)S.nparts * Q * 2);
    } else if (pl.passes == 2) {
      S.cps2 = cps_for(h, ns[s], (uint32_t)P1);
      S.hist2 = cv.take(Q * (use_claim(h, pl) ? 1 : S.cps2) * 4);
      S.bounds2 = cv.take((Q + 1) * 4);
    }
  }
  L.n_items_cap = (uint32_t)std::min<uint64_t>(Q + (n_s + pl.probe_slice - 1) / pl.probe_slice + 1, 0xFFFFFFFFu);
  L.items = cv.take((size_t)L.n_items_cap * 8);
  L.total = cv.off;
  return L;
}

template <class T>
static T* at(hape_join* h, size_t off) {
  return reinterpret_cast<T*>(static_cast<char*>(h->small.p) + off);
}

// Radix passes over one relation: in -> ping (AoS) -> pong (AoS) -> bounds.
// Launches are grouped by stage across both relations.
struct PassIO {
  Src in;       // pass-1 input
  void* p1;     // pass-1 output tuples
  void* p2;     // pass-2 output tuples
};

// side1_ready != nullptr: host-resident inputs whose S copy is still in
// flight on the copy stream -- run all of R's passes first (overlapping the S
// transfer), then wait for the copy and run S's.  Stage marks then cover
// both sides' work in sequence.
static hape_status run_partition_stages(hape_join* h, const hape_plan& pl, const CallLayout& L, PassIO io[2],
                                        int nside, const void** fin, const uint32_t** fin_bounds,
                                        cudaEvent_t side1_ready = nullptr) {
  const int kw = key_width(h->cfg);
  const uint32_t P1 = 1u << pl.bits[0], P2 = 1u << pl.bits[1];
  // DESIGN.md R3: pass 1 takes bits [B2, B2+B1) of h, pass 2 bits [0, B2), so
  // the final co-partition of a key is the low B1+B2 bits of h
  const BitField bf1{pl.passes == 2 ? pl.bits[1] : 0u, P1 - 1}, bf2{0u, P2 - 1};
  SegMap m1[2], m2[2];
  Src s2[2];
  for (int s = 0; s < nside; s++) {
    m1[s] = SegMap{nullptr, 1u, L.side[s].cps1, io[s].in.n};
    if (pl.passes == 2) m2[s] = SegMap{at<uint32_t>(h, L.side[s].bounds1), P1, L.side[s].cps2, io[s].in.n};
    s2[s] = Src{PartIn{nullptr, nullptr, io[s].p1}, true, io[s].in.n, io[s].in.pw};
  }
  // joint path (use_joint): hist1 = k_hist_joint (both passes' buckets),
  // scan1 = k_joint_reduce (bounds + claim cursors of both passes), both
  // scatters claim; hist2 / scan2 are empty.  Workspace reuse: hist1 / hist2
  // hold the pass-1 / pass-2 cursors, rowsum1 the row totals, rowsum2 the
  // spilled counts (both zeroed per call).
  const bool joint = use_joint(h, pl);
  const bool claim = use_claim(h, pl);
  // claim form: totals -> cursors (the scan reads them as a one-CTA histogram)
  auto totals_scan = [&](SegMap m, uint32_t P, size_t cur_off, size_t rs_off, size_t bnd_off) {
    const size_t rows = (size_t)m.nseg * P;
    CK(h, cudaMemcpyAsync(at<uint32_t>(h, cur_off), at<uint32_t>(h, rs_off), rows * 4, cudaMemcpyDeviceToDevice,
                          h->stream));
    return launch_scan(h, SegMap{m.bounds, m.nseg, 1u, m.n}, P, at<uint32_t>(h, cur_off), at<uint32_t>(h, rs_off),
                       at<uint32_t>(h, bnd_off));
  };
  auto hist1 = [&](int s) {
    // the persistent joint-histogram CTAs take one contiguous range each (the
    // claiming scatters do not depend on the histogram's chunking)
    if (joint)
      return launch_hist_joint(h, kw, io[s].in, SegMap{nullptr, 1u, L.side[s].nparts, io[s].in.n}, bf1, bf2, P1, P2,
                               at<uint32_t>(h, L.side[s].rowsum1),
                               at<uint16_t>(h, L.side[s].part), at<uint32_t>(h, L.side[s].rowsum2));
    return launch_hist(h, kw, io[s].in, m1[s], bf1, P1, claim ? nullptr : at<uint32_t>(h, L.side[s].hist1),
                       at<uint32_t>(h, L.side[s].rowsum1));
  };
  auto jr_args = [&](int s) {
    return JrArgs{at<uint16_t>(h, L.side[s].part), L.side[s].nparts, at<uint32_t>(h, L.side[s].rowsum2),
                  at<uint32_t>(h, L.side[s].rowsum1), at<uint32_t>(h, L.side[s].bounds1),
                  at<uint32_t>(h, L.side[s].hist1), at<uint32_t>(h, L.side[s].bounds2),
                  at<uint32_t>(h, L.side[s].hist2)};
  };
  auto scan1 = [&](int s) {
    if (joint) {
      const JrArgs a = jr_args(s);
      return launch_joint_reduce(h, &a, 1, P1, P2);
    }
    if (claim) return totals_scan(m1[s], P1, L.side[s].hist1, L.side[s].rowsum1, L.side[s].bounds1);
    return launch_scan(h, m1[s], P1, at<uint32_t>(h, L.side[s].hist1), at<uint32_t>(h, L.side[s].rowsum1),
                       at<uint32_t>(h, L.side[s].bounds1));
  };
  auto scatter1 = [&](int s) {
    return launch_scatter(h, kw, io[s].in, m1[s], bf1, P1, at<uint32_t>(h, L.side[s].hist1), io[s].p1,
                          joint || claim);
  };
  auto hist2 = [&](int s) {
    if (joint) return HAPE_OK;
    return launch_hist(h, kw, s2[s], m2[s], bf2, P2, claim ? nullptr : at<uint32_t>(h, L.side[s].hist2),
                       at<uint32_t>(h, L.side[s].rowsum2));
  };
  auto scan2 = [&](int s) {
    if (joint) return HAPE_OK;
    if (claim) return totals_scan(m2[s], P2, L.side[s].hist2, L.side[s].rowsum2, L.side[s].bounds2);
    return launch_scan(h, m2[s], P2, at<uint32_t>(h, L.side[s].hist2), at<uint32_t>(h, L.side[s].rowsum2),
                       at<uint32_t>(h, L.side[s].bounds2));
  };
  auto scatter2 = [&](int s) {
    return launch_scatter(h, kw, s2[s], m2[s], bf2, P2, at<uint32_t>(h, L.side[s].hist2), io[s].p2,
                          joint || claim);
  };
  if (use_linked(h, pl)) {
    // the single-scan form (P593-597): pass 1 claims into buffer chains with
    // no histogram before it; pass 2 reads the chains, counts its buckets
    // (totals), and claims into the dense pass-2 layout.  Stage marks:
    // hist1 = directory reset, scatter1 = linked scatter + pass-1 bounds.
    LinkMap lk[2];
    SegMap mb[2];
    for (int s = 0; s < nside; s++) {
      const uint64_t n = io[s].in.n;
      const size_t tb = tup_bytes(kw, io[s].in.pw);
      const uint32_t B = lb_buf(tb);
      const uint64_t nb = lb_nbuf(n, tb, P1), km = lb_kmax(n, tb);
      if (h->lbuf[s].bytes < lb_ws_bytes(n, tb, P1))
        return fail(h, HAPE_ERR_INVALID_ARG, "linked-buffer workspace not allocated before the passes");
      uint32_t* dir = static_cast<uint32_t*>(h->lbuf[s].p);
      uint32_t* owner = dir + (size_t)P1 * km;
      uint32_t* kidx = owner + nb;
      lk[s] = LinkMap{at<uint32_t>(h, L.side[s].rowsum1), at<uint32_t>(h, L.side[s].lpool), dir, owner, kidx,
                      (uint32_t)km, B};
      mb[s] = SegMap{nullptr, (uint32_t)nb, 1u, (uint32_t)n, owner, kidx, lk[s].cnt, lk[s].pool, B};
      s2[s] = Src{PartIn{nullptr, nullptr, io[s].p1}, true, (uint32_t)n, io[s].in.pw};
    }
    for (int s = 0; s < nside; s++) {
      if (s == 1 && side1_ready) CK(h, cudaStreamWaitEvent(h->stream, side1_ready, 0));
      if (s == 0) mark(h, HAPE_STAGE_HIST1);
      CK(h, cudaMemsetAsync(lk[s].dir, 0, (size_t)P1 * lk[s].kmax * 4, h->stream));
      if (s == 0) mark(h, HAPE_STAGE_SCATTER1);
      CKS(launch_scatter_linked(h, kw, io[s].in, m1[s], bf1, P1, io[s].p1, lk[s]));
      CKS(totals_scan(m1[s], P1, L.side[s].hist1, L.side[s].rowsum1, L.side[s].bounds1));
    }
    mark(h, HAPE_STAGE_HIST2);
    for (int s = 0; s < nside; s++)
      CKS(launch_hist(h, kw, s2[s], mb[s], bf2, P2, nullptr, at<uint32_t>(h, L.side[s].rowsum2)));
    mark(h, HAPE_STAGE_SCAN2);
    for (int s = 0; s < nside; s++) CKS(scan2(s));
    mark(h, HAPE_STAGE_SCATTER2);
    for (int s = 0; s < nside; s++)
      CKS(launch_scatter(h, kw, s2[s], mb[s], bf2, P2, at<uint32_t>(h, L.side[s].hist2), io[s].p2, true));
  } else if (side1_ready) {
    for (int s = 0; s < nside; s++) {
      if (s == 1) CK(h, cudaStreamWaitEvent(h->stream, side1_ready, 0));
      if (s == 0) mark(h, HAPE_STAGE_HIST1);
      CKS(hist1(s)); CKS(scan1(s)); CKS(scatter1(s));
      if (pl.passes == 2) { CKS(hist2(s)); CKS(scan2(s)); CKS(scatter2(s)); }
    }
  } else {
    mark(h, HAPE_STAGE_HIST1);
    for (int s = 0; s < nside; s++) CKS(hist1(s));
    mark(h, HAPE_STAGE_SCAN1);
    if (joint && nside == 2) {
      const JrArgs a[2] = {jr_args(0), jr_args(1)};
      CKS(launch_joint_reduce(h, a, 2, P1, P2));
    } else {
      for (int s = 0; s < nside; s++) CKS(scan1(s));
    }
    mark(h, HAPE_STAGE_SCATTER1);
    for (int s = 0; s < nside; s++) CKS(scatter1(s));
    if (pl.passes == 2) {
      mark(h, HAPE_STAGE_HIST2);
      for (int s = 0; s < nside; s++) CKS(hist2(s));
      mark(h, HAPE_STAGE_SCAN2);
      for (int s = 0; s < nside; s++) CKS(scan2(s));
      mark(h, HAPE_STAGE_SCATTER2);
      for (int s = 0; s < nside; s++) CKS(scatter2(s));
    }
  }
  for (int s = 0; s < nside; s++) {
    fin[s] = pl.passes == 2 ? io[s].p2 : io[s].p1;
    fin_bounds[s] = at<uint32_t>(h, pl.passes == 2 ? L.side[s].bounds2 : L.side[s].bounds1);
  }
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// argument checks
// ---------------------------------------------------------------------------
static hape_status check_rel(hape_join* h, const hape_relation* r, int kw, int pw, const char* name) {
  if (!r) return fail(h, HAPE_ERR_INVALID_ARG, "%s is NULL", name);
  if (r->n >= 0xFFFFFFFFull) return fail(h, HAPE_ERR_UNSUPPORTED, "%s.n >= 2^32 per rank", name);
  if (r->mem != HAPE_MEM_DEVICE && r->mem != HAPE_MEM_HOST)
    return fail(h, HAPE_ERR_INVALID_ARG, "%s.mem invalid", name);
  if (r->n && (!r->key || !r->payload)) return fail(h, HAPE_ERR_INVALID_ARG, "%s has NULL column with n>0", name);
  if (((uintptr_t)r->key % kw) || ((uintptr_t)r->payload % pw))
    return fail(h, HAPE_ERR_INVALID_ARG, "%s column not element-aligned", name);
  return HAPE_OK;
}

static hape_status stage_in(hape_join* h, const hape_relation* r, int kw, int pw, DevBuf& bk, DevBuf& bp,
                            Src* out, cudaStream_t st = nullptr) {
  if (!st) st = h->stream;
  out->n = (uint32_t)r->n;
  out->pw = pw;
  out->aos = false;
  if (r->mem == HAPE_MEM_DEVICE || r->n == 0) {
    out->in = PartIn{r->key, r->payload, nullptr};
    return HAPE_OK;
  }
  CKS(ensure(h, bk, r->n * kw));
  CKS(ensure(h, bp, r->n * pw));
  CK(h, cudaMemcpyAsync(bk.p, r->key, r->n * kw, cudaMemcpyHostToDevice, st));
  CK(h, cudaMemcpyAsync(bp.p, r->payload, r->n * pw, cudaMemcpyHostToDevice, st));
  out->in = PartIn{bk.p, bp.p, nullptr};
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// G>1: device partition by destination + NCCL exchange (a2-a5)
// ---------------------------------------------------------------------------
extern "C" hape_status hape_exchange_plan(int world_size, int rank, const uint64_t* counts, uint64_t* send_off,
                                          uint64_t* recv_off, uint64_t* recv_total) {
  if (world_size < 1 || rank < 0 || rank >= world_size || !counts || !send_off || !recv_off || !recv_total)
    return HAPE_ERR_INVALID_ARG;
  const int G = world_size;
  uint64_t s = 0;
  for (int d = 0; d < G; d++) { send_off[d] = s; s += counts[(size_t)rank * G + d]; }
  uint64_t r = 0;
  for (int src = 0; src < G; src++) { recv_off[src] = r; r += counts[(size_t)src * G + rank]; }
  *recv_total = r;
  return HAPE_OK;
}

// a2-a4: device partition of one relation by destination = the top log2(G)
// bits of h (R14) -- hist -> scan -> smem-staged scatter with
// fan-out G -- into `out` (AoS tuples, destination-major) and bounds[G+1]
// (device, tuple offsets relative to `out`).  The router of P643-652 ("hash-
// based" policy) as one partitioning pass.
static hape_status route(hape_join* h, const Src& in, uint32_t G, void* out, uint32_t* bounds) {
  const int kw = key_width(h->cfg);
  const uint32_t g = ceil_log2_u64((uint64_t)G);
  const uint32_t HW = kw * 8;
  const BitField bf{g ? HW - g : 0u, G - 1};
  const uint32_t cps = cps_for(h, in.n, 1);
  const size_t hist_b = ((size_t)G * cps * 4 + 255) & ~(size_t)255;
  CKS(ensure(h, h->route_ws, hist_b + (size_t)G * 4));
  uint32_t* hist = static_cast<uint32_t*>(h->route_ws.p);
  uint32_t* rs = hist + hist_b / 4;
  CK(h, cudaMemsetAsync(rs, 0, (size_t)G * 4, h->stream));
  const SegMap m{nullptr, 1u, cps, in.n};
  CKS(launch_hist(h, kw, in, m, bf, G, hist, rs));
  CKS(launch_scan(h, m, G, hist, rs, bounds));
  CKS(launch_scatter(h, kw, in, m, bf, G, hist, out));
  return HAPE_OK;
}

static hape_status exchange(hape_join* h, Src in[2], Src out[2]) {
  const int G = std::max(1, h->cfg.world_size), me = h->cfg.rank;
  const int kw = key_width(h->cfg);
  // bounds: local [2][G+1], then gathered [G][2][G+1]
  const size_t nl = (size_t)2 * (G + 1), nb = (size_t)G * nl;
  CKS(ensure(h, h->xb, (nl + nb) * 4));
  uint32_t* bl = static_cast<uint32_t*>(h->xb.p);
  uint32_t* bg = bl + nl;
  mark(h, HAPE_STAGE_DEVPART);
  size_t tb[2];
  for (int s = 0; s < 2; s++) {
    tb[s] = tup_bytes(kw, in[s].pw);
    CKS(ensure(h, h->send[s], (size_t)in[s].n * tb[s] + 16));
    CKS(route(h, in[s], (uint32_t)G, h->send[s].p, bl + s * (G + 1)));
  }
  mark(h, HAPE_STAGE_EXCHANGE);
  // count exchange: all-gather every rank's destination bounds
  CKN(h, ncclAllGather(bl, bg, nl, ncclUint32, h->comm, h->stream));
  if (h->h_bounds_cap < nb) {
    if (h->h_bounds) cudaFreeHost(h->h_bounds);
    h->h_bounds = nullptr;
    h->h_bounds_cap = 0;
    CK(h, cudaMallocHost(&h->h_bounds, nb * 4));
    h->h_bounds_cap = nb;
  }
  CK(h, cudaMemcpyAsync(h->h_bounds, bg, nb * 4, cudaMemcpyDeviceToHost, h->stream));
  CK(h, cudaStreamSynchronize(h->stream));
  for (int s = 0; s < 2; s++) {
    std::vector<uint64_t> counts((size_t)G * G), soff(G), roff(G);
    for (int src = 0; src < G; src++) {
      const uint32_t* b = h->h_bounds + (size_t)src * nl + s * (G + 1);
      for (int d = 0; d < G; d++) counts[(size_t)src * G + d] = b[d + 1] - b[d];
    }
    uint64_t rtot = 0;
    hape_exchange_plan(G, me, counts.data(), soff.data(), roff.data(), &rtot);
    if (rtot >= 0xFFFFFFFFull) return fail(h, HAPE_ERR_UNSUPPORTED, "received %llu tuples >= 2^32", (unsigned long long)rtot);
    CKS(ensure(h, h->recv[s], rtot * tb[s] + 16));
    const char* sb = static_cast<const char*>(h->send[s].p);
    char* rb = static_cast<char*>(h->recv[s].p);
    CKN(h, ncclGroupStart());
    for (int p = 0; p < G; p++) {
      const uint64_t sc = counts[(size_t)me * G + p], rc = counts[(size_t)p * G + me];
      if (sc) CKN(h, ncclSend(sb + soff[p] * tb[s], sc * tb[s], ncclUint8, p, h->comm, h->stream));
      if (rc) CKN(h, ncclRecv(rb + roff[p] * tb[s], rc * tb[s], ncclUint8, p, h->comm, h->stream));
    }
    CKN(h, ncclGroupEnd());
    out[s] = Src{PartIn{nullptr, nullptr, h->recv[s].p}, true, (uint32_t)rtot, in[s].pw};
  }
  h->xchg_path = 1;
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// G>1, fused form: the destination partition's scatter
// writes its claimed runs straight into the destination ranks' receive
// buffers over NVLink (peer pointers from CUDA IPC handles exchanged once per
// buffer growth), so the exchange costs no send buffer, no second read and
// no separate transfer: the NVLink traffic overlaps the partitioning tile by
// tile.  The router + mem-move of P643-656 as ONE kernel.
// ---------------------------------------------------------------------------
extern "C" hape_status hape_peer_plan(int world_size, int rank, const uint64_t* counts, uint64_t* write_off,
                                      uint64_t* recv_total, uint64_t* recv_capacity) {
  if (world_size < 1 || rank < 0 || rank >= world_size || !counts || !write_off || !recv_total || !recv_capacity)
    return HAPE_ERR_INVALID_ARG;
  const int G = world_size;
  uint64_t mx = 0;
  for (int d = 0; d < G; d++) {
    uint64_t t = 0, base = 0;
    for (int src = 0; src < G; src++) {
      const uint64_t x = counts[(size_t)src * G + d];
      if (src < rank) base += x;
      t += x;
    }
    write_off[d] = base;
    if (d == rank) *recv_total = t;
    mx = std::max(mx, t);
  }
  *recv_capacity = mx;
  return HAPE_OK;
}

static BitField dest_field(const hape_join* h, uint32_t G) {
  const uint32_t g = ceil_log2_u64((uint64_t)G);
  const uint32_t HW = key_width(h->cfg) * 8;
  return BitField{g ? HW - g : 0u, G - 1};  // destination = top g bits of h (R14)
}

// per-destination totals of one relation (totals-only histogram, += into
// `totals`, which the caller zeroes)
static hape_status route_totals(hape_join* h, const Src& in, uint32_t G, uint32_t* totals) {
  const SegMap m{nullptr, 1u, cps_for(h, in.n, 1), in.n};
  return launch_hist(h, key_width(h->cfg), in, m, dest_field(h, G), G, nullptr, totals);
}

static hape_status route_peer(hape_join* h, const Src& in, uint32_t G, uint32_t* cursors, void* const* peers) {
  const SegMap m{nullptr, 1u, cps_for(h, in.n, 1), in.n};
  return launch_peer_scatter(h, key_width(h->cfg), in, m, dest_field(h, G), G, cursors, peers);
}

static void close_peers(hape_join* h, int s) {
  for (auto& p : h->peer_rx[s])
    if (p) {
      cudaIpcCloseMemHandle(p);
      p = nullptr;
    }
}

// returns HAPE_ERR_UNSUPPORTED (on every rank alike) when some rank could not
// map its peers' buffers; the caller then runs the NCCL send/recv exchange
static hape_status exchange_p2p(hape_join* h, Src in[2], Src out[2]) {
  const int G = std::max(1, h->cfg.world_size), me = h->cfg.rank;
  const int kw = key_width(h->cfg);
  const size_t nl = (size_t)2 * G, nb = (size_t)G * nl;
  // xb: totals [2][G] | gathered [G][2][G] | cursors [2][G] | flag / barrier words
  CKS(ensure(h, h->xb, (nl + nb + nl + 8) * 4));
  uint32_t* tot = static_cast<uint32_t*>(h->xb.p);
  uint32_t* gat = tot + nl;
  uint32_t* cur = gat + nb;
  uint32_t* word = cur + nl;
  CK(h, cudaMemsetAsync(tot, 0, nl * 4, h->stream));
  mark(h, HAPE_STAGE_DEVPART);
  for (int s = 0; s < 2; s++) CKS(route_totals(h, in[s], (uint32_t)G, tot + s * G));
  // count exchange -- also the start barrier: a rank's all-gather runs after
  // its previous local join (stream order), and no rank scatters into a peer
  // before every rank has joined the all-gather
  CKN(h, ncclAllGather(tot, gat, nl, ncclUint32, h->comm, h->stream));
  if (h->h_bounds_cap < nb) {
    if (h->h_bounds) cudaFreeHost(h->h_bounds);
    h->h_bounds = nullptr;
    h->h_bounds_cap = 0;
    CK(h, cudaMallocHost(&h->h_bounds, nb * 4));
    h->h_bounds_cap = nb;
  }
  CK(h, cudaMemcpyAsync(h->h_bounds, gat, nb * 4, cudaMemcpyDeviceToHost, h->stream));
  CK(h, cudaStreamSynchronize(h->stream));
  const uint32_t* c = h->h_bounds;  // c[src*nl + s*G + d]
  size_t tb[2];
  uint64_t rtot[2], need[2];
  for (int s = 0; s < 2; s++) {
    tb[s] = tup_bytes(kw, in[s].pw);
    std::vector<uint64_t> counts((size_t)G * G), off(G);
    for (int src = 0; src < G; src++)
      for (int d = 0; d < G; d++) counts[(size_t)src * G + d] = c[(size_t)src * nl + s * G + d];
    uint64_t mx = 0;
    hape_peer_plan(G, me, counts.data(), off.data(), &rtot[s], &mx);
    for (int d = 0; d < G; d++) h->h_x[s * G + d] = (uint32_t)off[d];
    if (mx >= 0xFFFFFFFFull) return fail(h, HAPE_ERR_UNSUPPORTED, "a rank receives %llu tuples >= 2^32", (unsigned long long)mx);
    need[s] = mx * tb[s] + 16;  // the same on every rank: buffers grow together
  }
  bool remap = !h->peer_tab.p || h->peer_tab_dirty;
  h->peer_tab_dirty = false;
  for (int s = 0; s < 2; s++) {
    if (need[s] <= h->prx[s].bytes) continue;
    close_peers(h, s);
    CKS(ensure(h, h->prx[s], need[s] + need[s] / 8));
    remap = true;
  }
  if (remap) {
    void* tab[2][64] = {};
    int bad = 0;
    if (G > 1) {
      // all-gather the receive buffers' IPC handles, map the peers'
      cudaIpcMemHandle_t mine[2];
      for (int s = 0; s < 2; s++) CK(h, cudaIpcGetMemHandle(&mine[s], h->prx[s].p));
      const size_t hb = sizeof mine;
      CKS(ensure(h, h->xipc, hb * (G + 1)));
      std::vector<unsigned char> all(hb * G);
      CK(h, cudaMemcpyAsync(h->xipc.p, mine, hb, cudaMemcpyHostToDevice, h->stream));
      CKN(h, ncclAllGather(h->xipc.p, static_cast<char*>(h->xipc.p) + hb, hb, ncclUint8, h->comm, h->stream));
      CK(h, cudaMemcpyAsync(all.data(), static_cast<char*>(h->xipc.p) + hb, hb * G, cudaMemcpyDeviceToHost, h->stream));
      CK(h, cudaStreamSynchronize(h->stream));
      for (int p = 0; p < G && !bad; p++) {
        if (p == me) continue;
        for (int s = 0; s < 2 && !bad; s++) {
          cudaIpcMemHandle_t hd;
          memcpy(&hd, all.data() + hb * p + sizeof(cudaIpcMemHandle_t) * s, sizeof hd);
          if (h->peer_rx[s][p]) cudaIpcCloseMemHandle(h->peer_rx[s][p]);
          h->peer_rx[s][p] = nullptr;
          if (cudaIpcOpenMemHandle(&h->peer_rx[s][p], hd, cudaIpcMemLazyEnablePeerAccess) != cudaSuccess) {
            (void)cudaGetLastError();
            h->peer_rx[s][p] = nullptr;
            bad = 1;
          }
        }
      }
      // every rank takes the same path: max of the failure flags
      CK(h, cudaMemcpyAsync(word, &bad, 4, cudaMemcpyHostToDevice, h->stream));
      CKN(h, ncclAllReduce(word, word, 1, ncclInt32, ncclMax, h->comm, h->stream));
      CK(h, cudaMemcpyAsync(&bad, word, 4, cudaMemcpyDeviceToHost, h->stream));
      CK(h, cudaStreamSynchronize(h->stream));
      if (bad) {
        for (int s = 0; s < 2; s++) close_peers(h, s);
        h->p2p_failed = true;
        return fail(h, HAPE_ERR_UNSUPPORTED, "peer mapping of the receive buffers failed on some rank");
      }
    }
    for (int s = 0; s < 2; s++)
      for (int d = 0; d < G; d++) tab[s][d] = d == me ? h->prx[s].p : h->peer_rx[s][d];
    CKS(ensure(h, h->peer_tab, nl * sizeof(void*)));
    std::vector<void*> flat(nl);
    for (int s = 0; s < 2; s++)
      for (int d = 0; d < G; d++) flat[s * G + d] = tab[s][d];
    CK(h, cudaMemcpyAsync(h->peer_tab.p, flat.data(), nl * sizeof(void*), cudaMemcpyHostToDevice, h->stream));
    CK(h, cudaStreamSynchronize(h->stream));
  }
  // this rank's segment start inside every destination's buffer
  CK(h, cudaMemcpyAsync(cur, h->h_x, nl * 4, cudaMemcpyHostToDevice, h->stream));
  mark(h, HAPE_STAGE_EXCHANGE);
  void* const* ptab = static_cast<void* const*>(h->peer_tab.p);
  for (int s = 0; s < 2; s++) CKS(route_peer(h, in[s], (uint32_t)G, cur + s * G, ptab + s * G));
  // completion barrier: each rank's scatter (ending in a system-scope fence)
  // precedes its contribution, so afterwards every receive buffer is complete
  CKN(h, ncclAllReduce(word + 1, word + 1, 1, ncclUint32, ncclSum, h->comm, h->stream));
  for (int s = 0; s < 2; s++) out[s] = Src{PartIn{nullptr, nullptr, h->prx[s].p}, true, (uint32_t)rtot[s], in[s].pw};
  h->xchg_path = 2;
  return HAPE_OK;
}

// stage times after the final event: each used stage runs until the next
// used stage mark (stages are marked in enum order on the join stream)
static void stage_times(hape_join* h, hape_join_result* res) {
  static const bool off = getenv("HAPE_NO_STAGE_TIMES") != nullptr;  // (host-overhead A/B only)
  if (off) return;
  int order[HAPE_NSTAGES];
  int no = 0;
  for (int s = HAPE_STAGE_H2D; s < HAPE_STAGE_TOTAL; s++)
    if (h->ev_used[s]) order[no++] = s;
  for (int i = 0; i < no; i++) {
    cudaEvent_t end = i + 1 < no ? h->ev[order[i + 1]] : h->ev[HAPE_NSTAGES];
    float ms = 0;
    cudaEventElapsedTime(&ms, h->ev[order[i]], end);
    res->stage_ms[order[i]] = ms;
  }
  float tot = 0;
  cudaEventElapsedTime(&tot, h->ev[HAPE_STAGE_TOTAL], h->ev[HAPE_NSTAGES]);
  res->stage_ms[HAPE_STAGE_TOTAL] = tot;
  (void)cudaGetLastError();
}


// allocations of the passes that must precede enqueueing (CUDA-graph capture)
static hape_status ensure_pass_ws(hape_join* h, const hape_plan& pl, const uint64_t* n, const int* pw, int nside) {
  if (!use_linked(h, pl)) return HAPE_OK;
  const int kw = key_width(h->cfg);
  for (int s = 0; s < nside; s++) CKS(ensure(h, h->lbuf[s], lb_ws_bytes(n[s], tup_bytes(kw, pw[s]), 1u << pl.bits[0])));
  return HAPE_OK;
}

// pass-1 output bytes: the relation, or (linked pass 1) its buffer pool
static size_t ping_bytes(const hape_join* h, const hape_plan& pl, uint64_t n, size_t tb) {
  if (use_linked(h, pl)) return (size_t)lb_nbuf(n, tb, 1u << pl.bits[0]) * lb_buf(tb) * tb + 16;
  return (size_t)n * tb + 16;
}

// ---------------------------------------------------------------------------
// the local join (a6-a13 over one GPU's share): plan, radix passes, work
// list, build+probe, local result D2H into h_res[0..5] (acc[4], out_ctr,
// ctrs).  Enqueued on h->stream; no host sync.  When every pointer and size
// matches the previous call the sequence is replayed as one captured CUDA
// graph (launch-latency bound small joins, BASELINE configs[0]).
// ---------------------------------------------------------------------------
struct MatOut {
  bool on = false;
  void* r = nullptr;
  void* s = nullptr;
  uint64_t cap = 0;
};

static hape_status local_join(hape_join* h, const Src loc_in[2], const MatOut& mo, cudaEvent_t side1_ready,
                              bool graphable, hape_plan* pl_out) {
  const hape_join_config& c = h->cfg;
  const int kw = key_width(c), prw = pay_width(c.r_payload_type), psw = pay_width(c.s_payload_type);
  const Src loc[2] = {loc_in[0], loc_in[1]};
  hape_plan pl;
  if (make_plan(h, loc[0].n, loc[1].n, &pl) != HAPE_OK)
    return fail(h, HAPE_ERR_INVALID_ARG, "invalid radix plan (bits/passes)");
  const CallLayout L = layout_for(h, pl, loc[0].n, loc[1].n);
  CKS(ensure(h, h->small, L.total));
  const uint64_t n_loc[2] = {loc[0].n, loc[1].n};
  const int pw[2] = {prw, psw};
  for (int s = 0; s < 2; s++) {
    CKS(ensure(h, h->ping[s], ping_bytes(h, pl, n_loc[s], tup_bytes(kw, pw[s]))));
    if (pl.passes == 2) CKS(ensure(h, h->pong[s], n_loc[s] * tup_bytes(kw, pw[s]) + 16));
  }
  CKS(ensure_pass_ws(h, pl, n_loc, pw, 2));
  const uint32_t Q = 1u << (pl.bits[0] + (pl.passes == 2 ? pl.bits[1] : 0));
  uint32_t* ctrs = at<uint32_t>(h, L.ctrs);  // [0] n_items
  auto enqueue = [&]() -> hape_status {
    CK(h, cudaMemsetAsync(at<char>(h, L.zero_lo), 0, L.zero_hi - L.zero_lo, h->stream));
    PassIO io[2];
    for (int s = 0; s < 2; s++) io[s] = PassIO{loc[s], h->ping[s].p, h->pong[s].p};
    const void* ft[2];
    const uint32_t* fb[2];
    CKS(run_partition_stages(h, pl, L, io, 2, ft, fb, side1_ready));
    mark(h, HAPE_STAGE_WORKLIST);
    k_worklist<<<(Q + WL_THREADS - 1) / WL_THREADS, WL_THREADS, 0, h->stream>>>(fb[0], fb[1], Q, pl.probe_slice,
                                                                                at<uint2>(h, L.items), ctrs);
    CK_LAUNCH(h);
    mark(h, HAPE_STAGE_BUILD_PROBE);
    JoinArgs ja{};
    ja.rt = ft[0]; ja.st = ft[1];
    ja.bR = fb[0]; ja.bS = fb[1];
    ja.items = at<uint2>(h, L.items); ja.n_items = ctrs;
    ja.cap = pl.build_cap; ja.slice = pl.probe_slice; ja.slot_bits = pl.slot_bits;
    ja.qmask = Q - 1;
    // (HAPE_JN_EPOCH_PERIOD: test-only, forces frequent head resets)
    static const int ep_env = env_int("HAPE_JN_EPOCH_PERIOD", 65535);
    ja.ep_period = (uint32_t)std::max(1, std::min(65535, ep_env));
    ja.acc = at<unsigned long long>(h, L.acc);
    ja.out_r = mo.r; ja.out_s = mo.s; ja.out_cap = mo.on ? mo.cap : 0;
    ja.out_ctr = at<unsigned long long>(h, L.out_ctr);
    static const uint32_t jn_dbg = [] { const char* e = getenv("HAPE_JN_DBG"); return e ? (uint32_t)atoi(e) : 0u; }();
    ja.dbg = jn_dbg;  // timing experiments only: results are wrong when set
    ja.r_unique = (c.flags & HAPE_FLAG_R_UNIQUE) ? 1u : 0u;
    // L2 warm-up window per stage: the head of each S slice (a whole C2 slice;
    // larger slices would thrash L2 a stage ahead of their use)
    static const int pf_env = [] { const char* e = getenv("HAPE_JN_PF"); return e ? atoi(e) : -1; }();
    ja.pf_bytes = pf_env >= 0 ? (uint32_t)pf_env : 32768u;
    ja.probe_heavy = n_loc[1] >= 2 * n_loc[0] ? 1u : 0u;
    CKS(launch_join(h, kw, prw, psw, ja, mo.on, &pl.join_ctas));
    mark(h, HAPE_STAGE_FINALIZE);
    // local result: acc[4], out_ctr, ctrs
    CK(h, cudaMemcpyAsync(h->h_res, at<char>(h, L.acc), 4 * 8, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaMemcpyAsync(h->h_res + 4, at<char>(h, L.out_ctr), 8, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaMemcpyAsync(h->h_res + 5, at<char>(h, L.ctrs), 8, cudaMemcpyDeviceToHost, h->stream));
    return HAPE_OK;
  };
  static const bool no_graph = getenv("HAPE_NO_GRAPH") != nullptr;
  if (graphable && !no_graph && !side1_ready) {
    const uintptr_t key[] = {(uintptr_t)loc[0].in.k, (uintptr_t)loc[0].in.p, (uintptr_t)loc[0].in.t,
                             (uintptr_t)loc[0].n,    (uintptr_t)loc[1].in.k, (uintptr_t)loc[1].in.p,
                             (uintptr_t)loc[1].in.t, (uintptr_t)loc[1].n,    (uintptr_t)mo.r,
                             (uintptr_t)mo.s,        (uintptr_t)(mo.on ? mo.cap : 0), (uintptr_t)h->small.p,
                             (uintptr_t)h->ping[0].p, (uintptr_t)h->ping[1].p, (uintptr_t)h->pong[0].p,
                             (uintptr_t)h->pong[1].p, (uintptr_t)h->lbuf[0].p, (uintptr_t)h->lbuf[1].p};
    static_assert(sizeof key == sizeof h->gkey, "graph key size");
    if (!h->gexec || memcmp(key, h->gkey, sizeof key) != 0) {
      if (h->gexec) { cudaGraphExecDestroy(h->gexec); h->gexec = nullptr; }
      cudaGraph_t g = nullptr;
      CK(h, cudaStreamBeginCapture(h->stream, cudaStreamCaptureModeThreadLocal));
      const hape_status st = enqueue();
      const cudaError_t ce = cudaStreamEndCapture(h->stream, &g);
      if (st != HAPE_OK) { if (g) cudaGraphDestroy(g); return st; }
      CK(h, ce);
      const cudaError_t ie = cudaGraphInstantiate(&h->gexec, g, 0);
      cudaGraphDestroy(g);
      CK(h, ie);
      memcpy(h->gkey, key, sizeof key);
      h->g_launches = h->launches;
      memcpy(h->g_ev_used, h->ev_used, sizeof h->g_ev_used);
      h->g_join_ctas = pl.join_ctas;
    }
    CK(h, cudaGraphLaunch(h->gexec, h->stream));
    h->launches = h->g_launches;
    for (int i = HAPE_STAGE_HIST1; i < HAPE_STAGE_TOTAL; i++) h->ev_used[i] = h->g_ev_used[i];
    pl.join_ctas = h->g_join_ctas;
  } else {
    CKS(enqueue());
  }
  *pl_out = pl;
  return HAPE_OK;
}

static hape_status check_out(hape_join* h, const hape_output* out) {
  if (!out || out->capacity == 0) return HAPE_OK;
  if (!out->r_payload || !out->s_payload) return fail(h, HAPE_ERR_INVALID_ARG, "output buffers NULL");
  if (out->mem != HAPE_MEM_DEVICE && out->mem != HAPE_MEM_HOST) return fail(h, HAPE_ERR_INVALID_ARG, "out.mem");
  return HAPE_OK;
}

// device targets of the pair output: the caller's buffers, or handle-owned
// staging for host-resident outputs (copied back after the join)
static hape_status mat_targets(hape_join* h, const hape_output* out, MatOut* mo) {
  *mo = MatOut{};
  if (!out || out->capacity == 0) return HAPE_OK;
  mo->on = true;
  mo->cap = out->capacity;
  mo->r = out->r_payload;
  mo->s = out->s_payload;
  if (out->mem == HAPE_MEM_HOST) {
    CKS(ensure(h, h->outst[0], out->capacity * pay_width(h->cfg.r_payload_type)));
    CKS(ensure(h, h->outst[1], out->capacity * pay_width(h->cfg.s_payload_type)));
    mo->r = h->outst[0].p;
    mo->s = h->outst[1].p;
  }
  return HAPE_OK;
}

static void fill_plan_fields(hape_join_result* res, const hape_plan& pl, uint64_t nr, uint64_t ns) {
  res->r_local = nr;
  res->s_local = ns;
  res->passes = pl.passes;
  res->bits[0] = pl.bits[0];
  res->bits[1] = pl.passes == 2 ? pl.bits[1] : 0;
  res->n_partitions = 1u << (pl.bits[0] + (pl.passes == 2 ? pl.bits[1] : 0));
}

// ---------------------------------------------------------------------------
// the join
// ---------------------------------------------------------------------------
static hape_status join_impl(hape_join* h, const hape_relation* R, const hape_relation* S, const hape_output* out,
                             hape_join_result* res) {
  const hape_join_config& c = h->cfg;
  const int kw = key_width(c), prw = pay_width(c.r_payload_type), psw = pay_width(c.s_payload_type);
  CKS(check_rel(h, R, kw, prw, "R"));
  CKS(check_rel(h, S, kw, psw, "S"));
  CKS(check_out(h, out));
  const bool mat = out && out->capacity > 0;
  CK(h, cudaSetDevice(h->dev));
  memset(res, 0, sizeof *res);
  for (int i = 0; i < HAPE_NSTAGES; i++) h->ev_used[i] = false;
  h->launches = 0;
  const int world = c.world_size > 1 ? c.world_size : 1;

  mark(h, HAPE_STAGE_TOTAL);
  mark(h, HAPE_STAGE_H2D);
  Src in[2];
  // host-resident S (single GPU): copy it on the copy stream, overlapping the
  // R copy's successors (R's radix passes run while S is in flight)
  const bool overlap = world == 1 && !h->comm && S->mem == HAPE_MEM_HOST && S->n > 0;
  CKS(stage_in(h, R, kw, prw, h->stage[0], h->stage[1], &in[0]));
  if (overlap) {
    CK(h, cudaEventRecord(h->ev_copy, h->stream));          // S staging buffers are free
    CK(h, cudaStreamWaitEvent(h->copy_stream, h->ev_copy, 0));
    CKS(stage_in(h, S, kw, psw, h->stage[2], h->stage[3], &in[1], h->copy_stream));
    CK(h, cudaEventRecord(h->ev_copy, h->copy_stream));
  } else {
    CKS(stage_in(h, S, kw, psw, h->stage[2], h->stage[3], &in[1]));
  }
  Src loc[2] = {in[0], in[1]};
  h->xchg_path = 0;
  if (world > 1 || h->comm) {
    // fused peer-scatter exchange unless disabled (HAPE_XCHG=nccl) or the
    // peers' buffers could not be mapped (then NCCL send/recv, every rank)
    static const bool nccl_only = [] { const char* e = getenv("HAPE_XCHG"); return e && !strcmp(e, "nccl"); }();
    hape_status xs = HAPE_ERR_UNSUPPORTED;
    if (!nccl_only && !h->p2p_failed) {
      xs = exchange_p2p(h, in, loc);
      if (xs != HAPE_OK && xs != HAPE_ERR_UNSUPPORTED) return xs;
    }
    if (xs != HAPE_OK) CKS(exchange(h, in, loc));
  }

  MatOut mo;
  CKS(mat_targets(h, out, &mo));
  const bool graphable = !h->in_coprocess && world == 1 && !h->comm && R->mem == HAPE_MEM_DEVICE &&
                         S->mem == HAPE_MEM_DEVICE && (!mat || out->mem == HAPE_MEM_DEVICE);
  hape_plan pl;
  CKS(local_join(h, loc, mo, overlap ? h->ev_copy : nullptr, graphable, &pl));
  if (world > 1 || h->comm) {
    // global result: NCCL allreduce (sum, u64, wrapping) of the four fields
    // (layout_for puts acc[4] first in the small buffer)
    unsigned long long* acc = at<unsigned long long>(h, 0);
    CKN(h, ncclAllReduce(acc, acc, 4, ncclUint64, ncclSum, h->comm, h->stream));
    CK(h, cudaMemcpyAsync(h->h_res + 6, acc, 4 * 8, cudaMemcpyDeviceToHost, h->stream));
  }
  // without host-resident pairs to copy back, the end-of-call event goes in
  // now and one synchronisation serves both the result and the stage times
  const bool host_pairs = mat && out->mem == HAPE_MEM_HOST;
  if (!host_pairs) cudaEventRecord(h->ev[HAPE_NSTAGES], h->stream);
  CK(h, cudaStreamSynchronize(h->stream));
  const unsigned long long* r = h->h_res;
  res->local_match_count = r[0];
  res->local_sum_r = r[1];
  res->local_sum_s = r[2];
  res->local_pair_checksum = r[3];
  const unsigned long long* g = (world > 1 || h->comm) ? r + 6 : r;
  res->match_count = g[0];
  res->sum_r_payload = g[1];
  res->sum_s_payload = g[2];
  res->pair_checksum = g[3];
  res->n_required = r[0];
  res->n_written = mat ? std::min<uint64_t>(r[4], out->capacity) : 0;
  res->n_items = (uint32_t)(r[5] & 0xFFFFFFFFu);
  fill_plan_fields(res, pl, loc[0].n, loc[1].n);
  res->exchange_path = h->xchg_path;
  if (host_pairs) {
    if (res->n_written) {
      CK(h, cudaMemcpyAsync(out->r_payload, mo.r, res->n_written * prw, cudaMemcpyDeviceToHost, h->stream));
      CK(h, cudaMemcpyAsync(out->s_payload, mo.s, res->n_written * psw, cudaMemcpyDeviceToHost, h->stream));
    }
    cudaEventRecord(h->ev[HAPE_NSTAGES], h->stream);
    CK(h, cudaStreamSynchronize(h->stream));
  }
  res->kernel_launches = h->launches;
  stage_times(h, res);
  if (mat && r[4] > out->capacity)
    return fail(h, HAPE_ERR_OUTPUT_CAPACITY, "join produced %llu pairs > capacity %llu", (unsigned long long)r[4],
                (unsigned long long)out->capacity);
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// G simulated ranks on this one GPU (hape_debug_loopback_join): every
// device step of the G>1 path -- route() of each source shard with fan-out
// G, the count matrix, hape_exchange_plan's offsets, the AoS receive layout
// and the local join of each destination's received tuples -- with the NCCL
// transport replaced by device-to-device copies of the same segments to the
// same receive offsets.
// ---------------------------------------------------------------------------
static hape_status loopback_impl(hape_join* h, int G, bool peer, const hape_relation* Rs, const hape_relation* Ss,
                                 const hape_output* out, hape_join_result* per_dest, hape_join_result* total) {
  const hape_join_config& c = h->cfg;
  const int kw = key_width(c), prw = pay_width(c.r_payload_type), psw = pay_width(c.s_payload_type);
  if (G < 1 || G > 64 || (G & (G - 1))) return fail(h, HAPE_ERR_INVALID_ARG, "world must be a power of two <= 64");
  if (!Rs || !Ss || !total) return fail(h, HAPE_ERR_INVALID_ARG, "NULL shard arrays or result");
  if (c.world_size > 1 || h->comm) return fail(h, HAPE_ERR_UNSUPPORTED, "loopback needs a single-GPU handle");
  CKS(check_out(h, out));
  const int pws[2] = {prw, psw};
  const hape_relation* shards[2] = {Rs, Ss};
  uint64_t ntot[2] = {0, 0};
  for (int s = 0; s < 2; s++)
    for (int i = 0; i < G; i++) {
      CKS(check_rel(h, &shards[s][i], kw, pws[s], s ? "S shard" : "R shard"));
      if (shards[s][i].mem != HAPE_MEM_DEVICE)
        return fail(h, HAPE_ERR_UNSUPPORTED, "loopback shards must be device-resident");
      ntot[s] += shards[s][i].n;
    }
  if (ntot[0] >= 0xFFFFFFFFull || ntot[1] >= 0xFFFFFFFFull)
    return fail(h, HAPE_ERR_UNSUPPORTED, "loopback total >= 2^32 tuples");
  CK(h, cudaSetDevice(h->dev));
  memset(total, 0, sizeof *total);
  for (int i = 0; i < HAPE_NSTAGES; i++) h->ev_used[i] = false;
  h->launches = 0;
  size_t tb[2];
  for (int s = 0; s < 2; s++) tb[s] = tup_bytes(kw, pws[s]);
  std::vector<uint64_t> base[2];
  std::vector<uint64_t> counts[2];
  std::vector<uint32_t> hb((size_t)2 * G * (G + 1));
  if (!peer) {
    // (a2-a4) route every source shard into its region of the send buffer
    for (int s = 0; s < 2; s++) CKS(ensure(h, h->send[s], ntot[s] * tb[s] + 16));
    CKS(ensure(h, h->xb, (size_t)2 * G * (G + 1) * 4));
    uint32_t* dbounds = static_cast<uint32_t*>(h->xb.p);
    for (int s = 0; s < 2; s++) {
      base[s].assign(G + 1, 0);
      for (int i = 0; i < G; i++) {
        Src in;
        CKS(stage_in(h, &shards[s][i], kw, pws[s], h->stage[0], h->stage[1], &in));
        CKS(route(h, in, (uint32_t)G, static_cast<char*>(h->send[s].p) + base[s][i] * tb[s],
                  dbounds + ((size_t)s * G + i) * (G + 1)));
        base[s][i + 1] = base[s][i] + shards[s][i].n;
      }
    }
    // (a5) count exchange
    CK(h, cudaMemcpyAsync(hb.data(), dbounds, hb.size() * 4, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaStreamSynchronize(h->stream));
    for (int s = 0; s < 2; s++) {
      counts[s].assign((size_t)G * G, 0);
      for (int src = 0; src < G; src++) {
        const uint32_t* b = hb.data() + ((size_t)s * G + src) * (G + 1);
        for (int d = 0; d < G; d++) counts[s][(size_t)src * G + d] = b[d + 1] - b[d];
      }
    }
  } else {
    // fused form: per-destination totals of every shard (the all-gathered
    // count matrix), then every shard's peer scatter into the destinations'
    // receive buffers at its offset inside each
    const size_t nt = (size_t)G * 2 * G;
    CKS(ensure(h, h->xb, (nt + nt) * 4));
    uint32_t* tot = static_cast<uint32_t*>(h->xb.p);  // [src][s][d]
    uint32_t* cur = tot + nt;                           // [src][s][d] cursors
    CK(h, cudaMemsetAsync(tot, 0, nt * 4, h->stream));
    std::vector<Src> ins((size_t)2 * G);
    for (int s = 0; s < 2; s++)
      for (int i = 0; i < G; i++) {
        CKS(stage_in(h, &shards[s][i], kw, pws[s], h->stage[0], h->stage[1], &ins[(size_t)s * G + i]));
        CKS(route_totals(h, ins[(size_t)s * G + i], (uint32_t)G, tot + ((size_t)i * 2 + s) * G));
      }
    std::vector<uint32_t> ht(nt);
    CK(h, cudaMemcpyAsync(ht.data(), tot, nt * 4, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaStreamSynchronize(h->stream));
    std::vector<uint32_t> hc(nt);
    std::vector<void*> tab((size_t)2 * G);
    for (int s = 0; s < 2; s++) {
      counts[s].assign((size_t)G * G, 0);
      for (int d = 0; d < G; d++) {
        uint64_t run = 0;
        for (int src = 0; src < G; src++) {
          const uint32_t x = ht[((size_t)src * 2 + s) * G + d];
          counts[s][(size_t)src * G + d] = x;
          hc[((size_t)src * 2 + s) * G + d] = (uint32_t)run;
          run += x;
        }
        CKS(ensure(h, h->lb_rx[s][d], run * tb[s] + 16));
        tab[(size_t)s * G + d] = h->lb_rx[s][d].p;
      }
    }
    CKS(ensure(h, h->peer_tab, tab.size() * sizeof(void*)));
    CK(h, cudaMemcpyAsync(h->peer_tab.p, tab.data(), tab.size() * sizeof(void*), cudaMemcpyHostToDevice, h->stream));
    CK(h, cudaMemcpyAsync(cur, hc.data(), nt * 4, cudaMemcpyHostToDevice, h->stream));
    void* const* ptab = static_cast<void* const*>(h->peer_tab.p);
    for (int i = 0; i < G; i++)
      for (int s = 0; s < 2; s++)
        CKS(route_peer(h, ins[(size_t)s * G + i], (uint32_t)G, cur + ((size_t)i * 2 + s) * G, ptab + (size_t)s * G));
    CK(h, cudaStreamSynchronize(h->stream));  // (host vectors above are the copies' sources)
    h->peer_tab_dirty = true;                 // the exchange path re-uploads its own table
  }
  MatOut mo0;
  CKS(mat_targets(h, out, &mo0));
  uint64_t written = 0, required = 0;
  bool over = false;
  for (int d = 0; d < G; d++) {
    Src loc[2];
    for (int s = 0; s < 2; s++) {
      std::vector<uint64_t> soff(G), roff(G);
      uint64_t rtot = 0;
      hape_exchange_plan(G, d, counts[s].data(), soff.data(), roff.data(), &rtot);
      if (peer) {
        loc[s] = Src{PartIn{nullptr, nullptr, h->lb_rx[s][d].p}, true, (uint32_t)rtot, pws[s]};
        continue;
      }
      CKS(ensure(h, h->recv[s], rtot * tb[s] + 16));
      // the all-to-allv: source src's destination-d segment -> roff[src]
      for (int src = 0; src < G; src++) {
        const uint64_t cnt = counts[s][(size_t)src * G + d];
        if (!cnt) continue;
        const uint32_t* b = hb.data() + ((size_t)s * G + src) * (G + 1);
        CK(h, cudaMemcpyAsync(static_cast<char*>(h->recv[s].p) + roff[src] * tb[s],
                              static_cast<const char*>(h->send[s].p) + (base[s][src] + b[d]) * tb[s], cnt * tb[s],
                              cudaMemcpyDeviceToDevice, h->stream));
      }
      loc[s] = Src{PartIn{nullptr, nullptr, h->recv[s].p}, true, (uint32_t)rtot, pws[s]};
    }
    MatOut mo = mo0;
    if (mo.on) {
      const uint64_t off = std::min(written, mo.cap);
      mo.cap -= off;
      mo.r = static_cast<char*>(mo.r) + off * prw;
      mo.s = static_cast<char*>(mo.s) + off * psw;
      mo.on = mo.cap > 0;
    }
    hape_plan pl;
    CKS(local_join(h, loc, mo, nullptr, false, &pl));
    CK(h, cudaStreamSynchronize(h->stream));
    const unsigned long long* r = h->h_res;
    const uint64_t nw = mo.on ? std::min<uint64_t>(r[4], mo.cap) : 0;
    if (per_dest) {
      hape_join_result& pd = per_dest[d];
      memset(&pd, 0, sizeof pd);
      pd.local_match_count = r[0];
      pd.local_sum_r = r[1];
      pd.local_sum_s = r[2];
      pd.local_pair_checksum = r[3];
      pd.n_required = r[0];
      pd.n_written = nw;
      pd.n_items = (uint32_t)(r[5] & 0xFFFFFFFFu);
      fill_plan_fields(&pd, pl, loc[0].n, loc[1].n);
    }
    total->match_count += r[0];
    total->sum_r_payload += r[1];
    total->sum_s_payload += r[2];
    total->pair_checksum += r[3];
    written += nw;
    required += r[0];
    if (mo0.on && r[0] > nw) over = true;
  }
  total->local_match_count = total->match_count;
  total->local_sum_r = total->sum_r_payload;
  total->local_sum_s = total->sum_s_payload;
  total->local_pair_checksum = total->pair_checksum;
  total->n_written = written;
  total->n_required = required;
  total->r_local = ntot[0];
  total->s_local = ntot[1];
  total->n_partitions = (uint32_t)G;
  total->kernel_launches = h->launches;
  if (per_dest)
    for (int d = 0; d < G; d++) {
      per_dest[d].match_count = total->match_count;
      per_dest[d].sum_r_payload = total->sum_r_payload;
      per_dest[d].sum_s_payload = total->sum_s_payload;
      per_dest[d].pair_checksum = total->pair_checksum;
    }
  if (mo0.on && written && out->mem == HAPE_MEM_HOST) {
    CK(h, cudaMemcpyAsync(out->r_payload, mo0.r, written * prw, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaMemcpyAsync(out->s_payload, mo0.s, written * psw, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaStreamSynchronize(h->stream));
  }
  if (over)
    return fail(h, HAPE_ERR_OUTPUT_CAPACITY, "loopback join produced %llu pairs > capacity %llu",
                (unsigned long long)required, (unsigned long long)out->capacity);
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// the non-partitioned GPU hash join (Fig. 6's baseline; nonpart.cuh)
// ---------------------------------------------------------------------------
#include "coprocess.cuh"

template <int KW, int PRW, int PSW>
static hape_status np_launch(hape_join* h, const Src& r, const Src& s, void* table, uint32_t mask, bool mat,
                             void* mat_r, void* mat_s, unsigned long long cap, unsigned long long* acc,
                             unsigned long long* out_ctr) {
  using K = typename UW<KW>::T;
  auto* tab = static_cast<NpSlot<KW, PRW>*>(table);
  mark(h, HAPE_STAGE_NP_BUILD);
  CK(h, cudaMemsetAsync(table, 0, ((size_t)mask + 1) * sizeof(NpSlot<KW, PRW>), h->stream));
  const unsigned gmax = (unsigned)h->num_sms * 8;
  if (r.n) {
    k_np_build<KW, PRW><<<std::min<unsigned>(gmax, (r.n + NP_THREADS - 1) / NP_THREADS), NP_THREADS, 0, h->stream>>>(
        static_cast<const K*>(r.in.k), static_cast<const typename UW<PRW>::T*>(r.in.p), r.n, tab, mask);
    CK_LAUNCH(h);
  }
  mark(h, HAPE_STAGE_NP_PROBE);
  if (s.n) {
    const unsigned grid = std::min<unsigned>(gmax, (s.n + NP_THREADS - 1) / NP_THREADS);
    const uint32_t uq = (h->cfg.flags & HAPE_FLAG_R_UNIQUE) ? 1u : 0u;
    const auto* sk = static_cast<const K*>(s.in.k);
    const auto* sp = static_cast<const typename UW<PSW>::T*>(s.in.p);
    if (mat)
      k_np_probe<KW, PRW, PSW, true><<<grid, NP_THREADS, 0, h->stream>>>(sk, sp, s.n, tab, mask, uq, acc, mat_r,
                                                                         mat_s, cap, out_ctr);
    else
      k_np_probe<KW, PRW, PSW, false><<<grid, NP_THREADS, 0, h->stream>>>(sk, sp, s.n, tab, mask, uq, acc, nullptr,
                                                                          nullptr, 0, out_ctr);
    CK_LAUNCH(h);
  }
  return HAPE_OK;
}

static hape_status np_join_impl(hape_join* h, const hape_relation* R, const hape_relation* S, const hape_output* out,
                                hape_join_result* res) {
  const hape_join_config& c = h->cfg;
  const int kw = key_width(c), prw = pay_width(c.r_payload_type), psw = pay_width(c.s_payload_type);
  CKS(check_rel(h, R, kw, prw, "R"));
  CKS(check_rel(h, S, kw, psw, "S"));
  if (c.world_size > 1 || h->comm)
    return fail(h, HAPE_ERR_UNSUPPORTED, "the non-partitioned join is single-GPU (world_size 1)");
  if (R->n > (1ull << 30)) return fail(h, HAPE_ERR_UNSUPPORTED, "non-partitioned join: |R| > 2^30");
  const bool mat = out && out->capacity > 0;
  if (mat) {
    if (!out->r_payload || !out->s_payload) return fail(h, HAPE_ERR_INVALID_ARG, "output buffers NULL");
    if (out->mem != HAPE_MEM_DEVICE && out->mem != HAPE_MEM_HOST) return fail(h, HAPE_ERR_INVALID_ARG, "out.mem");
  }
  CK(h, cudaSetDevice(h->dev));
  memset(res, 0, sizeof *res);
  for (int i = 0; i < HAPE_NSTAGES; i++) h->ev_used[i] = false;
  h->launches = 0;
  mark(h, HAPE_STAGE_TOTAL);
  mark(h, HAPE_STAGE_H2D);
  Src in[2];
  CKS(stage_in(h, R, kw, prw, h->stage[0], h->stage[1], &in[0]));
  CKS(stage_in(h, S, kw, psw, h->stage[2], h->stage[3], &in[1]));
  const uint32_t tbits = std::max<uint32_t>(10, ceil_log2_u64(2 * std::max<uint64_t>(R->n, 1)));
  const size_t slot = (kw == 4) ? 16 : 32;
  CKS(ensure(h, h->np_table, ((size_t)1 << tbits) * slot));
  CKS(ensure(h, h->small, 64));
  unsigned long long* acc = at<unsigned long long>(h, 0);
  unsigned long long* out_ctr = acc + 4;
  CK(h, cudaMemsetAsync(acc, 0, 5 * 8, h->stream));
  void* mat_r = nullptr;
  void* mat_s = nullptr;
  if (mat) {
    mat_r = out->r_payload;
    mat_s = out->s_payload;
    if (out->mem == HAPE_MEM_HOST) {
      CKS(ensure(h, h->outst[0], out->capacity * prw));
      CKS(ensure(h, h->outst[1], out->capacity * psw));
      mat_r = h->outst[0].p;
      mat_s = h->outst[1].p;
    }
  }
  const uint32_t mask = (1u << tbits) - 1;
  const unsigned long long cap = mat ? out->capacity : 0;
  void* tab = h->np_table.p;
#define HAPE_NP(KW, PRW, PSW) np_launch<KW, PRW, PSW>(h, in[0], in[1], tab, mask, mat, mat_r, mat_s, cap, acc, out_ctr)
  hape_status st;
  if (kw == 4) {
    if (prw == 4) st = psw == 4 ? HAPE_NP(4, 4, 4) : HAPE_NP(4, 4, 8);
    else st = psw == 4 ? HAPE_NP(4, 8, 4) : HAPE_NP(4, 8, 8);
  } else {
    if (prw == 4) st = psw == 4 ? HAPE_NP(8, 4, 4) : HAPE_NP(8, 4, 8);
    else st = psw == 4 ? HAPE_NP(8, 8, 4) : HAPE_NP(8, 8, 8);
  }
#undef HAPE_NP
  CKS(st);
  mark(h, HAPE_STAGE_FINALIZE);
  CK(h, cudaMemcpyAsync(h->h_res, acc, 5 * 8, cudaMemcpyDeviceToHost, h->stream));
  CK(h, cudaStreamSynchronize(h->stream));
  const unsigned long long* r = h->h_res;
  res->match_count = res->local_match_count = r[0];
  res->sum_r_payload = res->local_sum_r = r[1];
  res->sum_s_payload = res->local_sum_s = r[2];
  res->pair_checksum = res->local_pair_checksum = r[3];
  res->n_required = r[0];
  res->n_written = mat ? std::min<uint64_t>(r[4], out->capacity) : 0;
  res->r_local = R->n;
  res->s_local = S->n;
  res->passes = 0;
  res->n_partitions = 1;
  if (mat && out->mem == HAPE_MEM_HOST && res->n_written) {
    CK(h, cudaMemcpyAsync(out->r_payload, mat_r, res->n_written * prw, cudaMemcpyDeviceToHost, h->stream));
    CK(h, cudaMemcpyAsync(out->s_payload, mat_s, res->n_written * psw, cudaMemcpyDeviceToHost, h->stream));
  }
  cudaEventRecord(h->ev[HAPE_NSTAGES], h->stream);
  CK(h, cudaStreamSynchronize(h->stream));
  res->kernel_launches = h->launches;
  stage_times(h, res);
  if (mat && r[4] > out->capacity)
    return fail(h, HAPE_ERR_OUTPUT_CAPACITY, "join produced %llu pairs > capacity %llu", (unsigned long long)r[4],
                (unsigned long long)out->capacity);
  return HAPE_OK;
}

// ---------------------------------------------------------------------------
// exported ABI
// ---------------------------------------------------------------------------
extern "C" {

const char* hape_version(void) { return "hape-b200 1.2 (sm_100a, ABI 3)"; }

const char* hape_status_string(hape_status s) {
  switch (s) {
    case HAPE_OK: return "HAPE_OK";
    case HAPE_ERR_INVALID_ARG: return "HAPE_ERR_INVALID_ARG";
    case HAPE_ERR_CUDA: return "HAPE_ERR_CUDA";
    case HAPE_ERR_OOM: return "HAPE_ERR_OOM";
    case HAPE_ERR_OUTPUT_CAPACITY: return "HAPE_ERR_OUTPUT_CAPACITY";
    case HAPE_ERR_NCCL: return "HAPE_ERR_NCCL";
    case HAPE_ERR_UNSUPPORTED: return "HAPE_ERR_UNSUPPORTED";
  }
  return "HAPE_ERR_UNKNOWN";
}

hape_status hape_join_create(const hape_join_config* cfg, hape_join** out_handle) {
  if (!cfg || !out_handle) return HAPE_ERR_INVALID_ARG;
  *out_handle = nullptr;
  if (cfg->key_type != HAPE_INT32 && cfg->key_type != HAPE_INT64) return HAPE_ERR_INVALID_ARG;
  if ((cfg->r_payload_type != HAPE_INT32 && cfg->r_payload_type != HAPE_INT64) ||
      (cfg->s_payload_type != HAPE_INT32 && cfg->s_payload_type != HAPE_INT64))
    return HAPE_ERR_INVALID_ARG;
  if (cfg->part_fn != HAPE_PART_HASH && cfg->part_fn != HAPE_PART_IDENTITY) return HAPE_ERR_INVALID_ARG;
  if (cfg->radix_passes < 0 || cfg->radix_passes > 2) return HAPE_ERR_INVALID_ARG;
  if (cfg->radix_bits[0] < 0 || cfg->radix_bits[1] < 0 || cfg->radix_bits[0] > (int)kMaxBitsPerPass ||
      cfg->radix_bits[1] > (int)kMaxBitsPerPass)
    return HAPE_ERR_INVALID_ARG;
  const int world = cfg->world_size > 1 ? cfg->world_size : 1;
  if (cfg->world_size < 0 || (world & (world - 1)) != 0 || world > 64) return HAPE_ERR_INVALID_ARG;
  if (cfg->rank < 0 || cfg->rank >= world) return HAPE_ERR_INVALID_ARG;
  if (world > 1 && !cfg->nccl_comm) return HAPE_ERR_INVALID_ARG;
  if (cfg->device < 0) return HAPE_ERR_INVALID_ARG;
  if (cfg->flags & ~(HAPE_FLAG_R_UNIQUE | HAPE_FLAG_LINKED)) return HAPE_ERR_INVALID_ARG;
  int ndev = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess || cfg->device >= ndev) {
    (void)cudaGetLastError();
    return HAPE_ERR_CUDA;
  }
  hape_join* h = new hape_join();
  h->cfg = *cfg;
  h->dev = cfg->device;
  h->comm = static_cast<ncclComm_t>(cfg->nccl_comm);
  hape_status st = HAPE_OK;
  do {
    if (cudaSetDevice(h->dev) != cudaSuccess) { st = HAPE_ERR_CUDA; break; }
    cudaDeviceGetAttribute(&h->num_sms, cudaDevAttrMultiProcessorCount, h->dev);
    if (cfg->stream) {
      h->stream = static_cast<cudaStream_t>(cfg->stream);
    } else {
      if (cudaStreamCreateWithFlags(&h->stream, cudaStreamNonBlocking) != cudaSuccess) { st = HAPE_ERR_CUDA; break; }
      h->own_stream = true;
    }
    for (auto& e : h->ev)
      if (cudaEventCreate(&e) != cudaSuccess) { st = HAPE_ERR_CUDA; break; }
    if (cudaStreamCreateWithFlags(&h->copy_stream, cudaStreamNonBlocking) != cudaSuccess ||
        cudaEventCreateWithFlags(&h->ev_copy, cudaEventDisableTiming) != cudaSuccess) { st = HAPE_ERR_CUDA; break; }
    if (st != HAPE_OK) break;
    if (cudaMallocHost(&h->h_res, 16 * sizeof(unsigned long long)) != cudaSuccess) { st = HAPE_ERR_OOM; break; }
    if (cudaMallocHost(&h->h_x, 2 * 64 * sizeof(uint32_t)) != cudaSuccess) { st = HAPE_ERR_OOM; break; }
    if (cfg->max_r || cfg->max_s) {
      hape_plan pl;
      if (make_plan(h, cfg->max_r, cfg->max_s, &pl) == HAPE_OK) {
        const CallLayout L = layout_for(h, pl, cfg->max_r, cfg->max_s);
        if (ensure(h, h->small, L.total) != HAPE_OK) { st = HAPE_ERR_OOM; break; }
      }
    }
  } while (0);
  if (st != HAPE_OK) {
    (void)cudaGetLastError();
    hape_join_destroy(h);
    return st;
  }
  *out_handle = h;
  return HAPE_OK;
}

hape_status hape_coprocess_join(hape_join* h, const hape_relation* R, const hape_relation* S,
                                const hape_coprocess_config* cp, const hape_output* out, hape_join_result* res) {
  if (!h) return HAPE_ERR_INVALID_ARG;
  if (!res) return fail(h, HAPE_ERR_INVALID_ARG, "res is NULL");
  try {
    const hape_status st = coprocess_impl(h, R, S, cp, out, res);
    h->in_coprocess = false;
    return st;
  } catch (...) {
    h->in_coprocess = false;
    return fail(h, HAPE_ERR_CUDA, "unexpected C++ exception (host partitioning threads)");
  }
}

hape_status hape_host_partition(const hape_relation* rel, hape_dtype key_type, hape_dtype payload_type,
                                hape_part_fn part_fn, uint32_t fanout_bits, int threads, void* out_keys,
                                void* out_payloads, uint64_t* out_bounds) {
  try {
    return host_partition(rel, key_type, payload_type, part_fn, fanout_bits, threads, out_keys, out_payloads,
                          out_bounds);
  } catch (...) {
    return HAPE_ERR_INVALID_ARG;
  }
}

hape_status hape_join_destroy(hape_join* h) {
  if (!h) return HAPE_OK;
  cudaSetDevice(h->dev);
  if (h->stream) cudaStreamSynchronize(h->stream);
  for (auto& b : h->stage)
    if (b.p) cudaFree(b.p);
  DevBuf* groups[] = {h->ping, h->pong, h->send, h->recv};
  for (DevBuf* g : groups)
    for (int i = 0; i < 2; i++)
      if (g[i].p) cudaFree(g[i].p);
  for (auto& b : h->outst)
    if (b.p) cudaFree(b.p);
  if (h->gexec) cudaGraphExecDestroy(h->gexec);
  if (h->small.p) cudaFree(h->small.p);
  if (h->route_ws.p) cudaFree(h->route_ws.p);
  for (int s2 = 0; s2 < 2; s2++) {
    close_peers(h, s2);
    if (h->prx[s2].p) cudaFree(h->prx[s2].p);
    for (auto& b : h->lb_rx[s2])
      if (b.p) cudaFree(b.p);
  }
  if (h->peer_tab.p) cudaFree(h->peer_tab.p);
  for (auto& b : h->lbuf)
    if (b.p) cudaFree(b.p);
  if (h->xipc.p) cudaFree(h->xipc.p);
  if (h->h_x) cudaFreeHost(h->h_x);
  if (h->xb.p) cudaFree(h->xb.p);
  if (h->np_table.p) cudaFree(h->np_table.p);
  if (h->h_res) cudaFreeHost(h->h_res);
  if (h->h_bounds) cudaFreeHost(h->h_bounds);
  for (auto& p : h->hp)
    if (p) cudaFreeHost(p);
  for (auto& set : h->cpst)
    for (auto& b : set)
      if (b.p) cudaFree(b.p);
  for (auto& pr : h->ev_h2d)
    for (auto& e : pr)
      if (e) cudaEventDestroy(e);
  for (auto& e : h->ev)
    if (e) cudaEventDestroy(e);
  if (h->copy_stream) { cudaStreamSynchronize(h->copy_stream); cudaStreamDestroy(h->copy_stream); }
  if (h->ev_copy) cudaEventDestroy(h->ev_copy);
  if (h->own_stream && h->stream) cudaStreamDestroy(h->stream);
  (void)cudaGetLastError();
  delete h;
  return HAPE_OK;
}

const char* hape_last_error(const hape_join* h) { return h ? h->err.c_str() : "NULL handle"; }

hape_status hape_join_plan(const hape_join* h, uint64_t n_r, uint64_t n_s, hape_plan* out) {
  if (!h || !out) return HAPE_ERR_INVALID_ARG;
  return make_plan(h, n_r, n_s, out);
}

hape_status hape_radix_join(hape_join* h, const hape_relation* R, const hape_relation* S, const hape_output* out,
                            hape_join_result* res) {
  if (!h) return HAPE_ERR_INVALID_ARG;
  if (!res) return fail(h, HAPE_ERR_INVALID_ARG, "res is NULL");
  try {
    return join_impl(h, R, S, out, res);
  } catch (...) {
    return fail(h, HAPE_ERR_CUDA, "unexpected C++ exception");
  }
}

hape_status hape_nonpartitioned_join(hape_join* h, const hape_relation* R, const hape_relation* S,
                                     const hape_output* out, hape_join_result* res) {
  if (!h) return HAPE_ERR_INVALID_ARG;
  if (!res) return fail(h, HAPE_ERR_INVALID_ARG, "res is NULL");
  try {
    return np_join_impl(h, R, S, out, res);
  } catch (...) {
    return fail(h, HAPE_ERR_CUDA, "unexpected C++ exception");
  }
}

hape_status hape_debug_partition(hape_join* h, const hape_relation* rel, int is_s, const hape_plan* plan_in,
                                 void* out_keys, void* out_payloads, uint32_t* out_bounds, hape_plan* plan_out) {
  if (!h) return HAPE_ERR_INVALID_ARG;
  const hape_join_config& c = h->cfg;
  const int kw = key_width(c), pw = pay_width(is_s ? c.s_payload_type : c.r_payload_type);
  CKS(check_rel(h, rel, kw, pw, "rel"));
  if (rel->n && (!out_keys || !out_payloads)) return fail(h, HAPE_ERR_INVALID_ARG, "outputs NULL");
  if (!out_bounds) return fail(h, HAPE_ERR_INVALID_ARG, "out_bounds NULL");
  CK(h, cudaSetDevice(h->dev));
  hape_plan pl;
  if (plan_in) pl = *plan_in;
  else if (make_plan(h, rel->n, rel->n, &pl) != HAPE_OK) return fail(h, HAPE_ERR_INVALID_ARG, "invalid plan");
  if (pl.passes < 1 || pl.passes > 2 || pl.bits[0] > kMaxBitsPerPass || pl.bits[1] > kMaxBitsPerPass)
    return fail(h, HAPE_ERR_INVALID_ARG, "invalid plan");
  h->launches = 0;
  Src in;
  CKS(stage_in(h, rel, kw, pw, h->stage[0], h->stage[1], &in));
  const CallLayout L = layout_for(h, pl, rel->n, rel->n);
  CKS(ensure(h, h->small, L.total));
  CKS(ensure(h, h->ping[0], ping_bytes(h, pl, rel->n, tup_bytes(kw, pw))));
  CKS(ensure(h, h->pong[0], rel->n * tup_bytes(kw, pw) + 16));
  {
    const uint64_t nn[1] = {rel->n};
    const int pp[1] = {pw};
    CKS(ensure_pass_ws(h, pl, nn, pp, 1));
  }
  CK(h, cudaMemsetAsync(at<char>(h, L.zero_lo), 0, L.zero_hi - L.zero_lo, h->stream));
  PassIO io[2];
  io[0] = PassIO{in, h->ping[0].p, h->pong[0].p};
  const void* ft[2];
  const uint32_t* fb[2];
  CKS(run_partition_stages(h, pl, L, io, 1, ft, fb));
  const uint64_t Q = 1ull << (pl.bits[0] + (pl.passes == 2 ? pl.bits[1] : 0));
  CKS(launch_unpack(h, kw, pw, ft[0], (uint32_t)rel->n, out_keys, out_payloads));
  CK(h, cudaMemcpyAsync(out_bounds, fb[0], (Q + 1) * 4, cudaMemcpyDeviceToDevice, h->stream));
  CK(h, cudaStreamSynchronize(h->stream));
  if (plan_out) *plan_out = pl;
  return HAPE_OK;
}

hape_status hape_join_stream(const hape_join* h, void** out_stream) {
  if (!h || !out_stream) return HAPE_ERR_INVALID_ARG;
  *out_stream = h->stream;
  return HAPE_OK;
}

hape_status hape_debug_route(hape_join* h, const hape_relation* rel, int is_s, int fanout, void* out_keys,
                             void* out_payloads, uint32_t* out_bounds) {
  if (!h) return HAPE_ERR_INVALID_ARG;
  try {
    const hape_join_config& c = h->cfg;
    const int kw = key_width(c), pw = pay_width(is_s ? c.s_payload_type : c.r_payload_type);
    CKS(check_rel(h, rel, kw, pw, "rel"));
    if (fanout < 1 || fanout > 4096 || (fanout & (fanout - 1)))
      return fail(h, HAPE_ERR_INVALID_ARG, "fanout must be a power of two in [1, 4096]");
    if (rel->n && (!out_keys || !out_payloads)) return fail(h, HAPE_ERR_INVALID_ARG, "outputs NULL");
    if (!out_bounds) return fail(h, HAPE_ERR_INVALID_ARG, "out_bounds NULL");
    CK(h, cudaSetDevice(h->dev));
    h->launches = 0;
    Src in;
    CKS(stage_in(h, rel, kw, pw, h->stage[0], h->stage[1], &in));
    CKS(ensure(h, h->send[0], rel->n * tup_bytes(kw, pw) + 16));
    CKS(ensure(h, h->xb, ((size_t)fanout + 1) * 4));
    CKS(route(h, in, (uint32_t)fanout, h->send[0].p, static_cast<uint32_t*>(h->xb.p)));
    CKS(launch_unpack(h, kw, pw, h->send[0].p, (uint32_t)rel->n, out_keys, out_payloads));
    CK(h, cudaMemcpyAsync(out_bounds, h->xb.p, ((size_t)fanout + 1) * 4, cudaMemcpyDeviceToDevice, h->stream));
    CK(h, cudaStreamSynchronize(h->stream));
    return HAPE_OK;
  } catch (...) {
    return fail(h, HAPE_ERR_CUDA, "unexpected C++ exception");
  }
}

hape_status hape_debug_loopback_join(hape_join* h, int world, int peer, const hape_relation* R_shards,
                                     const hape_relation* S_shards, const hape_output* out,
                                     hape_join_result* per_dest, hape_join_result* total) {
  if (!h) return HAPE_ERR_INVALID_ARG;
  try {
    return loopback_impl(h, world, peer != 0, R_shards, S_shards, out, per_dest, total);
  } catch (...) {
    return fail(h, HAPE_ERR_CUDA, "unexpected C++ exception");
  }
}

hape_status hape_nccl_unique_id(void* out_id_128) {
  if (!out_id_128) return HAPE_ERR_INVALID_ARG;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId size");
  ncclUniqueId id;
  if (ncclGetUniqueId(&id) != ncclSuccess) return HAPE_ERR_NCCL;
  memcpy(out_id_128, &id, sizeof id);
  return HAPE_OK;
}

hape_status hape_nccl_comm_init(const void* id_128, int world_size, int rank, int device, void** out_comm) {
  if (!id_128 || !out_comm || world_size < 1 || rank < 0 || rank >= world_size) return HAPE_ERR_INVALID_ARG;
  if (cudaSetDevice(device) != cudaSuccess) { (void)cudaGetLastError(); return HAPE_ERR_CUDA; }
  ncclUniqueId id;
  memcpy(&id, id_128, sizeof id);
  ncclComm_t comm;
  if (ncclCommInitRank(&comm, world_size, id, rank) != ncclSuccess) return HAPE_ERR_NCCL;
  *out_comm = comm;
  return HAPE_OK;
}

hape_status hape_nccl_comm_destroy(void* comm) {
  if (!comm) return HAPE_OK;
  return ncclCommDestroy(static_cast<ncclComm_t>(comm)) == ncclSuccess ? HAPE_OK : HAPE_ERR_NCCL;
}

}  // extern "C"
