// kernels.cuh -- sm_100a kernels of the partitioned radix hash equi-join.
//
// PAPER.md §4.1 (P528-598, Figs. 3-4) is the method:
//   * a partitioning pass reads "a chunk of the input (at a time) in the
//     scratchpad and reorganize[s] it in such a way that elements belonging
//     to the same output partition are located in consecutive scratchpad
//     entries. Then, we scan the scratchpad and write each tuple to its
//     corresponding output partition" (P579-584)  -> k_scatter;
//   * its write offsets come from histogram + exclusive scan, the two-scan
//     method of [27] that BASELINE.json's north_star mandates (the paper
//     contrasts it with its linked buffers, P593-597)  -> k_hist, k_scan;
//   * fan-out is bounded by the scratchpad that consolidates the stores, so
//     the join runs 1-2 passes (P531-534, P589-593);
//   * per co-partition: "load the smaller partition to the scratchpad, build
//     the hash-table using atomic operations and probe with the tuples of the
//     corresponding partition" (P537-540)  -> k_build_probe;
//   * the micro-benchmark consumer: count and sum over each payload column
//     (P789-793), fused into the probe epilogue.
//
// Data layout in HBM: caller columns are structure-of-arrays; the ping-pong
// workspace written by the radix passes holds (key, payload) tuples (AoS,
// struct Tup); uint32 tuple indices (n < 2^32 per relation per rank).
// Nothing here is a dense contraction: no tensor cores.
#pragma once
#include <cstdint>
#include <type_traits>
#include <cuda_runtime.h>

namespace hape {

// --------------------------------------------------------------------------
// widths and the partition function (reading R1)
// --------------------------------------------------------------------------
template <int W> struct UW;
template <> struct UW<4> { using T = uint32_t; using S = int32_t; };
template <> struct UW<8> { using T = uint64_t; using S = int64_t; };

__device__ __forceinline__ uint32_t fmix32(uint32_t h) {
  h ^= h >> 16; h *= 0x85ebca6bu;
  h ^= h >> 13; h *= 0xc2b2ae35u;
  h ^= h >> 16;
  return h;
}

__device__ __forceinline__ uint64_t fmix64(uint64_t x) {
  x ^= x >> 30; x *= 0xbf58476d1ce4e5b9ull;
  x ^= x >> 27; x *= 0x94d049bb133111ebull;
  x ^= x >> 31;
  return x;
}

// inverses of the two mixers (debug entry points only: they hand the
// workspace's h(k) back to the caller as the key k)
__device__ __forceinline__ uint32_t fmix32_inv(uint32_t h) {
  h ^= h >> 16; h *= 0x7ed1b41du;
  h ^= (h >> 13) ^ (h >> 26); h *= 0xa5cb9243u;
  h ^= h >> 16;
  return h;
}
__device__ __forceinline__ uint64_t fmix64_inv(uint64_t x) {
  x ^= (x >> 31) ^ (x >> 62); x *= 0x319642b2d24d8ec3ull;
  x ^= (x >> 27) ^ (x >> 54); x *= 0x96de1b173f119089ull;
  x ^= (x >> 30) ^ (x >> 60);
  return x;
}

// h(k): bijective mixer of the key bit pattern, or identity (P802-804)
// (IDENT is a template parameter: the per-tuple paths carry no branch on it)
template <int KW, bool IDENT>
__device__ __forceinline__ uint64_t part_hash(typename UW<KW>::T k) {
  if constexpr (IDENT) return (uint64_t)k;
  else if constexpr (KW == 4) return (uint64_t)fmix32(k);
  else return fmix64(k);
}

// bucket = (h >> shift) & mask  (R3: dest = top bits; pass 2 = bits
// [0, B2), pass 1 = bits [B2, B2+B1): the final co-partition = low B1+B2 bits)
struct BitField { uint32_t shift; uint32_t mask; };

__device__ __forceinline__ uint32_t bucket_of(uint64_t h, BitField bf) {
  return (uint32_t)(h >> bf.shift) & bf.mask;
}

// pair-checksum term (R10): mix(p,q) = fmix64(p*phi + q)
__device__ __forceinline__ uint64_t pair_mix(int64_t p, int64_t q) {
  return fmix64((uint64_t)p * 0x9E3779B97F4A7C15ull + (uint64_t)q);
}

// --------------------------------------------------------------------------
// segment -> CTA chunk mapping, shared by k_hist and k_scatter of one pass
// (the offsets are only right if both kernels see identical chunks)
// --------------------------------------------------------------------------
// Linked-buffer chains (the paper's single-scan partitioning, P593-597;
// SURVEY §8.f NEXT-2): bucket b's tuples sit in a chain of fixed-size
// buffers of `buf` tuples, buffer k of the chain at physical id dir[b*kmax+k]-1;
// owner[id] / kidx[id] invert it, cnt[b] is the bucket's tuple count, *pool
// the number of buffers handed out.
struct LinkMap {
  uint32_t* cnt;
  uint32_t* pool;
  uint32_t* dir;
  uint32_t* owner;
  uint32_t* kidx;
  uint32_t kmax;
  uint32_t buf;
};

struct SegMap {
  const uint32_t* bounds;  // nseg+1 segment bounds (device) or nullptr: one segment [0, n)
  uint32_t nseg;
  uint32_t cps;            // CTAs per segment
  uint32_t n;
  // chained input (a pass reading linked buffers): CTA j reads buffer j,
  // its segment is the buffer's owner; nseg = upper bound of buffers
  const uint32_t* owner = nullptr;
  const uint32_t* kidx = nullptr;
  const uint32_t* cnt = nullptr;
  const uint32_t* pool = nullptr;
  uint32_t buf = 0;
};

// buffer j of a chained input: segment and physical range (empty when j is
// beyond the buffers handed out)
__device__ __forceinline__ void buf_chunk(const SegMap& m, uint32_t cta, uint32_t& seg, uint32_t& j,
                                          uint32_t& lo, uint32_t& hi) {
  j = 0;
  if (cta >= *m.pool) { seg = 0; lo = hi = 0; return; }
  seg = m.owner[cta];
  const uint32_t k = m.kidx[cta];
  const uint32_t fill = min(m.buf, m.cnt[seg] - k * m.buf);
  lo = cta * m.buf;
  hi = lo + fill;
}

__device__ __forceinline__ void seg_chunk(const SegMap& m, uint32_t cta, uint32_t& seg,
                                          uint32_t& j, uint32_t& lo, uint32_t& hi) {
  if (m.owner) { buf_chunk(m, cta, seg, j, lo, hi); return; }
  seg = cta / m.cps;
  j = cta - seg * m.cps;
  uint32_t b = m.bounds ? m.bounds[seg] : 0u;
  uint32_t e = m.bounds ? m.bounds[seg + 1] : m.n;
  uint64_t len = (uint64_t)(e - b);
  lo = b + (uint32_t)((len * j) / m.cps);
  hi = b + (uint32_t)((len * (j + 1)) / m.cps);
}

// Tile-granular split of a segment (claiming scatters, whose chunking is free):
// every chunk is whole tiles of T tuples, so only a segment's last tile takes
// the partial-tile path.
__device__ __forceinline__ void seg_chunk_tiles(const SegMap& m, uint32_t cta, uint32_t T, uint32_t& seg,
                                                uint32_t& j, uint32_t& lo, uint32_t& hi) {
  if (m.owner) { buf_chunk(m, cta, seg, j, lo, hi); return; }
  seg = cta / m.cps;
  j = cta - seg * m.cps;
  const uint32_t b = m.bounds ? m.bounds[seg] : 0u;
  const uint32_t e = m.bounds ? m.bounds[seg + 1] : m.n;
  const uint32_t len = e - b;
  const uint64_t nt = (len + (uint64_t)T - 1) / T;
  const uint64_t t0 = nt * j / m.cps, t1 = nt * (j + 1) / m.cps;
  lo = b + (uint32_t)(t0 * T < len ? t0 * T : len);
  hi = b + (uint32_t)(t1 * T < len ? t1 * T : len);
}

// --------------------------------------------------------------------------
// small block primitives
// --------------------------------------------------------------------------
__device__ __forceinline__ uint32_t warp_incl_scan(uint32_t v) {
  const int lane = threadIdx.x & 31;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    uint32_t t = __shfl_up_sync(0xffffffffu, v, o);
    if (lane >= o) v += t;
  }
  return v;
}

// In-place exclusive scan of a[0..n) in shared memory; returns the total.
// All threads of the block must call it.  wtmp: >= 33 words of smem.
template <int BD>
__device__ uint32_t block_exscan_smem(uint32_t* a, int n, uint32_t* wtmp) {
  const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
  constexpr int NW = BD / 32;
  const int c = (n + BD - 1) / BD;
  const int lo = min(tid * c, n), hi = min(lo + c, n);
  uint32_t s = 0;
  for (int i = lo; i < hi; i++) s += a[i];
  uint32_t incl = warp_incl_scan(s);
  if (lane == 31) wtmp[warp] = incl;
  __syncthreads();
  if (warp == 0) {
    uint32_t v = lane < NW ? wtmp[lane] : 0u;
    uint32_t vi = warp_incl_scan(v);
    if (lane < NW) wtmp[lane] = vi - v;
    if (lane == 31) wtmp[32] = vi;
  }
  __syncthreads();
  uint32_t ex = wtmp[warp] + incl - s;
  for (int i = lo; i < hi; i++) { uint32_t t = a[i]; a[i] = ex; ex += t; }
  uint32_t total = wtmp[32];
  __syncthreads();
  return total;
}

// Conflict-free exclusive scan of a[0..n) in shared memory by the first NT
// threads: warp w owns a contiguous chunk and reads it lane-strided (one
// word per bank per access); PACK writes (start | end << 16) instead of the
// start.  wt: >= NT/32 words.  Two barriers (bar id 1 when NAMED, else 0).
template <int NT, bool PACK, bool NAMED>
__device__ __forceinline__ uint32_t block_exscan_strided(uint32_t* a, uint32_t n, uint32_t* wt) {
  constexpr int NW = NT / 32;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t chunk = ((n + NW - 1) / NW + 31) & ~31u;
  const uint32_t c0 = min(n, warp * chunk), c1 = min(n, c0 + chunk);
  uint32_t s = 0;
  for (uint32_t i = c0 + lane; i < c1; i += 32) s += a[i];
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
  if (lane == 0) wt[warp] = s;
  if constexpr (NAMED) asm volatile("bar.sync 1, %0;" ::"n"(NT) : "memory");
  else __syncthreads();
  uint32_t carry = 0, total = 0;
  for (int w = 0; w < NW; w++) {
    const uint32_t x = wt[w];
    carry += w < warp ? x : 0u;
    total += x;
  }
  for (uint32_t b = c0; b < c1; b += 32) {
    const uint32_t i = b + lane;
    const uint32_t v = i < c1 ? a[i] : 0u;
    const uint32_t inc = warp_incl_scan(v);
    const uint32_t ex = carry + inc - v;
    if (i < c1) a[i] = PACK ? (ex | ((ex + v) << 16)) : ex;
    carry += __shfl_sync(0xffffffffu, inc, 31);
  }
  if constexpr (NAMED) asm volatile("bar.sync 1, %0;" ::"n"(NT) : "memory");
  else __syncthreads();
  return total;
}

// --------------------------------------------------------------------------
// Workspace tuple: the radix passes write (key, payload) pairs (AoS), so a
// bucket run of r tuples is one contiguous r*sizeof(Tup)-byte store run
// instead of two half-length column runs -- the write-combining the paper's
// scratchpad reorder is for (P579-589) then works on twice the bytes.
// --------------------------------------------------------------------------
template <int KW, int PW>
struct alignas((KW + PW) <= 8 ? 8 : 16) Tup {
  typename UW<KW>::T k;
  typename UW<PW>::T v;
};

// streaming (evict-first) load of one tuple
template <int KW, int PW>
__device__ __forceinline__ Tup<KW, PW> ldcs_tup(const Tup<KW, PW>* p) {
  Tup<KW, PW> x;
  if constexpr (sizeof(Tup<KW, PW>) == 8) {
    const uint2 w = __ldcs(reinterpret_cast<const uint2*>(p));
    x = *reinterpret_cast<const Tup<KW, PW>*>(&w);
  } else {
    const uint4 w = __ldcs(reinterpret_cast<const uint4*>(p));
    x = *reinterpret_cast<const Tup<KW, PW>*>(&w);
  }
  return x;
}

// Input of a partitioning pass: caller SoA columns (pass 1) or workspace AoS
// tuples (pass 2, and pass 1 after the multi-GPU exchange).
struct PartIn {
  const void* k;   // SoA keys   (AOS = false)
  const void* p;   // SoA payloads
  const void* t;   // AoS tuples (AOS = true)
};

__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count));
}
__device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
#ifndef HAPE_MBAR_SUSPEND
#define HAPE_MBAR_SUSPEND 0
#endif
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t phase) {
#if HAPE_MBAR_SUSPEND
  // suspend inside try_wait (time-limit hint) instead of re-issuing it: a
  // waiting warp does not take issue slots from the warps that have work
  uint32_t ok = 0;
  while (true) {
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2, %3;\n selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(smem_u32(bar)), "r"(phase), "r"(HAPE_MBAR_SUSPEND)
        : "memory");
    if (ok) return;
  }
#else
  asm volatile(
      "{\n .reg .pred p;\n WAIT_%=:\n"
      " mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
      " @!p bra WAIT_%=;\n}\n" ::"r"(smem_u32(bar)),
      "r"(phase)
      : "memory");
#endif
}
// producer-side wait: the thread is suspended inside try_wait (time-limit
// hint) instead of polling, so a warp that is far ahead does not steal issue
// slots from the consumers
__device__ __forceinline__ void mbar_wait_backoff(uint64_t* bar, uint32_t phase) {
  uint32_t ok = 0;
  while (true) {
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2, %3;\n selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(smem_u32(bar)), "r"(phase), "r"(1000000u)
        : "memory");
    if (ok) return;
  }
}
__device__ __forceinline__ uint64_t policy_evict_first() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}
// 1-D bulk copy global -> shared (TMA engine), completion on an mbarrier,
// streamed-once data marked evict-first in L2
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar,
                                         uint64_t pol) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::"r"(
          smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(pol)
      : "memory");
}
// L2 prefetch of [src, src + bytes) rounded out to 16-byte boundaries (bulk
// engine, no destination, no completion tracking)
__device__ __forceinline__ void bulk_prefetch_l2(const void* src, size_t bytes) {
  const uintptr_t a = reinterpret_cast<uintptr_t>(src);
  const uintptr_t a0 = a & ~(uintptr_t)15, a1 = (a + bytes + 15) & ~(uintptr_t)15;
  asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(a0), "r"((uint32_t)(a1 - a0)) : "memory");
}
// copy [src, src + bytes) rounded out to 16-byte boundaries; returns the
// byte offset of src inside the destination buffer
__device__ __forceinline__ uint32_t bulk_g2s_any(void* dst, const void* src, size_t bytes, uint64_t* bar,
                                                 uint64_t pol, uint32_t* tx) {
  const uintptr_t a = reinterpret_cast<uintptr_t>(src);
  const uintptr_t a0 = a & ~(uintptr_t)15, a1 = (a + bytes + 15) & ~(uintptr_t)15;
  bulk_g2s(dst, reinterpret_cast<const void*>(a0), (uint32_t)(a1 - a0), bar, pol);
  *tx += (uint32_t)(a1 - a0);
  return (uint32_t)(a - a0);
}

// --------------------------------------------------------------------------
// a6: radix histogram of one pass.  One contiguous chunk per CTA; keys only
// (w_k bytes per tuple from SoA input; the whole tuple from AoS input);
// shared-memory counters (P166-168: "use shared memory to store histograms").
// Output hist[(seg*P + p)*cps + j] (partition-major inside each segment, so
// the segment's exclusive scan IS the offsets) and the row totals
// rowsum[seg*P + p].  16-byte vector loads, 4 in flight per thread.
// --------------------------------------------------------------------------
constexpr int HIST_THREADS = 512;
constexpr int HIST_VEC = 4;

template <int KW, int PW, bool AOS, bool IDENT>
__global__ void __launch_bounds__(HIST_THREADS)
k_hist(PartIn in, SegMap m, BitField bf, uint32_t P, uint32_t* __restrict__ hist,
       uint32_t* __restrict__ rowsum) {
  extern __shared__ uint32_t sh_cnt[];
  using K = typename UW<KW>::T;
  using E = typename std::conditional<AOS, Tup<KW, PW>, K>::type;  // element read
  constexpr int ES = sizeof(E);
  constexpr int PER = 16 / ES;  // elements per 16-byte vector
  const E* __restrict__ base = static_cast<const E*>(AOS ? in.t : in.k);
  auto key_of = [](const E& e) -> K {
    if constexpr (AOS) return e.k;
    else return e;
  };
  for (uint32_t i = threadIdx.x; i < P; i += HIST_THREADS) sh_cnt[i] = 0;
  __syncthreads();
  uint32_t seg, j, lo, hi;
  seg_chunk(m, blockIdx.x, seg, j, lo, hi);
  uint32_t vlo = lo;
  while (vlo < hi && (reinterpret_cast<uintptr_t>(base + vlo) & 15)) vlo++;
  const uint32_t nvec = (hi - vlo) / PER;
  const uint32_t vhi = vlo + nvec * PER;
  for (uint32_t i = lo + threadIdx.x; i < vlo; i += HIST_THREADS)
    atomicAdd(&sh_cnt[bucket_of(part_hash<KW, IDENT>(key_of(base[i])), bf)], 1u);
  for (uint32_t i = vhi + threadIdx.x; i < hi; i += HIST_THREADS)
    atomicAdd(&sh_cnt[bucket_of(part_hash<KW, IDENT>(key_of(base[i])), bf)], 1u);
  const uint4* __restrict__ vk = reinterpret_cast<const uint4*>(base + vlo);
  uint32_t v = threadIdx.x;
  for (; v + (HIST_VEC - 1) * HIST_THREADS < nvec; v += HIST_VEC * HIST_THREADS) {
    uint4 w[HIST_VEC];
#pragma unroll
    for (int u = 0; u < HIST_VEC; u++) w[u] = __ldcs(vk + v + u * HIST_THREADS);
#pragma unroll
    for (int u = 0; u < HIST_VEC; u++) {
      const E* ee = reinterpret_cast<const E*>(&w[u]);
#pragma unroll
      for (int e = 0; e < PER; e++) atomicAdd(&sh_cnt[bucket_of(part_hash<KW, IDENT>(key_of(ee[e])), bf)], 1u);
    }
  }
  for (; v < nvec; v += HIST_THREADS) {
    const uint4 w = __ldcs(vk + v);
    const E* ee = reinterpret_cast<const E*>(&w);
#pragma unroll
    for (int e = 0; e < PER; e++) atomicAdd(&sh_cnt[bucket_of(part_hash<KW, IDENT>(key_of(ee[e])), bf)], 1u);
  }
  __syncthreads();
  const uint32_t row0 = seg * P;
  for (uint32_t p = threadIdx.x; p < P; p += HIST_THREADS) {
    uint32_t c = sh_cnt[p];
    if (hist) hist[(size_t)(row0 + p) * m.cps + j] = c;  // (claiming passes need the totals only)
    if (c) atomicAdd(&rowsum[row0 + p], c);
  }
}

// --------------------------------------------------------------------------
// a6 for both passes in one read of the keys (two-pass plans with
// B1 + B2 <= 16).  The pass-2 histogram is what the paper's "extra scan"
// (P593-597) would re-read from the pass-1 output; here each key's pass-1 and
// pass-2 buckets are counted together, as one JOINT bucket q = b1*P2 + b2:
// a persistent CTA per SM walks chunks (blockIdx.x, +gridDim.x, ...) and
// accumulates 16-bit shared-memory counters, two per 32-bit word (2^16 bins =
// 128 KB).  Wrap-around is handled exactly from the atomic's return value:
//   * the low half of word w counts bin 2w, the high half bin 2w+1;
//   * an increment that finds its half at 0xFFFF wraps it: it adds 65536 to
//     ovf[q] (u32, global);
//   * a wrapping low half also carries 1 into the high half: ovf[q+1] -= 1,
//     and if that carry wrapped the high half too (old word 0xFFFFFFFF),
//     ovf[q+1] += 65536.
// Each wrap is seen by exactly the atomic that causes it, so for every bin
// count = half + ovf (mod 2^32), with no periodic checks.  Row totals go to
// rowsum[b1] (the ovf deltas too), the counters to part[blockIdx.x][Q]
// (coalesced, no atomics); k_joint_reduce turns the partials into both
// passes' bounds and cursors, and both scatters claim their runs (k_scatter
// CLAIM): no per-chunk histograms, no scan over them, one shared-memory
// atomic per key.
// --------------------------------------------------------------------------
constexpr int HJ_THREADS = 1024;
// key vectors per thread and batch, software pipelined (the next batch's
// loads in flight while one is counted): C2 joint histogram 0.273 -> 0.257 ms
// at 4 (2: 0.261, 3: 0.259); 0 = the unpipelined 4-vector batches (A/B)
#ifndef HAPE_HJ_PIPE
#define HAPE_HJ_PIPE 4
#endif
// TMA form: the keys stream through a ring of HJ_NS stages of HJ_SB bytes,
// filled by the last warp with the bulk-copy engine (mbarrier full / empty
// pairs) while 31 warps count -- bytes in flight without registers
constexpr uint32_t HJ_SB = 16384;
constexpr int HJ_NS = 4;
constexpr int HJ_NCW = HJ_THREADS / 32 - 1;  // consumer warps

__host__ __device__ constexpr size_t hj_ring_off(uint32_t QW, uint32_t P1) {
  return ((size_t)(QW + P1) * 4 + 127) / 128 * 128;
}

template <int KW, int PW, bool AOS, bool IDENT, bool TMA = false>
__global__ void __launch_bounds__(HJ_THREADS, 1)
k_hist_joint(PartIn in, SegMap m, uint32_t P1, uint32_t P2, uint32_t* __restrict__ rowsum, uint16_t* __restrict__ part, uint32_t* __restrict__ ovf) {
  extern __shared__ __align__(16) uint32_t sh_hj[];
  using K = typename UW<KW>::T;
  using E = typename std::conditional<AOS, Tup<KW, PW>, K>::type;
  constexpr int ES = sizeof(E);
  constexpr int PER = 16 / ES;
  const uint32_t Q = P1 * P2, QW = Q / 2, WPR = P2 / 2;  // words (2 bins) per row
  uint32_t* j16 = sh_hj;                // [QW] pairs of 16-bit counters, row-major
  uint32_t* rowtot = j16 + QW;          // [P1] row totals
  const E* __restrict__ base = static_cast<const E*>(AOS ? in.t : in.k);
  auto key_of = [](const E& e) -> K {
    if constexpr (AOS) return e.k;
    else return e;
  };
  for (uint32_t i = threadIdx.x; i < QW; i += HJ_THREADS) j16[i] = 0;
  for (uint32_t p = threadIdx.x; p < P1; p += HJ_THREADS) rowtot[p] = 0;
  __syncthreads();
  // joint bucket = b1 * P2 + b2 = the low B1+B2 bits of h (R3:
  // pass 1 reads bits [B2, B2+B1), pass 2 bits [0, B2))
  const uint32_t qmask = Q - 1;
  // wrap test: the half is 0xFFFF iff (old | ~(0xFFFF << sh)) is all ones
  auto wrapped = [](uint32_t q, uint32_t old) -> bool {
    return (old | ~(0xFFFFu << ((q & 1u) << 4))) == 0xFFFFFFFFu;
  };
  auto fixup = [&](uint32_t q, uint32_t old) {  // this increment wrapped its half
    const uint32_t p = q / P2;
    atomicAdd(&ovf[q], 65536u);
    uint32_t dr = 65536u;
    if (!(q & 1u)) {  // the carry went into the neighbour's half
      const uint32_t d = (old >> 16) == 0xFFFFu ? 65535u : 0xFFFFFFFFu;
      atomicAdd(&ovf[q + 1], d);
      dr += d;
    }
    atomicAdd(&rowsum[p], dr);
  };
  auto inc = [&](K k, uint32_t& q) -> uint32_t {
    q = (uint32_t)part_hash<KW, IDENT>(k) & qmask;
    return atomicAdd(&j16[q >> 1], 1u << ((q & 1u) << 4));
  };
  auto count = [&](K k) {
    uint32_t q;
    const uint32_t old = inc(k, q);
    if (wrapped(q, old)) fixup(q, old);
  };
  // the PER keys of one 16-byte vector: all increments issue before any
  // return value is tested (no atomic round trip per key on the warp's
  // critical path), one warp vote per vector guards the rare fix-up
  auto count_vec = [&](const uint4& w) {
    const E* ee = reinterpret_cast<const E*>(&w);
    uint32_t q[PER], old[PER];
#pragma unroll
    for (int e = 0; e < PER; e++) old[e] = inc(key_of(ee[e]), q[e]);
    bool any = false;
#pragma unroll
    for (int e = 0; e < PER; e++) any |= wrapped(q[e], old[e]);
    if (__any_sync(__activemask(), any) && any) {
#pragma unroll
      for (int e = 0; e < PER; e++)
        if (wrapped(q[e], old[e])) fixup(q[e], old[e]);
    }
  };
  const uint32_t nchunks = m.nseg * m.cps;
  auto chunk_of = [&](uint32_t c, uint32_t& lo, uint32_t& vlo, uint32_t& vhi, uint32_t& hi) {
    uint32_t seg, j;
    seg_chunk(m, c, seg, j, lo, hi);
    vlo = lo;
    while (vlo < hi && (reinterpret_cast<uintptr_t>(base + vlo) & 15)) vlo++;
    vhi = vlo + (hi - vlo) / PER * PER;
  };
  if constexpr (!TMA) {
    for (uint32_t c = blockIdx.x; c < nchunks; c += gridDim.x) {
      uint32_t lo, vlo, vhi, hi;
      chunk_of(c, lo, vlo, vhi, hi);
      const uint32_t nvec = (vhi - vlo) / PER;
      for (uint32_t i = lo + threadIdx.x; i < vlo; i += HJ_THREADS) count(key_of(base[i]));
      for (uint32_t i = vhi + threadIdx.x; i < hi; i += HJ_THREADS) count(key_of(base[i]));
      const uint4* __restrict__ vk = reinterpret_cast<const uint4*>(base + vlo);
      uint32_t v = threadIdx.x;
#if HAPE_HJ_PIPE > 0
      // software pipelined: the next batch's loads are in flight while the
      // current batch is counted (A/B build option)
      constexpr int PV = HAPE_HJ_PIPE;
      if (v + (PV - 1) * HJ_THREADS < nvec) {
        uint4 w[PV];
#pragma unroll
        for (int u = 0; u < PV; u++) w[u] = __ldcs(vk + v + u * HJ_THREADS);
        v += PV * HJ_THREADS;
        for (; v + (PV - 1) * HJ_THREADS < nvec; v += PV * HJ_THREADS) {
          uint4 nx[PV];
#pragma unroll
          for (int u = 0; u < PV; u++) nx[u] = __ldcs(vk + v + u * HJ_THREADS);
#pragma unroll
          for (int u = 0; u < PV; u++) count_vec(w[u]);
#pragma unroll
          for (int u = 0; u < PV; u++) w[u] = nx[u];
        }
#pragma unroll
        for (int u = 0; u < PV; u++) count_vec(w[u]);
      }
#else
      for (; v + (HIST_VEC - 1) * HJ_THREADS < nvec; v += HIST_VEC * HJ_THREADS) {
        uint4 w[HIST_VEC];
#pragma unroll
        for (int u = 0; u < HIST_VEC; u++) w[u] = __ldcs(vk + v + u * HJ_THREADS);
#pragma unroll
        for (int u = 0; u < HIST_VEC; u++) count_vec(w[u]);
      }
#endif
      for (; v < nvec; v += HJ_THREADS) count_vec(__ldcs(vk + v));
    }
  } else {
    unsigned char* ring = reinterpret_cast<unsigned char*>(sh_hj) + hj_ring_off(QW, P1);
    uint64_t* full = reinterpret_cast<uint64_t*>(ring + HJ_NS * HJ_SB);
    uint64_t* empty = full + HJ_NS;
    uint32_t* s_len = reinterpret_cast<uint32_t*>(empty + HJ_NS);
    if (threadIdx.x == 0) {
      for (int i = 0; i < HJ_NS; i++) { mbar_init(&full[i], 1); mbar_init(&empty[i], HJ_NCW); }
      asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (warp == HJ_NCW) {
      // producer: every chunk's vector-aligned middle, stage by stage
      if (lane == 0) {
        const uint64_t pol = policy_evict_first();
        uint32_t seq = 0;
        for (uint32_t c = blockIdx.x; c < nchunks; c += gridDim.x) {
          uint32_t lo, vlo, vhi, hi;
          chunk_of(c, lo, vlo, vhi, hi);
          const char* src = reinterpret_cast<const char*>(base + vlo);
          const size_t nb = (size_t)(vhi - vlo) * ES;
          for (size_t off = 0; off < nb; off += HJ_SB, seq++) {
            const uint32_t st = seq % HJ_NS, ph = (seq / HJ_NS) & 1;
            mbar_wait_backoff(&empty[st], ph ^ 1);
            const uint32_t len = (uint32_t)min((size_t)HJ_SB, nb - off);
            s_len[st] = len;
            mbar_expect_tx(&full[st], len);
            bulk_g2s(ring + (size_t)st * HJ_SB, src + off, len, &full[st], pol);
          }
        }
        const uint32_t st = seq % HJ_NS, ph = (seq / HJ_NS) & 1;
        mbar_wait_backoff(&empty[st], ph ^ 1);
        s_len[st] = 0;  // end of the stream
        mbar_arrive(&full[st]);
      }
    } else {
      // consumers: unaligned heads / tails straight from HBM, then the ring
      constexpr uint32_t NCT = HJ_NCW * 32;
      for (uint32_t c = blockIdx.x; c < nchunks; c += gridDim.x) {
        uint32_t lo, vlo, vhi, hi;
        chunk_of(c, lo, vlo, vhi, hi);
        for (uint32_t i = lo + threadIdx.x; i < vlo; i += NCT) count(key_of(base[i]));
        for (uint32_t i = vhi + threadIdx.x; i < hi; i += NCT) count(key_of(base[i]));
      }
      for (uint32_t seq = 0;; seq++) {
        const uint32_t st = seq % HJ_NS, ph = (seq / HJ_NS) & 1;
        mbar_wait(&full[st], ph);
        const uint32_t len = s_len[st];
        if (len == 0) break;
        const uint4* vp = reinterpret_cast<const uint4*>(ring + (size_t)st * HJ_SB);
        const uint32_t nv = len / 16;
        for (uint32_t v = threadIdx.x; v < nv; v += NCT) count_vec(vp[v]);
        __syncwarp();
        if (lane == 0) mbar_arrive(&empty[st]);
      }
    }
  }
  __syncthreads();
  // row totals of the 16-bit counters: a warp covers 32 consecutive words;
  // the lanes of one row differ only in the low log2(min(WPR, 32)) bits
  // (QW is a multiple of 32: Q >= 64)
  const uint32_t rseg = WPR < 32 ? WPR : 32u;
  for (uint32_t w = threadIdx.x; w < QW; w += HJ_THREADS) {
    const uint32_t x = j16[w];
    uint32_t t = (x & 0xFFFFu) + (x >> 16);
    for (uint32_t o = 1; o < rseg; o <<= 1) t += __shfl_xor_sync(0xffffffffu, t, o);
    if (((threadIdx.x & 31) & (rseg - 1)) == 0) atomicAdd(&rowtot[w / WPR], t);
  }
  __syncthreads();
  for (uint32_t p = threadIdx.x; p < P1; p += HJ_THREADS)
    if (rowtot[p]) atomicAdd(&rowsum[p], rowtot[p]);
  uint4* __restrict__ dst = reinterpret_cast<uint4*>(part + (size_t)blockIdx.x * Q);
  const uint4* src = reinterpret_cast<const uint4*>(j16);
  for (uint32_t i = threadIdx.x; i < QW / 4; i += HJ_THREADS) dst[i] = src[i];
}

// Row b1 = blockIdx.x: pass-1 bound = sum of the earlier rows' totals; sum
// the per-CTA joint partials of the row (+ spills), scan its P2 counts and
// emit the pass-2 sub-partition bounds; cursors (claim start points) for
// both passes.  P2/2 words per row; thread groups split the partial index.
constexpr int JR_THREADS = 512;  // (1024 threads, 8 groups per row: measured +0.1 ms per C2 step)

// one relation's joint-reduce arguments; blockIdx.y picks the relation, so
// R's and S's reductions run as one launch
struct JrArgs {
  const uint16_t* part; uint32_t nparts; const uint32_t* ovf; const uint32_t* rowsum;
  uint32_t* bounds1; uint32_t* cursor1; uint32_t* bounds2; uint32_t* cursor2;
};
struct JrArgs2 { JrArgs r[2]; };

__global__ void __launch_bounds__(JR_THREADS)
k_joint_reduce(JrArgs2 args, uint32_t P1, uint32_t P2) {
  const JrArgs& A = args.r[blockIdx.y];
  const uint16_t* __restrict__ part = A.part;
  const uint32_t nparts = A.nparts;
  const uint32_t* __restrict__ ovf = A.ovf;
  const uint32_t* __restrict__ rowsum = A.rowsum;
  uint32_t* __restrict__ bounds1 = A.bounds1;
  uint32_t* __restrict__ cursor1 = A.cursor1;
  uint32_t* __restrict__ bounds2 = A.bounds2;
  uint32_t* __restrict__ cursor2 = A.cursor2;
  __shared__ uint32_t row[4096];
  __shared__ uint32_t wtmp[33];
  __shared__ uint32_t s_b0;
  const uint32_t Q = P1 * P2, p = blockIdx.x, WPR = P2 / 2;
  // pass-1 bound of row p
  uint32_t pre = 0;
  for (uint32_t i = threadIdx.x; i < p; i += JR_THREADS) pre += rowsum[i];
  for (int o = 16; o > 0; o >>= 1) pre += __shfl_xor_sync(0xffffffffu, pre, o);
  if (threadIdx.x == 0) s_b0 = 0;
  for (uint32_t b = threadIdx.x; b < P2; b += JR_THREADS) row[b] = ovf[p * P2 + b];
  __syncthreads();
  if ((threadIdx.x & 31) == 0 && pre) atomicAdd(&s_b0, pre);
  // partial sums: thread (g0, w) adds words w of partials g0, g0+NG, ...
  const uint32_t NG = WPR >= JR_THREADS ? 1u : JR_THREADS / WPR;
  const uint32_t* pw = reinterpret_cast<const uint32_t*>(part);
  for (uint32_t t = threadIdx.x; t < NG * WPR; t += JR_THREADS) {
    const uint32_t w = t % WPR, g0 = t / WPR;
    uint32_t lo = 0, hi = 0;
#pragma unroll 4
    for (uint32_t g = g0; g < nparts; g += NG) {
      const uint32_t x = __ldg(pw + (size_t)g * (Q / 2) + p * WPR + w);
      lo += x & 0xFFFFu;
      hi += x >> 16;
    }
    atomicAdd(&row[2 * w], lo);
    atomicAdd(&row[2 * w + 1], hi);
  }
  __syncthreads();
  block_exscan_smem<JR_THREADS>(row, (int)P2, wtmp);
  const uint32_t b0 = s_b0;
  if (threadIdx.x == 0) { bounds1[p] = b0; cursor1[p] = b0; }
  for (uint32_t b = threadIdx.x; b < P2; b += JR_THREADS) {
    bounds2[p * P2 + b] = b0 + row[b];
    cursor2[p * P2 + b] = b0 + row[b];
  }
  if (p == P1 - 1 && threadIdx.x == 0) {
    const uint32_t n = b0 + rowsum[p];
    bounds1[P1] = n;
    bounds2[Q] = n;
  }
}

// --------------------------------------------------------------------------
// a7: exclusive prefix sum of the histograms -> absolute write offsets (in
// place) and the partition bounds of the pass.  CTA (seg, row-group) scans a
// contiguous tile of rows; the tile's base is the segment start plus the sum
// of earlier rows' totals (rowsum), so no inter-CTA waiting is needed.
// --------------------------------------------------------------------------
constexpr int SCAN_THREADS = 256;
constexpr int SCAN_TILE = 4096;

__global__ void __launch_bounds__(SCAN_THREADS)
k_scan(uint32_t* __restrict__ hist, const uint32_t* __restrict__ rowsum, SegMap m, uint32_t P,
       uint32_t rows_per_cta, uint32_t* __restrict__ bounds_out) {
  __shared__ uint32_t tile[SCAN_TILE];
  __shared__ uint32_t wtmp[33];
  __shared__ uint32_t s_prefix;
  const uint32_t groups = (P + rows_per_cta - 1) / rows_per_cta;
  const uint32_t seg = blockIdx.x / groups, g = blockIdx.x - seg * groups;
  const uint32_t p0 = g * rows_per_cta, p1 = min(P, p0 + rows_per_cta);
  const uint32_t row0 = seg * P;
  // prefix = sum of rowsum over rows [0, p0) of this segment
  uint32_t s = 0;
  for (uint32_t p = threadIdx.x; p < p0; p += SCAN_THREADS) s += rowsum[row0 + p];
  for (int o = 16; o > 0; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
  if (threadIdx.x == 0) s_prefix = 0;
  __syncthreads();
  if ((threadIdx.x & 31) == 0 && s) atomicAdd(&s_prefix, s);
  __syncthreads();
  const uint32_t seg_base = m.bounds ? m.bounds[seg] : 0u;
  uint32_t carry = seg_base + s_prefix;
  const size_t e0 = (size_t)(row0 + p0) * m.cps, e1 = (size_t)(row0 + p1) * m.cps;
  for (size_t c0 = e0; c0 < e1; c0 += SCAN_TILE) {
    const int cn = (int)min((size_t)SCAN_TILE, e1 - c0);
    for (int i = threadIdx.x; i < cn; i += SCAN_THREADS) tile[i] = hist[c0 + i];
    __syncthreads();
    uint32_t tot = block_exscan_strided<SCAN_THREADS, false, false>(tile, (uint32_t)cn, wtmp);
    for (int i = threadIdx.x; i < cn; i += SCAN_THREADS) {
      uint32_t off = carry + tile[i];
      hist[c0 + i] = off;
      size_t e = c0 + i;
      if (e % m.cps == 0) bounds_out[e / m.cps] = off;  // row start = partition bound
    }
    carry += tot;
    __syncthreads();
  }
  if (seg == m.nseg - 1 && g == groups - 1 && threadIdx.x == 0)
    bounds_out[(size_t)m.nseg * P] = m.bounds ? m.bounds[m.nseg] : m.n;
}

// --------------------------------------------------------------------------
// a8/a9: smem-staged, write-combined scatter (Fig. 4, P579-589).
// "we read a chunk of the input (at a time) in the scratchpad and reorganize
// it in such a way that elements belonging to the same output partition are
// located in consecutive scratchpad entries.  Then, we scan the scratchpad and
// write each tuple to its corresponding output partition" (P579-584).
//
// Per tile of T tuples: the bulk-copy engine (cp.async.bulk + mbarrier, a
// STAGES-deep ring) streams the raw tile into shared memory while the previous
// tile is processed; phase 1 ranks each tuple inside its bucket with a
// shared-memory atomic; phase 2 scans the tile's bucket counts and advances
// the per-bucket HBM cursors; phase 3 places every tuple at its bucket run in
// the reordered tile; phase 4 writes the runs with consecutive threads on
// consecutive addresses.  The runs of a bucket continue where the previous
// tile's stopped, so L2 merges partial sectors before they reach HBM.
//
// Odd chunks fill their per-bucket regions back to front: the sector shared
// by the end of region (p, j) and the start of region (p, j+1) is then written
// by both neighbours at the same moment of their lifetimes (both at the start,
// or both at the end), so L2 merges it instead of evicting a half-written
// sector and paying a DRAM read-modify-write.
// --------------------------------------------------------------------------
// The first scatter over the caller's SoA columns stores h(k) in the
// workspace tuples' key field, so every later pass (and the hist / join
// kernels over AoS workspace tuples) reads its buckets straight from it;
// hape.cu launches those with IDENT = true.  0: keys stay raw (A/B only --
// the host side must then launch AoS passes with the configured function).
#ifndef HAPE_STORE_H
#define HAPE_STORE_H 1
#endif
template <int NT_, int ITEMS_, int STAGES_, int MINB_ = 1024 / NT_, bool DST_ = false>
struct ScCfg {
  static constexpr int NT = NT_, ITEMS = ITEMS_, STAGES = STAGES_, T = NT_ * ITEMS_, MINB = MINB_;
  static constexpr bool DST = DST_;  // reorder phase stores each tuple's HBM slot
};

template <int KW, int PW, bool AOS, class C>
struct ScLayout {
  using Tp = Tup<KW, PW>;
  static constexpr int T = C::T;
  // landing buffer per stage: AoS tile, or key column + payload column.  The
  // reordered tile is written back into the same buffer (in place: every
  // tuple is in registers once ranked), so a stage costs T tuples of smem.
  static constexpr size_t RK = AOS ? (size_t)T * sizeof(Tp) + 32 : (size_t)T * KW + 32;
  static constexpr size_t RP = AOS ? 0 : (size_t)T * PW + 32;
  static constexpr size_t RAW0 = (RK + RP + 15) / 16 * 16;
  static constexpr size_t RAW = RAW0 > (size_t)T * sizeof(Tp) ? RAW0 : (size_t)T * sizeof(Tp);
  static __host__ __device__ constexpr size_t bytes(uint32_t P, bool peer = false, bool linked = false) {
    return C::STAGES * RAW + (C::DST ? (size_t)T * 4 : 0) + (size_t)((P + 3) & ~3u) * 16 + 64 * 4 +
           C::STAGES * 8 + 64 + (peer ? (size_t)((P + 1) & ~1u) * 8 : 0) +
           (linked ? (size_t)((P + 3) & ~3u) * 12 : 0);
  }
};

template <int KW, int PW, bool AOS, class C>
__device__ __forceinline__ void sc_issue(const PartIn& in, uint32_t t0, uint32_t tn, unsigned char* raw,
                                         uint64_t* bar, uint64_t pol) {
  using L = ScLayout<KW, PW, AOS, C>;
  uint32_t tx = 0;
  if constexpr (AOS) {
    // expect_tx must precede the copies' completion: compute the size first
    const uintptr_t a = reinterpret_cast<uintptr_t>(static_cast<const Tup<KW, PW>*>(in.t) + t0);
    const uintptr_t a0 = a & ~(uintptr_t)15, a1 = (a + (size_t)tn * sizeof(Tup<KW, PW>) + 15) & ~(uintptr_t)15;
    mbar_expect_tx(bar, (uint32_t)(a1 - a0));
    bulk_g2s_any(raw, static_cast<const Tup<KW, PW>*>(in.t) + t0, (size_t)tn * sizeof(Tup<KW, PW>), bar, pol, &tx);
  } else {
    const uintptr_t ka = reinterpret_cast<uintptr_t>(static_cast<const char*>(in.k) + (size_t)t0 * KW);
    const uintptr_t pa = reinterpret_cast<uintptr_t>(static_cast<const char*>(in.p) + (size_t)t0 * PW);
    const uintptr_t k0 = ka & ~(uintptr_t)15, k1 = (ka + (size_t)tn * KW + 15) & ~(uintptr_t)15;
    const uintptr_t p0 = pa & ~(uintptr_t)15, p1 = (pa + (size_t)tn * PW + 15) & ~(uintptr_t)15;
    mbar_expect_tx(bar, (uint32_t)((k1 - k0) + (p1 - p0)));
    bulk_g2s_any(raw, reinterpret_cast<const void*>(ka), (size_t)tn * KW, bar, pol, &tx);
    bulk_g2s_any(raw + L::RK, reinterpret_cast<const void*>(pa), (size_t)tn * PW, bar, pol, &tx);
  }
}

// CLAIM (pass 2 after k_hist_joint): `offsets` is the per-sub-partition
// cursor array [seg*P + b]; each tile claims its bucket runs with one global
// atomic per non-empty bucket instead of reading per-CTA offsets.  Runs of a
// sub-partition then land in claim order (any order is a valid partition,
// DESIGN.md R9); the claimed regions of concurrently running tiles are
// adjacent, so L2 still merges the partial sectors at their seams.
//
// PEER (the fused device partition + exchange of the G>1 path, SURVEY §8.f
// NEXT-1): bucket b is destination rank b, `peer_out[b]` is that rank's
// receive buffer (a peer pointer over NVLink, or this rank's own buffer) and
// offsets[b] starts at this rank's segment inside it: the runs land in the
// peers' memory straight from the staging tile -- no send buffer, no separate
// transfer.  Every thread fences at system scope before exiting, so the
// stores are visible to the peers once their stream-ordered barrier passes.
//
// LINKED (the paper's single-scan partitioning, P593-597: "we scan the data
// once and write them to a linked list of buffers managed with atomic
// operations"): no histogram precedes the pass.  offsets[b] = lk.cnt[b] is
// the bucket's running tuple count; a claimed run [pos, pos + c) of bucket b
// lives in buffers pos / buf .. (pos + c - 1) / buf of b's chain.  The
// claimant of a run that contains a buffer's first position allocates that
// buffer (one atomic on the pool), publishes it in the directory, and only
// then waits for the buffer its own run starts in, which the earlier
// claimant of that buffer's first position allocates without waiting on
// anything -- so every wait ends.  A run (<= one tile <= buf tuples) spans at
// most two buffers.
template <int KW, int PW, bool AOS, class C, bool IDENT, bool CLAIM = false, bool PEER = false,
          bool LINKED = false>
__global__ void __launch_bounds__(C::NT, C::MINB)
k_scatter(PartIn in, SegMap m, BitField bf, uint32_t P, uint32_t* __restrict__ offsets,
          Tup<KW, PW>* __restrict__ out, Tup<KW, PW>* const* __restrict__ peer_out = nullptr,
          uint32_t agg = 0, LinkMap lk = LinkMap{}) {
  static_assert(!PEER || CLAIM, "peer scatters claim their runs");
  static_assert(!LINKED || (CLAIM && !PEER), "linked scatters claim their runs into local chains");
  using K = typename UW<KW>::T;
  using V = typename UW<PW>::T;
  using Tp = Tup<KW, PW>;
  using L = ScLayout<KW, PW, AOS, C>;
  constexpr int NT = C::NT, T = C::T, ITEMS = C::ITEMS, STAGES = C::STAGES;
  // SoA caller columns hashed here for the last time (HAPE_STORE_H)
  constexpr bool STORE_H = HAPE_STORE_H && !AOS && !IDENT;
  extern __shared__ __align__(128) unsigned char smem[];
  unsigned char* raw = smem;                                            // [STAGES][RAW]
  const uint32_t P4 = (P + 3) & ~3u;                  // keep the arrays below 16-byte aligned
  uint32_t* s_dst = reinterpret_cast<uint32_t*>(smem + STAGES * L::RAW);  // DST only
  uint32_t* s_cnt = s_dst + (C::DST ? T : 0);
  uint32_t* s_st = s_cnt + P4;                        // tile start of the bucket's run
  uint32_t* s_dl = s_st + P4;                         // HBM run start - tile start
  uint32_t* s_cur = s_dl + P4;                        // HBM write cursor per bucket
  uint32_t* s_wt = s_cur + P4;                        // warp totals
  uint64_t* bar = reinterpret_cast<uint64_t*>(s_wt + 64);
  Tup<KW, PW>** s_out = reinterpret_cast<Tup<KW, PW>**>(bar + STAGES + 8);  // PEER: [P] destinations
  uint2* s_dlsp = reinterpret_cast<uint2*>(bar + STAGES + 8);      // LINKED: [P] {run start - tile start, buffer switch}
  uint32_t* s_dl2 = reinterpret_cast<uint32_t*>(s_dlsp + P4);       // LINKED: [P] second buffer's run start - tile start

  uint32_t seg, j, lo, hi;
  if constexpr (CLAIM) seg_chunk_tiles(m, blockIdx.x, (uint32_t)C::T, seg, j, lo, hi);
  else seg_chunk(m, blockIdx.x, seg, j, lo, hi);
  const bool backward = !CLAIM && (j & 1u) != 0;
  const uint32_t row0 = seg * P;
  const size_t nflat = (size_t)m.nseg * P * m.cps;
  const uint32_t ntiles = (hi - lo + T - 1) / T;
  uint64_t pol = 0;
  if (threadIdx.x == 0) {
    pol = policy_evict_first();
    for (int s = 0; s < STAGES; s++) mbar_init(&bar[s], 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    for (uint32_t t = 0; t < (uint32_t)STAGES && t < ntiles; t++) {
      const uint32_t t0 = lo + t * T;
      sc_issue<KW, PW, AOS, C>(in, t0, min((uint32_t)T, hi - t0), raw + t * L::RAW, &bar[t], pol);
    }
  }
  for (uint32_t p = threadIdx.x; p < P; p += NT) {
    if constexpr (!CLAIM) {
      const size_t f = (size_t)(row0 + p) * m.cps + j;
      s_cur[p] = backward ? (f + 1 < nflat ? offsets[f + 1] : m.n) : offsets[f];
    }
    if constexpr (PEER) s_out[p] = peer_out[p];
    s_cnt[p] = 0;
  }
  __syncthreads();

  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  for (uint32_t t = 0; t < ntiles; t++) {
    const uint32_t s = t % STAGES, ph = (t / STAGES) & 1;
    const uint32_t t0 = lo + t * T, tn = min((uint32_t)T, hi - t0);
    unsigned char* rb = raw + s * L::RAW;
    Tp* s_tile = reinterpret_cast<Tp*>(rb);            // reordered tile (in place)
    const K* tk;
    const V* tp;
    const Tp* tt;
    if constexpr (AOS) {
      tt = reinterpret_cast<const Tp*>(rb + (reinterpret_cast<uintptr_t>(static_cast<const Tp*>(in.t) + t0) & 15));
    } else {
      tk = reinterpret_cast<const K*>(rb + ((reinterpret_cast<uintptr_t>(in.k) + (uintptr_t)t0 * KW) & 15));
      tp = reinterpret_cast<const V*>(rb + L::RK + ((reinterpret_cast<uintptr_t>(in.p) + (uintptr_t)t0 * PW) & 15));
    }
    auto load = [&](uint32_t i) -> Tp {
      if constexpr (AOS) return tt[i];
      else { Tp x; x.k = tk[i]; x.v = tp[i]; return x; }
    };
    mbar_wait(&bar[s], ph);
    // phase 1: bucket + rank (shared-memory atomic claim); tuples -> registers
    // (STORE_H: the tuple keeps h(k) in its key field from here on -- h is a
    // bijection, so later passes take their buckets from the stored value and
    // the join compares h(k) for k; keys never leave the workspace)
    auto hb = [&](Tp& t) -> uint32_t {
      const uint64_t hv = part_hash<KW, IDENT>(t.k);
      if constexpr (STORE_H) t.k = (K)hv;
      return bucket_of(hv, bf);
    };
    Tp x[ITEMS];
    uint32_t br[ITEMS];
    const bool full = tn == (uint32_t)T;
    // agg (skewed inputs): lanes of a warp that share a bucket rank through
    // one leader atomic (__match_any_sync) instead of
    // serialising on the same shared-memory word
    // agg == 2 (hot-bucket form): the lanes whose bucket equals lane 0's
    // rank through lane 0's one atomic (one shuffle + one ballot per tuple);
    // a skewed tile's hot bucket holds lane 0 most of the time
    auto rank_hot = [&](uint32_t b) -> uint32_t {
      const uint32_t b0 = __shfl_sync(0xffffffffu, b, 0);
      const uint32_t m = __ballot_sync(0xffffffffu, b == b0);
      if (__popc(m) < 4) return atomicAdd(&s_cnt[b], 1u);
      uint32_t base = 0;
      if (lane == 0) base = atomicAdd(&s_cnt[b0], (uint32_t)__popc(m));
      base = __shfl_sync(0xffffffffu, base, 0);
      return b == b0 ? base + (uint32_t)__popc(m & ((1u << lane) - 1u)) : atomicAdd(&s_cnt[b], 1u);
    };
    auto rank_agg = [&](uint32_t b, uint32_t mask) -> uint32_t {
      const uint32_t peers = __match_any_sync(mask, b);
      const int leader = __ffs(peers) - 1;
      uint32_t base = 0;
      if (lane == leader) base = atomicAdd(&s_cnt[b], (uint32_t)__popc(peers));
      base = __shfl_sync(peers, base, leader);
      return base + (uint32_t)__popc(peers & ((1u << lane) - 1u));
    };
    if (full) {
#pragma unroll
      for (int u = 0; u < ITEMS; u++) x[u] = load(u * NT + threadIdx.x);
      if (agg == 1) {
#pragma unroll
        for (int u = 0; u < ITEMS; u++) {
          const uint32_t b = hb(x[u]);
          br[u] = (b << 16) | rank_agg(b, 0xffffffffu);
        }
      } else if (agg == 2) {
#pragma unroll
        for (int u = 0; u < ITEMS; u++) {
          const uint32_t b = hb(x[u]);
          br[u] = (b << 16) | rank_hot(b);
        }
      } else {
#pragma unroll
        for (int u = 0; u < ITEMS; u++) {
          const uint32_t b = hb(x[u]);
          br[u] = (b << 16) | atomicAdd(&s_cnt[b], 1u);
        }
      }
    } else {
#pragma unroll
      for (int u = 0; u < ITEMS; u++) {
        const uint32_t i = u * NT + threadIdx.x;
        const uint32_t vm = __ballot_sync(0xffffffffu, i < tn);
        if (i < tn) {
          x[u] = load(i);
          const uint32_t b = hb(x[u]);
          br[u] = (b << 16) | (agg == 1 ? rank_agg(b, vm) : atomicAdd(&s_cnt[b], 1u));
        }
      }
    }
    __syncthreads();  // A: counts complete; the whole tile is in registers
    // the previous tile's buffer is now free (its write-out finished before A)
    if (threadIdx.x == 0 && t >= 1 && t - 1 + STAGES < ntiles) {
      const uint32_t n0 = lo + (t - 1 + STAGES) * T;
      sc_issue<KW, PW, AOS, C>(in, n0, min((uint32_t)T, hi - n0), raw + ((t - 1) % STAGES) * L::RAW,
                               &bar[(t - 1) % STAGES], pol);
    }
    // phase 2: exclusive scan of the tile's bucket counts; advance the cursors
    // (storing the claimed run starts only after phase 3, so the claim's round
    // trip overlaps the reorder, measured slower: C2 0.936 -> 0.943, C4 18.75
    // -> 19.03 ms -- the other resident CTA already covers it)
    {
      const uint32_t per = (P + NT - 1) / NT;
      const uint32_t b0 = min(threadIdx.x * per, P), b1 = min(b0 + per, P);
      uint32_t sum = 0;
      for (uint32_t b = b0; b < b1; b++) sum += s_cnt[b];
      // CLAIM with one bucket per thread: issue the claim now so its latency
      // overlaps the scan and barrier X
      uint32_t claim0 = 0;
      if constexpr (CLAIM)
        if (b1 == b0 + 1 && sum) claim0 = atomicAdd(&offsets[row0 + b0], sum);
      const uint32_t inc = warp_incl_scan(sum);
      if (lane == 31) s_wt[warp] = inc;
      __syncthreads();  // X
      // warps past the last bucket have nothing to place (warp-uniform skip);
      // the others add the totals of the warps before them (one load + a
      // shuffle scan instead of a loop over the earlier warps)
      if (warp * 32 * per < P) {
        constexpr int NW = NT / 32;
        const uint32_t wt = lane < NW ? s_wt[lane] : 0u;
        const uint32_t wpre = warp_incl_scan(wt);
        const uint32_t before = __shfl_sync(0xffffffffu, wpre, (warp + 31) & 31);
        uint32_t ex = inc - sum + (warp ? before : 0u);
        for (uint32_t b = b0; b < b1; b++) {
        const uint32_t c = s_cnt[b];
        uint32_t run;
        if constexpr (CLAIM) {
          run = b1 == b0 + 1 ? claim0 : (c ? atomicAdd(&offsets[row0 + b], c) : 0u);
        } else {
          const uint32_t cur = s_cur[b];
          run = backward ? cur - c : cur;
          s_cur[b] = backward ? cur - c : cur + c;
        }
          s_st[b] = ex;
          s_dl[b] = run - ex;
          if constexpr (LINKED) {
            if (c) {
              const uint32_t B = lk.buf;
              const uint32_t k0 = run / B, k1 = (run + c - 1) / B;
              uint32_t* drow = lk.dir + (size_t)b * lk.kmax;
              // the buffers whose first position lies in this run are ours to allocate
              for (uint32_t k = k0; k <= k1; k++) {
                if (k * B < run) continue;
                const uint32_t id = atomicAdd(lk.pool, 1u);
                lk.owner[id] = b;
                lk.kidx[id] = k;
                __threadfence();
                atomicExch(drow + k, id + 1u);
              }
              auto wait_id = [&](uint32_t k) -> uint32_t {
                uint32_t v;
                while ((v = *reinterpret_cast<volatile uint32_t*>(drow + k)) == 0u) __nanosleep(64);
                return v - 1u;
              };
              const uint32_t id0 = wait_id(k0), id1 = k1 != k0 ? wait_id(k1) : id0;
              s_dlsp[b] = make_uint2(id0 * B - k0 * B + run - ex, (k0 + 1) * B - run + ex);
              s_dl2[b] = id1 * B - k1 * B + run - ex;
            }
          }
          s_cnt[b] = 0;
          ex += c;
        }
      }
    }
    __syncthreads();  // B: run starts known
    // phase 3: reorder the tile in shared memory (in place), bucket runs consecutive
    if (full) {
      // all run-start loads first, then the stores: the compiler cannot tell
      // s_tile from s_st apart, so interleaving them serialises on LDS latency
      uint32_t pos[ITEMS];
#pragma unroll
      for (int u = 0; u < ITEMS; u++) pos[u] = s_st[br[u] >> 16] + (br[u] & 0xFFFFu);
      if constexpr (C::DST) {
        uint32_t dl[ITEMS];
#pragma unroll
        for (int u = 0; u < ITEMS; u++) dl[u] = s_dl[br[u] >> 16];
#pragma unroll
        for (int u = 0; u < ITEMS; u++) s_dst[pos[u]] = dl[u] + pos[u];
      }
#pragma unroll
      for (int u = 0; u < ITEMS; u++) s_tile[pos[u]] = x[u];
    } else {
#pragma unroll
      for (int u = 0; u < ITEMS; u++)
        if (u * NT + threadIdx.x < tn) {
          const uint32_t pos = s_st[br[u] >> 16] + (br[u] & 0xFFFFu);
          s_tile[pos] = x[u];
          if constexpr (C::DST) s_dst[pos] = s_dl[br[u] >> 16] + pos;
        }
    }
    // generic-proxy writes to a buffer the bulk-copy engine refills later
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    __syncthreads();  // C: the reordered tile is complete
    // phase 4: write the runs; consecutive threads -> consecutive addresses
    // (the bucket is taken again from the tuple's h(k) -- stored in phase 1,
    // STORE_H -- which is cheaper than another random shared-memory store +
    // load)
    auto dst_of = [&](uint32_t i, const Tp& y) -> uint32_t {
      if constexpr (C::DST) return s_dst[i];
      else if constexpr (LINKED) {
        // one 8-byte load; the second buffer's start only for the rare
        // tuples past a buffer boundary
        const uint32_t b = bucket_of(part_hash<KW, IDENT || STORE_H>(y.k), bf);
        const uint2 v = s_dlsp[b];
        return (i < v.y ? v.x : s_dl2[b]) + i;
      } else return s_dl[bucket_of(part_hash<KW, IDENT || STORE_H>(y.k), bf)] + i;
    };
    if constexpr (PEER) {
      auto put = [&](uint32_t i) {
        const Tp y = s_tile[i];
        const uint32_t b = bucket_of(part_hash<KW, IDENT || STORE_H>(y.k), bf);
        s_out[b][s_dl[b] + i] = y;
      };
      if (full) {
#pragma unroll
        for (int u = 0; u < ITEMS; u++) put(u * NT + threadIdx.x);
      } else {
        for (uint32_t i = threadIdx.x; i < tn; i += NT) put(i);
      }
    } else if (full) {
#pragma unroll
      for (int u = 0; u < ITEMS; u++) {
        const uint32_t i = u * NT + threadIdx.x;
        const Tp y = s_tile[i];
        out[dst_of(i, y)] = y;
      }
    } else {
      for (uint32_t i = threadIdx.x; i < tn; i += NT) {
        const Tp y = s_tile[i];
        out[dst_of(i, y)] = y;
      }
    }
  }
  if constexpr (PEER) __threadfence_system();
}

// --------------------------------------------------------------------------
// a10: co-partition work list.  Item = (partition q, S-slice index); one item
// per probe_slice S tuples of a non-empty co-partition (skewed S partitions
// are split across CTAs; R partitions larger than the smem build capacity
// are chunked inside the item).  Zip of co-partitions, P740-747; one
// co-partition per thread block, P804-806.
// --------------------------------------------------------------------------
constexpr int WL_THREADS = 1024;

__global__ void __launch_bounds__(WL_THREADS)
k_worklist(const uint32_t* __restrict__ bR, const uint32_t* __restrict__ bS, uint32_t Q,
           uint32_t slice, uint2* __restrict__ items, uint32_t* __restrict__ n_items) {
  __shared__ uint32_t sc[WL_THREADS];
  __shared__ uint32_t wtmp[33];
  __shared__ uint32_t s_base;
  const uint32_t q = blockIdx.x * WL_THREADS + threadIdx.x;
  uint32_t k = 0;
  if (q < Q) {
    const uint32_t nr = bR[q + 1] - bR[q], ns = bS[q + 1] - bS[q];
    k = (nr && ns) ? (ns + slice - 1) / slice : 0u;
  }
  sc[threadIdx.x] = k;
  __syncthreads();
  const uint32_t tot = block_exscan_smem<WL_THREADS>(sc, WL_THREADS, wtmp);
  if (threadIdx.x == 0) s_base = tot ? atomicAdd(n_items, tot) : 0u;
  __syncthreads();
  const uint32_t base = s_base + sc[threadIdx.x];
  for (uint32_t t = 0; t < k; t++) items[base + t] = make_uint2(q, t);
}

// --------------------------------------------------------------------------
// a11-a13: per-co-partition build + probe with the hash table in shared
// memory (Fig. 3, P535-541, P806-810), aggregation fused (P789-793),
// optional materialisation through a block-aggregated output claim
// ("Buffer output ... ATOMICS!", Fig. 3 P488-493).
//
// Warp-specialised pipeline (the Blackwell producer/consumer idiom):
//   * a producer warp walks this CTA's static share of the work list
//     (items blockIdx.x, +gridDim.x, ...; co-partitions are near-uniform, so a
//     static split balances), reads the item's bounds and streams each R chunk
//     into a 2-deep ring of shared-memory buffers with the bulk-copy engine
//     (cp.async.bulk + mbarrier), one "stage" per (R chunk, S slice);
//   * 8 consumer warps build a chained table over the landed chunk (heads
//     reset per stage, atomicExch on the heads, u16 next links) and probe the
//     S slice, streaming S tuples from HBM, JN_U independent loads per thread.
// The next stage's R chunk lands while the current one is probed.
//
// The slot of a key inside the smem table is a multiplicative hash of the key
// (2 instructions) rather than more bits of the partition hash: every tuple of
// a co-partition shares the partition bits, and any function of the key that
// spreads them works -- the result does not depend on it.  For each S tuple
// the chain is walked to its end (bag semantics); the aggregation body of a
// match runs with the lanes converged, once per round.
// --------------------------------------------------------------------------
// consumer threads per build+probe CTA: a template parameter (JN_CONSUMERS,
// 256 or 512) of the kernel; one producer warp on top
// S tuples per consumer thread per batch of the direct form (C2 build+probe
// with the pipelined tail: U = 1 / 2 / 3 / 4 -> 0.692 / 0.649 / 0.640 /
// 0.654 ms; C4 10.05 -> 9.92, C5 3.89 -> 3.80 ms at 3)
#ifndef HAPE_JN_U
#define HAPE_JN_U 3
#endif
constexpr int JN_U = HAPE_JN_U;
#ifndef HAPE_JN_PTAIL
#define HAPE_JN_PTAIL 1
#endif

#ifndef HAPE_JN_REL_MODE
#define HAPE_JN_REL_MODE 0
#endif
// SR tile release after the consumers' copy to registers: 0 = per-warp
// __syncwarp + lane-0 arrival on the tile's empty barrier (16 arrivals: the
// producer/consumer pattern of TMA pipelines -- the warp's reads are ordered
// before the release arrive, the producer's acquire wait before its refill;
// C3 build+probe 10.13-10.22 -> 9.84-9.88 ms, round 2 default); 1 = one
// consumer barrier, then one arrival (the form racecheck could verify, the
// default while compute-sanitizer ran on this pool).  Releasing at the
// materialising probe's claim barrier instead measured 14.4 ms (the refill
// starts a whole probe later), and a runtime switch between the forms slowed
// every form to ~14 ms (a barrier under a runtime branch), so the form is a
// compile-time choice.
constexpr int JN_REL = HAPE_JN_REL_MODE;
constexpr uint32_t JN_MAXCAP = 16384;
constexpr uint32_t JN_NIL = 0xFFFFu;
constexpr uint32_t JN_STOP = 0xFFFFFFFFu;
// chain heads: 32-bit words (16-bit heads need a CAS-loop insert: measured
// C2 build+probe 0.73 -> 0.93 ms, C3 -2%)
using JnHead = uint32_t;


template <int KW, int PRW>
__host__ __device__ constexpr size_t join_ring_bytes(uint32_t cap) {
  return ((size_t)cap * sizeof(Tup<KW, PRW>) + 32 + 15) / 16 * 16;
}
// staged S tile: SU tuples per consumer thread
template <int KW, int PSW, int SU, int NC = 256>
__host__ __device__ constexpr size_t join_stile_bytes() {
  return ((size_t)SU * NC * sizeof(Tup<KW, PSW>) + 32 + 15) / 16 * 16;
}
// nrb R-chunk buffers, nsb staged S tiles of SU*256 tuples (SU = 0: S read
// straight from HBM)
// Table layouts (LAY):
//   JN_AOS (0): chains over the landed AoS R tuples, a u16 next[] beside them;
//   JN_KN  (1): key|next nodes -- the build moves each R payload to pay[] and
//               stores the chain link in the tuple's payload field, so a chain
//               hop is one shared load of {key, next};
//   JN_SK  (2): the build also copies the keys to a dense keys[] array: a key
//               load spreads over all 32 banks (a key inside 8-byte AoS tuples
//               only reaches the 16 even ones); payloads stay in the tuples
constexpr int JN_AOS = 0, JN_KN = 1, JN_SK = 2;
template <int KW, int PRW>
__host__ __device__ constexpr size_t join_link_bytes(uint32_t cap, int lay) {
  return lay == JN_KN ? ((size_t)cap * PRW + 15) / 16 * 16
                      : ((size_t)cap * 2 + 15) / 16 * 16 + (lay == JN_SK ? ((size_t)cap * KW + 15) / 16 * 16 : 0);
}
template <int KW, int PRW, int PSW, int SU = 0, int NC = 256, int LAY = JN_AOS>
__host__ __device__ constexpr size_t join_smem_bytes(uint32_t cap, uint32_t slot_bits, uint32_t nrb = 2,
                                                     uint32_t nsb = 0) {
  return nrb * join_ring_bytes<KW, PRW>(cap)                               // R ring
         + (SU ? nsb * join_stile_bytes<KW, PSW, SU, NC>() : 0)           // S ring
         + join_link_bytes<KW, PRW>(cap, LAY)                              // next[] / pay[] / keys[]
         + (sizeof(JnHead) << slot_bits);                                  // heads[]
}

struct JoinArgs {
  const void* rt; const void* st;            // R / S tuples (AoS workspace)
  const uint32_t* bR; const uint32_t* bS;
  const uint2* items; const uint32_t* n_items;
  uint32_t cap; uint32_t slice; uint32_t slot_bits;
  unsigned long long* acc;                   // [4] count, sum_r, sum_s, checksum
  void* out_r; void* out_s; unsigned long long out_cap; unsigned long long* out_ctr;
  uint32_t dbg;                              // timing experiments only (HAPE_JN_DBG); 0 in production
  uint32_t r_unique;                         // caller guarantees unique R keys (HAPE_FLAG_R_UNIQUE)
  uint32_t pf_bytes;                         // L2 prefetch window at the head of each S slice (0 = off)
  uint32_t nrb;                              // R-chunk ring buffers (1 or 2)
  uint32_t nsb;                              // SR kernels: staged S tiles in the ring (>= 2)
  uint32_t qmask;                            // co-partitions - 1: q = h(key) & qmask (k_join_oa)
  uint32_t ep_period;                        // chain-head epochs before a head reset (<= 65535)
  uint32_t probe_heavy;                      // host-side shape hint: |S| >= 2|R| (kernels ignore it)
};

struct JnStage {
  uint32_t nr;      // R tuples in the chunk (JN_STOP = no more stages)
  uint32_t off;     // byte offset of tuple 0 inside the ring buffer
  uint32_t s_lo, s_hi;
};

// slot and mbarrier phase of the seq-th use of an n-deep ring (n is 1 or 2
// on the hot paths: no integer division per stage)
__device__ __forceinline__ void ring_pos(uint32_t seq, uint32_t n, uint32_t& slot, uint32_t& phase) {
  if (n == 1) { slot = 0; phase = seq & 1u; }
  else if (n == 2) { slot = seq & 1u; phase = (seq >> 1) & 1u; }
  else { slot = seq % n; phase = (seq / n) & 1u; }
}

template <int NC>
__device__ __forceinline__ void consumer_sync() {
  asm volatile("bar.sync 1, %0;" ::"n"(NC) : "memory");
}

// slot of a key in the smem table: top slot_bits bits of key * odd constant
template <int KW>
__device__ __forceinline__ uint32_t jn_slot(typename UW<KW>::T k, uint32_t sbits) {
  if constexpr (KW == 4) return (uint32_t)(k * 0x9E3779B1u) >> (32 - sbits);
  else return (uint32_t)((k * 0x9E3779B97F4A7C15ull) >> (64 - sbits));
}

struct JnAcc {
  unsigned long long cnt = 0, sr = 0, ss = 0, sx = 0;
};

template <int KW, int PRW, int LAY = JN_AOS>
struct JnTable {
  using K = typename UW<KW>::T;
  using V = typename UW<PRW>::T;
  const Tup<KW, PRW>* r;    // R chunk (ring buffer); JN_KN: {key, next} nodes
  const void* link;         // next[] (u16), or JN_KN: pay[] (the R payloads)
  const K* keys;            // JN_SK: dense keys[]
  const JnHead* head;
  uint32_t sbits;
  bool dup;                 // the chunk holds some key twice (bag semantics path)
  uint32_t ep;              // stage epoch: a head is valid iff its high half == ep
  // does entry e hold key k?  (loads y = r[e] where the layout keeps the
  // key in the tuple)
  __device__ __forceinline__ bool hit(uint32_t e, K k, Tup<KW, PRW>& y) const {
    if constexpr (LAY == JN_SK) return keys[e] == k;
    else { y = r[e]; return y.k == k; }
  }
  // chain successor of e (y as loaded by hit(e))
  __device__ __forceinline__ uint32_t next_of(uint32_t e, const Tup<KW, PRW>& y) const {
    if constexpr (LAY == JN_KN) return (uint32_t)y.v;
    else return static_cast<const uint16_t*>(link)[e];
  }
  __device__ __forceinline__ uint32_t next_at(uint32_t e) const {
    if constexpr (LAY == JN_KN) return (uint32_t)r[e].v;
    else return static_cast<const uint16_t*>(link)[e];
  }
  __device__ __forceinline__ K key_at(uint32_t e) const {
    if constexpr (LAY == JN_SK) return keys[e];
    else return r[e].k;
  }
  // R payload of e (y as loaded by hit(e))
  __device__ __forceinline__ V pay_of(uint32_t e, const Tup<KW, PRW>& y) const {
    if constexpr (LAY == JN_KN) return static_cast<const V*>(link)[e];
    else if constexpr (LAY == JN_SK) return r[e].v;
    else return y.v;
  }
  __device__ __forceinline__ V pay_at(uint32_t e) const {
    if constexpr (LAY == JN_KN) return static_cast<const V*>(link)[e];
    else return r[e].v;
  }
};

// chain head of a slot: (epoch << 16) | tuple index; a head written in an
// earlier stage (other epoch) reads as an empty chain, so the heads are never
// reset between stages
__device__ __forceinline__ uint32_t jn_head(JnHead hv, uint32_t ep) {
  // heads of earlier epochs (and the zeroed epoch 0) are smaller than
  // ep << 16, so the difference wraps above 0xFFFF: one subtract and one
  // unsigned min instead of a shift, compare, mask and select
  return min(hv - (ep << 16), 0xFFFFu);
}

// Load U S tuples per consumer thread: j = base + u*256 + tid.  (Two
// neighbouring tuples per 16-byte load measured neutral: C2 0.706 ms both,
// profiles/r2/ab_build_probe_pair.jsonl)
template <int KW, int PSW, int U, int JN_CONSUMERS>
__device__ __forceinline__ void jn_load_batch(const JoinArgs& a, uint32_t base, uint32_t s_hi, Tup<KW, PSW> (&x)[U]) {
  const Tup<KW, PSW>* __restrict__ sT = static_cast<const Tup<KW, PSW>*>(a.st);
#pragma unroll
  for (int u = 0; u < U; u++) {
    const uint32_t j = base + u * JN_CONSUMERS + threadIdx.x;
    if (j < s_hi) x[u] = ldcs_tup(sT + j);
  }
}

// Probe the U S tuples x[] (loaded by jn_load_batch for the same base).
template <int KW, int PRW, int PSW, bool MAT, int U, int JN_CONSUMERS, int LAY>
__device__ __forceinline__ void jn_probe_batch(const JnTable<KW, PRW, LAY>& t, const JoinArgs& a, uint32_t base,
                                               uint32_t s_hi, const Tup<KW, PSW> (&x)[U], JnAcc& acc,
                                               uint32_t* s_wsum, unsigned long long* s_wbase) {
  using PR = typename UW<PRW>::S;
  using PS = typename UW<PSW>::S;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint32_t e0[U];
#pragma unroll
  for (int u = 0; u < U; u++) {
    const uint32_t j = base + u * JN_CONSUMERS + threadIdx.x;
    e0[u] = j < s_hi ? jn_head(t.head[jn_slot<KW>(x[u].k, t.sbits)], t.ep) : JN_NIL;
  }
  uint32_t c[U], m[U];
#pragma unroll
  for (int u = 0; u < U; u++) {
    // walk to the next match (divergent, cheap), then run the aggregation
    // body once per round with every lane that found one (converged).  A
    // chunk without duplicate keys has at most one match per S tuple, so the
    // walk stops at the first match.
    c[u] = 0;
    m[u] = JN_NIL;
    uint32_t e = e0[u];
    if (!t.dup) {
      // unique build side: walk to the first equal key (one 8/16-byte shared
      // load per visited tuple gives key and payload), aggregate once
      Tup<KW, PRW> y;
      while (e != JN_NIL) {
        if (t.hit(e, x[u].k, y)) break;
        e = t.next_of(e, y);
      }
      // reconverge before the aggregation body: without it the compiler
      // ran the body of the KN / SK layouts once per group of lanes leaving
      // the walk together (the 37-instruction body 2.7x per warp round: 1.03
      // vs 0.75 ms); the AoS walk reconverges by itself and is faster
      // without the explicit barrier (0.718 vs 0.750 ms)
      if constexpr (LAY != JN_AOS) __syncwarp();
      if (e != JN_NIL) {
        const int64_t pr = (int64_t)(PR)t.pay_of(e, y), ps = (int64_t)(PS)x[u].v;
        if (MAT) m[u] = e;
        c[u] = 1;
        acc.sr += (unsigned long long)pr;
        acc.ss += (unsigned long long)ps;
        acc.sx += pair_mix(pr, ps);
      }
    } else {
      while (true) {
        Tup<KW, PRW> y;
        while (e != JN_NIL) {
          if (t.hit(e, x[u].k, y)) break;
          e = t.next_of(e, y);
        }
        const bool hit = e != JN_NIL;
        if (!__any_sync(0xffffffffu, hit)) break;
        if (hit) {
          const int64_t pr = (int64_t)(PR)t.pay_of(e, y), ps = (int64_t)(PS)x[u].v;
          if (MAT && c[u] == 0) m[u] = e;
          c[u]++;
          acc.sr += (unsigned long long)pr;
          acc.ss += (unsigned long long)ps;
          acc.sx += pair_mix(pr, ps);
          e = t.next_of(e, y);
        }
      }
    }
    acc.cnt += c[u];
  }
  if constexpr (MAT) {
    // positions in (u-major, lane-minor) order inside the warp, warps in order
    // inside the block, one global claim per block per batch.  With a unique
    // build side every count is 0/1: a ballot gives the positions and the
    // recorded match is written without walking the chain again.
    uint32_t incl[U], before[U], wtot = 0;
    if (!t.dup) {
      const uint32_t lt = (1u << lane) - 1u;
#pragma unroll
      for (int u = 0; u < U; u++) {
        const uint32_t mk = __ballot_sync(0xffffffffu, c[u] != 0);
        before[u] = wtot;
        incl[u] = __popc(mk & lt) + c[u];
        wtot += __popc(mk);
      }
    } else {
#pragma unroll
      for (int u = 0; u < U; u++) {
        incl[u] = warp_incl_scan(c[u]);
        before[u] = wtot;
        wtot += __shfl_sync(0xffffffffu, incl[u], 31);
      }
    }
    if (lane == 0) s_wsum[warp] = wtot;
    consumer_sync<JN_CONSUMERS>();
    if (warp == 0) {
      const uint32_t v = lane < JN_CONSUMERS / 32 ? s_wsum[lane] : 0u;
      const uint32_t inc = warp_incl_scan(v);
      const uint32_t tot = __shfl_sync(0xffffffffu, inc, 31);
      unsigned long long g = 0;
      if (lane == 0 && tot) g = atomicAdd(a.out_ctr, (unsigned long long)tot);
      g = __shfl_sync(0xffffffffu, g, 0);
      if (lane < JN_CONSUMERS / 32) s_wbase[lane] = g + inc - v;
    }
    consumer_sync<JN_CONSUMERS>();
    const unsigned long long wb = s_wbase[warp];
    if (!t.dup) {
#pragma unroll
      for (int u = 0; u < U; u++) {
        if (!c[u]) continue;
        const unsigned long long pos = wb + before[u] + incl[u] - 1;
        if (pos < a.out_cap) {
          static_cast<PR*>(a.out_r)[pos] = (PR)t.pay_at(m[u]);
          static_cast<PS*>(a.out_s)[pos] = (PS)x[u].v;
        }
      }
      return;
    }
#pragma unroll
    for (int u = 0; u < U; u++) {
      if (!c[u]) continue;
      unsigned long long pos = wb + before[u] + incl[u] - c[u];
      for (uint32_t e = e0[u]; e != JN_NIL; e = t.next_at(e)) {
        if (t.key_at(e) == x[u].k) {
          if (pos < a.out_cap) {
            static_cast<PR*>(a.out_r)[pos] = (PR)t.pay_at(e);
            static_cast<PS*>(a.out_s)[pos] = (PS)x[u].v;
          }
          pos++;
        }
      }
    }
  }
}

// SU > 0: the producer warp also stages the S slice through an nsb-deep
// ring of SU*256-tuple tiles (bulk copies, mbarrier full/empty pairs; each
// consumer warp releases a tile once its tuples are in registers), so the
// consumers never wait on HBM latency -- the form for materialising and
// 16-byte-tuple joins, whose probe cannot keep a software-pipelined S batch
// in registers.
// (HAPE_JN_MINB / HAPE_JN_SR_MINB: CTAs per SM the direct / staged-S forms
// are register-budgeted for; A/B builds)
#ifndef HAPE_JN_MINB
// the direct form (8-byte S tuples, no pairs) at 4 CTAs per SM: <= 56
// registers, no spills; unbounded it took 63 (3 CTAs per SM: C2 0.78 vs 0.74 ms).
// 5 CTAs per SM compiles to 40 registers without spills since the batch
// changes, but measured no faster (C2 0.638 vs 0.633 ms, bag 0.910 vs 0.841)
#define HAPE_JN_MINB 4
#endif
#ifndef HAPE_JN_SR_MINB
// the staged-S form needs 2 CTAs per SM: unbounded it took 72 registers (one
// 544-thread CTA per SM, 36 % barrier stalls): C3 build+probe 15.3 vs 10.6 ms
#define HAPE_JN_SR_MINB 2
#endif
template <int KW, int PRW, int PSW, bool MAT, int SU, int JN_CONSUMERS = 256, int LAY = JN_AOS>
__global__ void __launch_bounds__(JN_CONSUMERS + 32,
                                  SU == 0 ? ((KW + PSW <= 8 && !MAT) ? (JN_CONSUMERS == 256 ? HAPE_JN_MINB : 2) : 1)
                                          : HAPE_JN_SR_MINB)
k_build_probe(JoinArgs a) {
  constexpr int JN_THREADS = JN_CONSUMERS + 32;
  constexpr bool SR = SU > 0;
  constexpr uint32_t JN_STILE = (uint32_t)(SR ? SU : 1) * JN_CONSUMERS;
  using TR = Tup<KW, PRW>;
  using TS = Tup<KW, PSW>;
  extern __shared__ __align__(128) unsigned char smem[];
  const uint32_t RB = (uint32_t)join_ring_bytes<KW, PRW>(a.cap);
  constexpr uint32_t SB = SR ? (uint32_t)join_stile_bytes<KW, PSW, SR ? SU : 1, JN_CONSUMERS>() : 0u;
  const uint32_t NRB = a.nrb, NSB = SR ? a.nsb : 0u;
  unsigned char* ring = smem;                                           // [NRB][RB]
  unsigned char* sring = smem + NRB * RB;                               // [NSB][SB]
  constexpr bool KN = LAY == JN_KN;
  using K = typename UW<KW>::T;
  uint16_t* s_next = reinterpret_cast<uint16_t*>(sring + NSB * SB);               // JN_AOS / JN_SK
  typename UW<PRW>::T* s_pay = reinterpret_cast<typename UW<PRW>::T*>(sring + NSB * SB);  // JN_KN
  K* s_keys = reinterpret_cast<K*>(sring + NSB * SB + ((size_t)a.cap * 2 + 15) / 16 * 16);  // JN_SK
  JnHead* s_head = reinterpret_cast<JnHead*>(sring + NSB * SB + join_link_bytes<KW, PRW>(a.cap, LAY));
  constexpr int MAXS = 8;
  __shared__ JnStage s_meta[2];
  __shared__ uint32_t s_soff[MAXS];
  __shared__ __align__(8) uint64_t full[2], empty[2], sfull[MAXS], sempty[MAXS];
  __shared__ uint32_t s_wsum[JN_CONSUMERS / 32];
  __shared__ unsigned long long s_wbase[JN_CONSUMERS / 32];
  __shared__ unsigned long long s_red[4][JN_THREADS / 32];

  const uint32_t nslots = 1u << a.slot_bits;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  JnAcc acc;

  if (threadIdx.x == 0) {
    for (uint32_t i = 0; i < NRB; i++) { mbar_init(&full[i], 1); mbar_init(&empty[i], 1); }
    for (uint32_t i = 0; i < NSB; i++) {
      mbar_init(&sfull[i], 1);
      mbar_init(&sempty[i], JN_REL == 0 ? JN_CONSUMERS / 32 : 1);
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  // heads start in epoch 0, which no stage uses: every chain reads as empty
  for (uint32_t i = threadIdx.x * 4; i < nslots; i += JN_THREADS * 4)
    *reinterpret_cast<uint4*>(s_head + i) = make_uint4(0u, 0u, 0u, 0u);
  __syncthreads();

  if (warp == JN_CONSUMERS / 32) {
    // ------------------------------ producer warp ------------------------------
    if (lane == 0) {
      const uint64_t pol = policy_evict_first();
      const uint32_t n_items = *a.n_items;
      const TR* rT = static_cast<const TR*>(a.rt);
      const TS* sT = static_cast<const TS*>(a.st);
      uint32_t stage = 0, sseq = 0;
      for (uint32_t it = blockIdx.x; it < n_items; it += gridDim.x) {
        const uint2 item = a.items[it];
        const uint32_t q = item.x;
        const uint32_t r_lo = a.bR[q], r_hi = a.bR[q + 1];
        const uint32_t s_lo = a.bS[q] + item.y * a.slice;
        const uint32_t s_hi = min(a.bS[q + 1], s_lo + a.slice);
        for (uint32_t c_lo = r_lo; c_lo < r_hi; c_lo += a.cap, stage++) {
          uint32_t bi, ph;
      ring_pos(stage, NRB, bi, ph);
          mbar_wait_backoff(&empty[bi], ph ^ 1);
          const uint32_t nr = min(a.cap, r_hi - c_lo);
          const uintptr_t ra = reinterpret_cast<uintptr_t>(rT + c_lo);
          const uintptr_t r0 = ra & ~(uintptr_t)15, r1 = (ra + (size_t)nr * sizeof(TR) + 15) & ~(uintptr_t)15;
          s_meta[bi] = JnStage{nr, (uint32_t)(ra - r0), s_lo, s_hi};
          mbar_expect_tx(&full[bi], (uint32_t)(r1 - r0));
          bulk_g2s(ring + bi * RB, reinterpret_cast<const void*>(r0), (uint32_t)(r1 - r0), &full[bi], pol);
          if constexpr (SR) {
            // the stage's S slice, tile by tile, through the S ring
            for (uint32_t t0 = s_lo; t0 < s_hi; t0 += JN_STILE, sseq++) {
              uint32_t sb, sph;
              ring_pos(sseq, NSB, sb, sph);
              mbar_wait_backoff(&sempty[sb], sph ^ 1);
              const uint32_t n = min(JN_STILE, s_hi - t0);
              const uintptr_t sa = reinterpret_cast<uintptr_t>(sT + t0);
              const uintptr_t a0 = sa & ~(uintptr_t)15, a1 = (sa + (size_t)n * sizeof(TS) + 15) & ~(uintptr_t)15;
              s_soff[sb] = (uint32_t)(sa - a0);
              mbar_expect_tx(&sfull[sb], (uint32_t)(a1 - a0));
              bulk_g2s(sring + sb * SB, reinterpret_cast<const void*>(a0), (uint32_t)(a1 - a0), &sfull[sb], pol);
            }
          } else {
            // warm L2 with the stage's S slice: the consumers reach it a stage later
            if (c_lo == r_lo && s_hi > s_lo && a.pf_bytes)
              bulk_prefetch_l2(sT + s_lo, min((size_t)(s_hi - s_lo) * sizeof(TS), (size_t)a.pf_bytes));
          }
          // warm L2 with the next item's R chunk (and the head of its S
          // slice): its bulk copy, issued once this stage releases the ring,
          // then streams from L2 instead of HBM
          if ((a.dbg & 8u) == 0 && c_lo == r_lo && it + gridDim.x < n_items) {
            const uint2 nx = a.items[it + gridDim.x];
            const uint32_t nr_lo = a.bR[nx.x], nr_hi = min(a.bR[nx.x + 1], nr_lo + a.cap);
            if (nr_hi > nr_lo) bulk_prefetch_l2(rT + nr_lo, (size_t)(nr_hi - nr_lo) * sizeof(TR));
            if (!SR && a.pf_bytes) {
              const uint32_t ns_lo = a.bS[nx.x] + nx.y * a.slice;
              const uint32_t ns_hi = min(a.bS[nx.x + 1], ns_lo + a.slice);
              if (ns_hi > ns_lo)
                bulk_prefetch_l2(sT + ns_lo, min((size_t)(ns_hi - ns_lo) * sizeof(TS), (size_t)a.pf_bytes));
            }
          }
        }
      }
      uint32_t bi, ph;
      ring_pos(stage, NRB, bi, ph);
      mbar_wait_backoff(&empty[bi], ph ^ 1);
      s_meta[bi].nr = JN_STOP;
      mbar_arrive(&full[bi]);
    }
  } else {
    // ------------------------------ consumer warps -----------------------------
    uint32_t sseq = 0, ep = 0;
    for (uint32_t stage = 0;; stage++) {
      uint32_t bi, ph;
      ring_pos(stage, NRB, bi, ph);
      // stage epoch (1..ep_period, ep_period <= 65535): heads of other
      // epochs read as empty chains, so the table needs no reset; every
      // ep_period stages the heads are zeroed (epoch 0 is never used) -- the
      // previous stage's probe is complete (barrier at the end of the loop body)
      if (++ep > a.ep_period) ep = 1u;
      if (ep == 1u && stage > 0) {
        for (uint32_t i = threadIdx.x * 4; i < nslots; i += JN_CONSUMERS * 4)
          *reinterpret_cast<uint4*>(s_head + i) = make_uint4(0u, 0u, 0u, 0u);
        consumer_sync<JN_CONSUMERS>();
      }
      mbar_wait(&full[bi], ph);
      const JnStage st = s_meta[bi];
      if (st.nr == JN_STOP) break;
      const TR* r = reinterpret_cast<const TR*>(ring + bi * RB + st.off);
      // ---- build (a11): chained table via atomicExch on the heads
      // the first S batch is loaded before the build so its latency hides
      // behind the table construction
      constexpr uint32_t BATCH = JN_U * JN_CONSUMERS;
      // (materialising kernels hold more live state: there the batch is
      // loaded just before it is probed -- HAPE measured the pipelined form 2x
      // slower for C3)
      constexpr bool PIPE = !MAT && !SR;
      Tup<KW, PSW> xs[JN_U];
      // (PTAIL: the ragged last batch is pipelined too, its loads predicated)
      constexpr bool PTAIL = PIPE && HAPE_JN_PTAIL;
      if (PIPE && (PTAIL ? st.s_lo < st.s_hi : st.s_lo + BATCH <= st.s_hi))
        jn_load_batch<KW, PSW, JN_U, JN_CONSUMERS>(a, st.s_lo, st.s_hi, xs);
      if (!(a.dbg & 4u)) {
        if constexpr (KN) {
          // the payload moves to pay[i], the link takes its place in the node
          TR* rw = reinterpret_cast<TR*>(ring + bi * RB + st.off);
          for (uint32_t i = threadIdx.x; i < st.nr; i += JN_CONSUMERS) {
            const TR y = rw[i];
            const uint32_t nx = jn_head(atomicExch(&s_head[jn_slot<KW>(y.k, a.slot_bits)], (ep << 16) | i), ep);
            s_pay[i] = y.v;
            rw[i].v = (typename UW<PRW>::T)nx;
          }
        } else if constexpr (LAY == JN_SK) {
          for (uint32_t i = threadIdx.x; i < st.nr; i += JN_CONSUMERS) {
            const K k = r[i].k;
            s_keys[i] = k;
            s_next[i] = (uint16_t)jn_head(atomicExch(&s_head[jn_slot<KW>(k, a.slot_bits)], (ep << 16) | i), ep);
          }
        } else {
          // (2 / 4 inserts per thread in flight measured 0.634 / 0.642 vs
          // 0.638 ms: the exchanges are not the stage's critical path)
          for (uint32_t i = threadIdx.x; i < st.nr; i += JN_CONSUMERS)
            s_next[i] = (uint16_t)jn_head(atomicExch(&s_head[jn_slot<KW>(r[i].k, a.slot_bits)], (ep << 16) | i), ep);
        }
      }
      consumer_sync<JN_CONSUMERS>();
      // ---- probe (a12): stream the S slice.  Bag semantics walk every chain
      // to its end; a caller-declared unique build side (HAPE_FLAG_R_UNIQUE, a
      // primary key) stops at the first match.
      const JnTable<KW, PRW, LAY> tab{r, KN ? static_cast<const void*>(s_pay) : static_cast<const void*>(s_next),
                                      s_keys, s_head, a.slot_bits, a.r_unique == 0, ep};
      if constexpr (SR) {
        // staged S tiles: wait for the tile, copy this thread's tuples to
        // registers, release the tile (one arrival per warp), probe
        for (uint32_t base = st.s_lo; base < st.s_hi; base += JN_STILE, sseq++) {
          uint32_t sb, sph;
              ring_pos(sseq, NSB, sb, sph);
          mbar_wait(&sfull[sb], sph);
          const TS* tile = reinterpret_cast<const TS*>(sring + sb * SB + s_soff[sb]);
          const uint32_t n = min(JN_STILE, st.s_hi - base);
          constexpr int XU = SR ? SU : 1;
          Tup<KW, PSW> x[XU];
#pragma unroll
          for (int u = 0; u < XU; u++) {
            const uint32_t j = u * JN_CONSUMERS + threadIdx.x;
            if (j < n) x[u] = tile[j];
          }
          // release the tile once every consumer holds its tuples (JN_REL)
          if constexpr (JN_REL == 0) {
            __syncwarp();
            if (lane == 0) mbar_arrive(&sempty[sb]);
          } else {
            consumer_sync<JN_CONSUMERS>();
            if (threadIdx.x == 0) mbar_arrive(&sempty[sb]);
          }
          jn_probe_batch<KW, PRW, PSW, MAT, XU, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, x, acc, s_wsum, s_wbase);
        }
      } else {
        // Full batches are software pipelined (PIPE): batch b+1 is loaded into
        // registers while b is probed.
        uint32_t base = st.s_lo;
        if constexpr (PTAIL) {
          // two register sets alternate (unrolled by two): no copy of the
          // prefetched batch into the probed one
          Tup<KW, PSW> xt[JN_U];
          while (base < st.s_hi) {
            if (base + BATCH < st.s_hi) jn_load_batch<KW, PSW, JN_U, JN_CONSUMERS>(a, base + BATCH, st.s_hi, xt);
            jn_probe_batch<KW, PRW, PSW, MAT, JN_U, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, xs, acc, s_wsum, s_wbase);
            base += BATCH;
            if (base >= st.s_hi) break;
            if (base + BATCH < st.s_hi) jn_load_batch<KW, PSW, JN_U, JN_CONSUMERS>(a, base + BATCH, st.s_hi, xs);
            jn_probe_batch<KW, PRW, PSW, MAT, JN_U, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, xt, acc, s_wsum, s_wbase);
            base += BATCH;
          }
        }
        while (!PTAIL && base + BATCH <= st.s_hi) {
          Tup<KW, PSW> x[JN_U];
          if constexpr (PIPE) {
#pragma unroll
            for (int u = 0; u < JN_U; u++) x[u] = xs[u];
            if (PTAIL ? base + BATCH < st.s_hi : base + 2 * BATCH <= st.s_hi)
              jn_load_batch<KW, PSW, JN_U, JN_CONSUMERS>(a, base + BATCH, st.s_hi, xs);
          } else {
            jn_load_batch<KW, PSW, JN_U, JN_CONSUMERS>(a, base, st.s_hi, x);
          }
          jn_probe_batch<KW, PRW, PSW, MAT, JN_U, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, x, acc, s_wsum, s_wbase);
          base += BATCH;
        }
        // ragged tail (< BATCH tuples, any JN_U): 4-, 2- and 1-wide batches
        // until the slice is exhausted (rem is uniform over the consumers);
        // PTAIL forms have none left
        while (!PTAIL && st.s_hi > base) {
          const uint32_t rem = st.s_hi - base;
          if (rem > 2 * JN_CONSUMERS) {
            Tup<KW, PSW> x[4];
            jn_load_batch<KW, PSW, 4, JN_CONSUMERS>(a, base, st.s_hi, x);
            jn_probe_batch<KW, PRW, PSW, MAT, 4, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, x, acc, s_wsum, s_wbase);
            base += 4 * JN_CONSUMERS;
          } else if (rem > JN_CONSUMERS) {
            Tup<KW, PSW> x[2];
            jn_load_batch<KW, PSW, 2, JN_CONSUMERS>(a, base, st.s_hi, x);
            jn_probe_batch<KW, PRW, PSW, MAT, 2, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, x, acc, s_wsum, s_wbase);
            base += 2 * JN_CONSUMERS;
          } else {
            Tup<KW, PSW> x[1];
            jn_load_batch<KW, PSW, 1, JN_CONSUMERS>(a, base, st.s_hi, x);
            jn_probe_batch<KW, PRW, PSW, MAT, 1, JN_CONSUMERS, LAY>(tab, a, base, st.s_hi, x, acc, s_wsum, s_wbase);
            base += JN_CONSUMERS;
          }
        }
      }
      // KN: generic-proxy writes went into ring buffer bi, which the
      // bulk-copy engine refills next (fenced here, after the probe: a fence
      // right after the build also waited for the S batch loads in flight)
      if constexpr (KN) asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
      consumer_sync<JN_CONSUMERS>();  // everyone is done with heads/next and ring buffer bi
      if (threadIdx.x == 0) mbar_arrive(&empty[bi]);
    }
  }
  // ---- a13: block reduction of the four u64 partials, one atomic each
  unsigned long long cnt = acc.cnt, sr = acc.sr, ss = acc.ss, sx = acc.sx;
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) {
    cnt += __shfl_xor_sync(0xffffffffu, cnt, o);
    sr += __shfl_xor_sync(0xffffffffu, sr, o);
    ss += __shfl_xor_sync(0xffffffffu, ss, o);
    sx += __shfl_xor_sync(0xffffffffu, sx, o);
  }
  if (lane == 0) { s_red[0][warp] = cnt; s_red[1][warp] = sr; s_red[2][warp] = ss; s_red[3][warp] = sx; }
  __syncthreads();
  if (threadIdx.x < 4) {
    unsigned long long t = 0;
    for (int w = 0; w < JN_THREADS / 32; w++) t += s_red[threadIdx.x][w];
    if (t) atomicAdd(&a.acc[threadIdx.x], t);
  }
}

// unpack AoS tuples into key / payload columns (debug entry point only)
template <int KW, int PW>
__global__ void k_unpack(const Tup<KW, PW>* __restrict__ t, uint32_t n, typename UW<KW>::T* __restrict__ k,
                         typename UW<PW>::T* __restrict__ p, uint32_t unmix) {
  for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < n; i += gridDim.x * blockDim.x) {
    const Tup<KW, PW> x = t[i];
    if constexpr (KW == 4) k[i] = unmix ? fmix32_inv(x.k) : x.k;
    else k[i] = unmix ? fmix64_inv(x.k) : x.k;
    p[i] = x.v;
  }
}

}  // namespace hape
