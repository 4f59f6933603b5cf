// join_oa.cuh -- a11-a13, open-addressing form of the per-co-partition
// build + probe (§4.1: "load the smaller partition to the
// scratchpad, build the hash-table using atomic operations and probe with
// the tuples of the corresponding partition", P537-540; Fig. 3, P472-494).
//
// The table of a stage IS the R chunk: 2^sb slots of (key, payload) tuples in
// shared memory, filled by linear probing with one shared-memory CAS per R
// tuple (the "atomic operations" of P538-539), probed by every S tuple of the
// co-partition with one 8- or 16-byte shared load per visited slot.  There
// is no R staging ring, no next[] / head[] indirection and no per-stage table
// reset:
//
//   * "empty" is decided by the partition function, not by a sentinel: every
//     tuple of co-partition q has (h(key) & qmask) == q (the radix passes put
//     it there, R3), so a slot whose key belongs to another
//     co-partition is free for stage q -- whatever earlier stage left it.
//     A slot can look occupied only if an earlier stage of the SAME
//     co-partition wrote it (R-chunks of one co-partition, or consecutive
//     S-slices of it on this CTA) or if the fill key belongs to q: then
//     (and only then) the table is refilled with a key of another
//     co-partition first.  Items of one co-partition are contiguous in the
//     work list, so this CTA meets them in consecutive stages: remembering
//     the last co-partition built into each table (and the fill key's
//     co-partition) decides the refill exactly.
//   * NTAB = 2 alternates two tables: the build of stage t+1 goes into the
//     other table while slower warps still probe stage t, so a stage costs
//     one block barrier (build -> barrier -> probe).  NTAB = 1: two.
//
// The R chunk streams into registers (coalesced 8/16-byte loads, the next
// item's chunk prefetched into L2 one item ahead by the bulk-copy engine),
// S tuples stream from HBM in register-pipelined batches of U per thread.
// Unique build side (HAPE_FLAG_R_UNIQUE): a probe stops at its match; bag
// semantics: it walks the cluster to the first free slot, counting every
// equal key (duplicates occupy their own slots).
#pragma once
#include "kernels.cuh"

namespace hape {

constexpr int OA_CAPMAX = 3072;  // R tuples per stage (registers: OA_CAPMAX / NC per thread)
// CTAs per SM the 256-thread form is register-budgeted for (78 registers,
// no spills; two 32 KB int32 tables per CTA also fit 3 per SM)
#ifndef OA_MINB
#define OA_MINB 3
#endif
// 8-byte tuples: one 64-bit CAS of the whole tuple (OA_CAS64 = 1) or a 32-bit
// CAS of the key then the payload store (0; 64-bit shared CAS measured ~6x
// slower per build on B200)
#ifndef OA_CAS64
#define OA_CAS64 0
#endif

// a key that is NOT in co-partition q (fill value of a refilled table):
// h(0) = 0 for all three partition functions, and h(1) is odd for each
// (identity: 1; fmix32(1) = 0x514e28b7; fmix64(1) = 0x5692161d100b05e5),
// so with qmask >= 1 key 1 is never in co-partition 0.
__host__ __device__ __forceinline__ uint32_t oa_fill_key(uint32_t q) { return q != 0 ? 0u : 1u; }

template <int KW, bool IDENT>
__device__ __forceinline__ uint32_t oa_part(typename UW<KW>::T k, uint32_t qmask) {
  return (uint32_t)part_hash<KW, IDENT>(k) & qmask;
}

template <int KW, int PRW>
__device__ __forceinline__ Tup<KW, PRW> lds_tup(const Tup<KW, PRW>* p) {
  return *p;  // one LDS.64 / LDS.128
}

// insert one R tuple by linear probing (CAS on the whole 8-byte tuple, or on
// the key of a 16-byte tuple followed by the payload store; probes only run
// after the stage barrier)
template <int KW, int PRW, bool IDENT>
__device__ __forceinline__ void oa_insert(Tup<KW, PRW>* T, uint32_t smask, uint32_t sb, const Tup<KW, PRW>& x,
                                          uint32_t q, uint32_t qmask) {
  using K = typename UW<KW>::T;
  uint32_t s = jn_slot<KW>(x.k, sb);
  if constexpr (sizeof(Tup<KW, PRW>) == 8 && OA_CAS64) {
    // (the only 8-byte tuple is (u32 key, u32 payload): key = low word)
    static_assert(KW == 4 && PRW == 4, "8-byte tuple layout");
    unsigned long long* T64 = reinterpret_cast<unsigned long long*>(T);
    const unsigned long long nv = (unsigned long long)x.k | ((unsigned long long)x.v << 32);
    unsigned long long cur = T64[s];
    while (true) {
      if (oa_part<KW, IDENT>((K)(uint32_t)cur, qmask) != q) {
        const unsigned long long prev = atomicCAS(T64 + s, cur, nv);
        if (prev == cur) return;
        cur = prev;  // taken meanwhile: re-examine the same slot
        continue;
      }
      s = (s + 1) & smask;
      cur = T64[s];
    }
  } else {
    using KC = typename std::conditional<KW == 4, unsigned int, unsigned long long>::type;
    KC* kp = reinterpret_cast<KC*>(&T[s].k);
    KC cur = *kp;
    while (true) {
      if (oa_part<KW, IDENT>((K)cur, qmask) != q) {
        const KC prev = atomicCAS(kp, cur, (KC)x.k);
        if (prev == cur) {
          T[s].v = x.v;
          return;
        }
        cur = prev;
        continue;
      }
      s = (s + 1) & smask;
      kp = reinterpret_cast<KC*>(&T[s].k);
      cur = *kp;
    }
  }
}

struct OaTab {
  uint32_t smask, sb, q, qmask;
  bool unique;
};

// probe U S tuples (x[u] valid iff base + u*NC + tid < s_hi)
template <int KW, int PRW, int PSW, bool MAT, bool IDENT, int U, int NC>
__device__ __forceinline__ void oa_probe_batch(const Tup<KW, PRW>* T, const OaTab& t, const JoinArgs& a,
                                               uint32_t base, uint32_t s_hi, const Tup<KW, PSW> (&x)[U],
                                               JnAcc& acc, uint32_t* s_wsum, unsigned long long* s_wbase) {
  using PR = typename UW<PRW>::S;
  using PS = typename UW<PSW>::S;
  using TR = Tup<KW, PRW>;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint32_t sl[U];
  TR e[U];
  bool v[U];
#pragma unroll
  for (int u = 0; u < U; u++) {
    v[u] = base + u * NC + threadIdx.x < s_hi;
    sl[u] = jn_slot<KW>(x[u].k, t.sb);
    if (v[u]) e[u] = lds_tup(T + sl[u]);
  }
  uint32_t c[U];
  typename UW<PRW>::T m[U];
#pragma unroll
  for (int u = 0; u < U; u++) {
    c[u] = 0;
    m[u] = 0;
    if (!v[u]) continue;
    uint32_t s = sl[u];
    TR y = e[u];
    if (t.unique) {
      // first equal key ends the walk; a slot of another co-partition is free
      bool hit = true;
      while (y.k != x[u].k) {
        if (oa_part<KW, IDENT>(y.k, t.qmask) != t.q) { hit = false; break; }
        s = (s + 1) & t.smask;
        y = lds_tup(T + s);
      }
      if (hit) {
        const int64_t pr = (int64_t)(PR)y.v, ps = (int64_t)(PS)x[u].v;
        c[u] = 1;
        m[u] = y.v;
        acc.sr += (unsigned long long)pr;
        acc.ss += (unsigned long long)ps;
        acc.sx += pair_mix(pr, ps);
      }
    } else {
      // bag semantics: every equal key of the cluster
      while (true) {
        if (y.k == x[u].k) {
          const int64_t pr = (int64_t)(PR)y.v, ps = (int64_t)(PS)x[u].v;
          if (MAT && c[u] == 0) m[u] = y.v;
          c[u]++;
          acc.sr += (unsigned long long)pr;
          acc.ss += (unsigned long long)ps;
          acc.sx += pair_mix(pr, ps);
        } else if (oa_part<KW, IDENT>(y.k, t.qmask) != t.q) {
          break;
        }
        s = (s + 1) & t.smask;
        y = lds_tup(T + s);
      }
    }
    acc.cnt += c[u];
  }
  if constexpr (MAT) {
    // positions in (u-major, lane-minor) order inside the warp, warps in
    // order inside the block, one global claim per block per batch
    uint32_t incl[U], before[U], wtot = 0;
#pragma unroll
    for (int u = 0; u < U; u++) {
      incl[u] = warp_incl_scan(c[u]);
      before[u] = wtot;
      wtot += __shfl_sync(0xffffffffu, incl[u], 31);
    }
    if (lane == 0) s_wsum[warp] = wtot;
    __syncthreads();
    if (warp == 0) {
      const uint32_t vv = lane < NC / 32 ? s_wsum[lane] : 0u;
      const uint32_t inc = warp_incl_scan(vv);
      const uint32_t tot = __shfl_sync(0xffffffffu, inc, 31);
      unsigned long long g = 0;
      if (lane == 0 && tot) g = atomicAdd(a.out_ctr, (unsigned long long)tot);
      g = __shfl_sync(0xffffffffu, g, 0);
      if (lane < NC / 32) s_wbase[lane] = g + inc - vv;
    }
    __syncthreads();
    const unsigned long long wb = s_wbase[warp];
#pragma unroll
    for (int u = 0; u < U; u++) {
      if (!c[u]) continue;
      unsigned long long pos = wb + before[u] + incl[u] - c[u];
      if (c[u] == 1) {
        if (pos < a.out_cap) {
          static_cast<PR*>(a.out_r)[pos] = (PR)m[u];
          static_cast<PS*>(a.out_s)[pos] = (PS)x[u].v;
        }
        continue;
      }
      // several equal keys: walk the cluster again, writing each
      uint32_t s = sl[u];
      while (true) {
        const TR y = lds_tup(T + s);
        if (y.k == x[u].k) {
          if (pos < a.out_cap) {
            static_cast<PR*>(a.out_r)[pos] = (PR)y.v;
            static_cast<PS*>(a.out_s)[pos] = (PS)x[u].v;
          }
          pos++;
        } else if (oa_part<KW, IDENT>(y.k, t.qmask) != t.q) {
          break;
        }
        s = (s + 1) & t.smask;
      }
    }
  }
}

template <int KW, int PRW, int NC, int NTAB>
__host__ __device__ constexpr size_t oa_smem_bytes(uint32_t sb) {
  return (size_t)NTAB * ((size_t)sizeof(Tup<KW, PRW>) << sb);
}

template <int KW, int PRW, int PSW, bool MAT, bool IDENT, int NC, int NTAB, int U>
__global__ void __launch_bounds__(NC, NC >= 512 ? 2 : OA_MINB) k_join_oa(JoinArgs a) {
  using TR = Tup<KW, PRW>;
  using TS = Tup<KW, PSW>;
  constexpr int RPT = (OA_CAPMAX + NC - 1) / NC;
  constexpr int RG = sizeof(TR) == 8 ? RPT : 2;
  extern __shared__ __align__(128) unsigned char smem[];
  TR* tabs = reinterpret_cast<TR*>(smem);
  __shared__ uint32_t s_wsum[NC / 32];
  __shared__ unsigned long long s_wbase[NC / 32];
  __shared__ unsigned long long s_red[4][NC / 32];
  const uint32_t nslot = 1u << a.slot_bits, smask = nslot - 1;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const TR* __restrict__ rT = static_cast<const TR*>(a.rt);
  const TS* __restrict__ sT = static_cast<const TS*>(a.st);
  const uint32_t qmask = a.qmask;

  // every slot starts with key 0 (co-partition 0).  Per table: tq = the
  // co-partition last built into it, tf = the co-partition of its fill key
  {
    TR z;
    z.k = 0;
    z.v = 0;
    for (uint32_t i = threadIdx.x; i < NTAB * nslot; i += NC) tabs[i] = z;
  }
  uint32_t tq0 = 0xFFFFFFFFu, tf0 = 0u, tq1 = 0xFFFFFFFFu, tf1 = 0u;
  __syncthreads();

  JnAcc acc;
  const uint32_t n_items = *a.n_items;
  uint32_t stage = 0;
  for (uint32_t it = blockIdx.x; it < n_items; it += gridDim.x) {
    const uint2 item = a.items[it];
    const uint32_t q = item.x;
    const uint32_t r_lo = a.bR[q], r_hi = a.bR[q + 1];
    const uint32_t s_lo = a.bS[q] + item.y * a.slice;
    const uint32_t s_hi = min(a.bS[q + 1], s_lo + a.slice);
    // warm L2 with the next item's R chunk and the head of its S slice
    if (threadIdx.x == 0 && it + gridDim.x < n_items && a.pf_bytes) {
      const uint2 nx = a.items[it + gridDim.x];
      const uint32_t nr_lo = a.bR[nx.x], nr_hi = a.bR[nx.x + 1];
      const uint32_t ns_lo = a.bS[nx.x] + nx.y * a.slice;
      const uint32_t ns_hi = min(a.bS[nx.x + 1], ns_lo + a.slice);
      if (nr_hi > nr_lo) bulk_prefetch_l2(rT + nr_lo, (size_t)min(nr_hi - nr_lo, a.cap) * sizeof(TR));
      if (ns_hi > ns_lo) bulk_prefetch_l2(sT + ns_lo, min((size_t)(ns_hi - ns_lo) * sizeof(TS), (size_t)a.pf_bytes));
    }
    for (uint32_t c_lo = r_lo; c_lo < r_hi; c_lo += a.cap, stage++) {
      const bool t1 = NTAB == 2 && (stage & 1u);
      TR* T = tabs + (t1 ? nslot : 0u);
      const uint32_t c_hi = min(r_hi, c_lo + a.cap);
      // R chunk -> registers (coalesced; the loads overlap the refill check).
      // 16-byte tuples go in groups of RG per thread (register budget).
      TR xr[RG];
#pragma unroll
      for (int u = 0; u < RG; u++) {
        const uint32_t i = c_lo + u * NC + threadIdx.x;
        if (i < c_hi) xr[u] = ldcs_tup(rT + i);
      }
      // Entries of this very co-partition (an earlier chunk or slice of it)
      // or fill keys of it would read as occupied: refill the table with a
      // key of another co-partition first.  Uniform over the block; the
      // table's last probe is ordered before this point by the previous
      // stage's barrier (NTAB = 1: the end-of-stage barrier; NTAB = 2: the
      // build barrier of stage - 1).
      uint32_t tf = t1 ? tf1 : tf0;
      if (q == (t1 ? tq1 : tq0) || q == tf) {
        const typename UW<KW>::T fk = (typename UW<KW>::T)oa_fill_key(q);
        TR z;
        z.k = fk;
        z.v = 0;
        for (uint32_t i = threadIdx.x; i < nslot; i += NC) T[i] = z;
        tf = oa_part<KW, IDENT>(fk, qmask);
        __syncthreads();
      }
      if (t1) { tq1 = q; tf1 = tf; } else { tq0 = q; tf0 = tf; }
      // ---- build (a11)
      if constexpr (RG == RPT) {
#pragma unroll
        for (int u = 0; u < RPT; u++) {
          const uint32_t i = c_lo + u * NC + threadIdx.x;
          if (i < c_hi) oa_insert<KW, PRW, IDENT>(T, smask, a.slot_bits, xr[u], q, qmask);
        }
      } else {
#pragma unroll
      for (int u0 = 0; u0 < RPT; u0 += RG) {
        if (u0 > 0) {
#pragma unroll
          for (int u = 0; u < RG; u++) {
            const uint32_t i = c_lo + (u0 + u) * NC + threadIdx.x;
            if (u0 + u < RPT && i < c_hi) xr[u] = ldcs_tup(rT + i);
          }
        }
#pragma unroll
        for (int u = 0; u < RG; u++) {
          const uint32_t i = c_lo + (u0 + u) * NC + threadIdx.x;
          if (u0 + u < RPT && i < c_hi) oa_insert<KW, PRW, IDENT>(T, smask, a.slot_bits, xr[u], q, qmask);
        }
      }
      }
      __syncthreads();
      // ---- probe (a12): the S slice in register-pipelined batches
      const OaTab tab{smask, a.slot_bits, q, qmask, a.r_unique != 0};
      constexpr uint32_t BATCH = U * NC;
      constexpr bool PIPE = !MAT;
      uint32_t base = s_lo;
      TS xs[U];
      if (PIPE && base + BATCH <= s_hi) {
#pragma unroll
        for (int u = 0; u < U; u++) xs[u] = ldcs_tup(sT + base + u * NC + threadIdx.x);
      }
      while (base + BATCH <= s_hi) {
        TS x[U];
        if constexpr (PIPE) {
#pragma unroll
          for (int u = 0; u < U; u++) x[u] = xs[u];
          if (base + 2 * BATCH <= s_hi) {
#pragma unroll
            for (int u = 0; u < U; u++) xs[u] = ldcs_tup(sT + base + BATCH + u * NC + threadIdx.x);
          }
        } else {
#pragma unroll
          for (int u = 0; u < U; u++) x[u] = ldcs_tup(sT + base + u * NC + threadIdx.x);
        }
        oa_probe_batch<KW, PRW, PSW, MAT, IDENT, U, NC>(T, tab, a, base, s_hi, x, acc, s_wsum, s_wbase);
        base += BATCH;
      }
      while (s_hi > base) {  // ragged tail, uniform over the block
        TS x[1];
        const uint32_t j = base + threadIdx.x;
        if (j < s_hi) x[0] = ldcs_tup(sT + j);
        oa_probe_batch<KW, PRW, PSW, MAT, IDENT, 1, NC>(T, tab, a, base, s_hi, x, acc, s_wsum, s_wbase);
        base += NC;
      }
      if (NTAB == 1) __syncthreads();  // the next build overwrites this table
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
    for (int w = 0; w < NC / 32; w++) t += s_red[threadIdx.x][w];
    if (t) atomicAdd(&a.acc[threadIdx.x], t);
  }
}

}  // namespace hape
