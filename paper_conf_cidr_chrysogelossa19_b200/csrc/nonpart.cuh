// nonpart.cuh -- the non-partitioned GPU hash join.
//
// PAPER.md §6.2 / Fig. 6 (P859-870) compares the hardware-conscious
// partitioned join against "non-partitioned CPU and GPU joins implemented in
// our system" and reports "an over 3x speed-up against the non-partitioned
// variant for the highest supported in-GPU size".  This is that variant,
// rebuilt for B200 so the comparison can be re-run on this hardware: ONE hash
// table over all of R in HBM (no partitioning, no scratchpad), built with
// global atomics, probed by every S tuple with random HBM accesses.
//
// Table: open addressing with linear probing, 2^t >= 2|R| slots (load factor
// <= 0.5), one slot = {key, payload, tag} in one 16- or 32-byte aligned
// record, so a probe step is one sector.  Slot of a key = low bits of the
// same bijective mixer the radix join partitions with (fmix32 / fmix64);
// the table does not depend on the partition function option.
//
// Build: claim a slot with atomicCAS on its tag, then store key and payload.
// Probe (a later kernel, so every build store is visible): walk from the
// key's slot to the first empty tag; every slot with an equal key is a match
// (bag semantics), or stop at the first match for a declared unique R.  The
// aggregation (count, two sums, the pair checksum) is that of the radix
// join; materialisation claims output space once per block per batch.
#pragma once
#include "kernels.cuh"

namespace hape {

// key and payload first (one 8- or 16-byte store after the claim), the tag
// behind them; the probe reads a whole slot with 16-byte loads
template <int KW, int PW> struct NpSlot;
template <> struct alignas(16) NpSlot<4, 4> { uint32_t key; uint32_t pay; uint32_t tag; uint32_t pad; };
template <> struct alignas(16) NpSlot<4, 8> { uint32_t key; uint32_t tag; uint64_t pay; };
template <> struct alignas(32) NpSlot<8, 4> { uint64_t key; uint32_t pay; uint32_t tag; uint64_t pad[2]; };
template <> struct alignas(32) NpSlot<8, 8> { uint64_t key; uint64_t pay; uint32_t tag; uint32_t pad; uint64_t pad2; };

template <int KW, int PW>
__device__ __forceinline__ NpSlot<KW, PW> np_load(const NpSlot<KW, PW>* p) {
  NpSlot<KW, PW> e;
  const uint4* src = reinterpret_cast<const uint4*>(p);
  uint4* dst = reinterpret_cast<uint4*>(&e);
  if constexpr (sizeof(NpSlot<KW, PW>) == 16) {
    dst[0] = __ldg(src);
  } else {
    const uint4 a = __ldg(src), b = __ldg(src + 1);
    dst[0] = a;
    dst[1] = b;
  }
  return e;
}

template <int KW>
__device__ __forceinline__ uint32_t np_slot(typename UW<KW>::T k, uint32_t mask) {
  return (uint32_t)part_hash<KW, false>(k) & mask;
}

constexpr int NP_THREADS = 256;

// one claim attempt of an insert at slot s: true when the tuple now owns it
template <int KW, int PW>
__device__ __forceinline__ bool np_try(NpSlot<KW, PW>* __restrict__ tab, uint32_t s, typename UW<KW>::T k,
                                       typename UW<PW>::T p) {
  if constexpr (sizeof(NpSlot<KW, PW>) == 16) {
    // 16-byte slots: the whole slot (tag set) in one 128-bit compare-and-swap
    // (C2 build 11.7 ms, ~11.5 G random-address CAS/s -- the L2 atomic
    // units' rate; a 32-bit tag CAS + two stores measured 14.8 ms)
    // against an empty slot -- one memory operation per insert attempt
    NpSlot<KW, PW> v{};
    v.key = k;
    v.pay = p;
    v.tag = 1;
    const ulonglong2 nv = *reinterpret_cast<const ulonglong2*>(&v);
    unsigned long long olo, ohi;
    asm volatile(
        "{\n .reg .b128 d, b, c;\n mov.b128 b, {%2, %3};\n mov.b128 c, {%4, %5};\n"
        " atom.global.cas.b128 d, [%6], b, c;\n mov.b128 {%0, %1}, d;\n}"
        : "=l"(olo), "=l"(ohi)
        : "l"(0ull), "l"(0ull), "l"(nv.x), "l"(nv.y), "l"(tab + s)
        : "memory");
    return olo == 0ull && ohi == 0ull;
  } else {
    if (atomicCAS(&tab[s].tag, 0u, 1u) != 0u) return false;
    if constexpr (KW == 8 && PW == 8) {
      *reinterpret_cast<ulonglong2*>(&tab[s]) = make_ulonglong2(k, p);
    } else {
      tab[s].key = k;
      tab[s].pay = p;
    }
    return true;
  }
}

// NP_U probes per thread in flight (C2 probe 4.74 -> 4.37 ms).  The build
// stays one insert at a time: four independent 128-bit CAS per thread
// measured 13.2 vs 12.1 ms -- the inserts are bound by random atomics into
// the 4 GB table (a read-modify-write of a random DRAM sector each), not by
// latency.
constexpr int NP_U = 4;

template <int KW, int PW>
__global__ void __launch_bounds__(NP_THREADS)
k_np_build(const typename UW<KW>::T* __restrict__ rk, const typename UW<PW>::T* __restrict__ rp, uint32_t n,
           NpSlot<KW, PW>* __restrict__ tab, uint32_t mask) {
  for (uint32_t i = blockIdx.x * NP_THREADS + threadIdx.x; i < n; i += gridDim.x * NP_THREADS) {
    const typename UW<KW>::T k = rk[i];
    const typename UW<PW>::T p = rp[i];
    uint32_t s = np_slot<KW>(k, mask);
    while (!np_try<KW, PW>(tab, s, k, p)) s = (s + 1) & mask;
  }
}

template <int KW, int PRW, int PSW, bool MAT>
__global__ void __launch_bounds__(NP_THREADS)
k_np_probe(const typename UW<KW>::T* __restrict__ sk, const typename UW<PSW>::T* __restrict__ sp, uint32_t n,
           const NpSlot<KW, PRW>* __restrict__ tab, uint32_t mask, uint32_t r_unique,
           unsigned long long* __restrict__ acc_out, void* out_r, void* out_s, unsigned long long out_cap,
           unsigned long long* __restrict__ out_ctr) {
  using PR = typename UW<PRW>::S;
  using PS = typename UW<PSW>::S;
  __shared__ unsigned long long s_red[4][NP_THREADS / 32];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  unsigned long long cnt = 0, sr = 0, ss = 0, sx = 0;
  if constexpr (MAT) {
    // materialising: block-synchronous batches of one S tuple per thread;
    // walk (count + aggregate, remember the first match), block scan of the
    // match counts, ONE output claim per block per batch, then write (a
    // second walk only for tuples with more than one match).  NP_U tuples per
    // thread per batch measured slower for C3 (57.1 vs 54.3 ms): 2^30 probes
    // into an 8 GB table are bound by random 32-byte DRAM reads (~0.9 TB/s
    // incl. the pair stores), not by the latency of one probe per thread.
    __shared__ uint32_t s_c[NP_THREADS];
    __shared__ uint32_t s_wt[33];
    __shared__ unsigned long long s_base;
    for (uint32_t base = blockIdx.x * NP_THREADS; base < n; base += gridDim.x * NP_THREADS) {
      const uint32_t j = base + threadIdx.x;
      uint32_t c = 0, s0 = 0;
      typename UW<KW>::T k{};
      int64_t q = 0, p0 = 0;
      if (j < n) {
        k = sk[j];
        q = (int64_t)(PS)sp[j];
        s0 = np_slot<KW>(k, mask);
        for (uint32_t s = s0;; s = (s + 1) & mask) {
          const NpSlot<KW, PRW> e = np_load(tab + s);
          if (!e.tag) break;
          if (e.key == k) {
            const int64_t p = (int64_t)(PR)e.pay;
            if (!c) p0 = p;
            c++;
            sr += (unsigned long long)p;
            ss += (unsigned long long)q;
            sx += pair_mix(p, q);
            if (r_unique) break;
          }
        }
        cnt += c;
      }
      s_c[threadIdx.x] = c;
      __syncthreads();
      const uint32_t tot = block_exscan_smem<NP_THREADS>(s_c, NP_THREADS, s_wt);
      if (threadIdx.x == 0) s_base = tot ? atomicAdd(out_ctr, (unsigned long long)tot) : 0ull;
      __syncthreads();
      unsigned long long pos = s_base + s_c[threadIdx.x];
      if (c == 1) {
        if (pos < out_cap) {
          static_cast<PR*>(out_r)[pos] = (PR)p0;
          static_cast<PS*>(out_s)[pos] = (PS)q;
        }
      } else if (c > 1) {
        for (uint32_t s = s0;; s = (s + 1) & mask) {
          const NpSlot<KW, PRW> e = np_load(tab + s);
          if (!e.tag) break;
          if (e.key == k) {
            if (pos < out_cap) {
              static_cast<PR*>(out_r)[pos] = (PR)e.pay;
              static_cast<PS*>(out_s)[pos] = (PS)q;
            }
            pos++;
          }
        }
      }
      __syncthreads();  // s_c / s_base are reused by the next batch
    }
  } else {
    // NP_U S tuples per thread: their first slot loads are issued together
    // (independent random HBM reads in flight), then each walks on from its
    // loaded slot to the first empty one (or its first match, unique R)
    for (uint32_t base = blockIdx.x * NP_THREADS * NP_U + threadIdx.x; base < n;
         base += gridDim.x * NP_THREADS * NP_U) {
      typename UW<KW>::T k[NP_U];
      int64_t q[NP_U];
      uint32_t sl[NP_U];
      NpSlot<KW, PRW> e[NP_U];
      bool v[NP_U];
#pragma unroll
      for (int u = 0; u < NP_U; u++) {
        const uint32_t j = base + u * NP_THREADS;
        v[u] = j < n;
        if (v[u]) {
          k[u] = sk[j];
          q[u] = (int64_t)(PS)sp[j];
          sl[u] = np_slot<KW>(k[u], mask);
        }
      }
#pragma unroll
      for (int u = 0; u < NP_U; u++)
        if (v[u]) e[u] = np_load(tab + sl[u]);
#pragma unroll
      for (int u = 0; u < NP_U; u++) {
        if (!v[u]) continue;
        uint32_t s = sl[u];
        NpSlot<KW, PRW> x = e[u];
        while (x.tag) {
          if (x.key == k[u]) {
            const int64_t p = (int64_t)(PR)x.pay;
            cnt++;
            sr += (unsigned long long)p;
            ss += (unsigned long long)q[u];
            sx += pair_mix(p, q[u]);
            if (r_unique) break;
          }
          s = (s + 1) & mask;
          x = np_load(tab + s);
        }
      }
    }
  }
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
    for (int w = 0; w < NP_THREADS / 32; w++) t += s_red[threadIdx.x][w];
    if (t) atomicAdd(&acc_out[threadIdx.x], t);
  }
}

}  // namespace hape
