// Memory-side ceilings for the scatter's write pattern (developer tool, not
// product code).  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o membench tools/membench.cu
//
//   copy      : streaming uint4 copy (the MEASURED_PEAKS kind of number)
//   read      : streaming uint4 read + reduce (the histogram's ceiling)
//   runs<R>   : read tuples coalesced, write them as runs of R 8-byte tuples
//               into 256 bucket regions (one global claim atomic per bucket per
//               tile, as k_scatter's CLAIM form): the scatter's write pattern
//               without its shared-memory work
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("%s: %s\n", #x, cudaGetErrorString(e)); return 1; } } while (0)

__global__ void k_copy(const uint4* __restrict__ a, uint4* __restrict__ b, size_t n) {
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) b[i] = a[i];
}
__global__ void k_read(const uint4* __restrict__ a, size_t n, unsigned* out) {
  unsigned s = 0;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) {
    uint4 v = a[i];
    s ^= v.x ^ v.y ^ v.z ^ v.w;
  }
  if (s == 0x12345678u) *out = s;
}
// tiles of T tuples; NB buckets; run length T/NB; claim one run per bucket per tile
template <int NT, int T, int NB>
__global__ void __launch_bounds__(NT) k_runs(const uint2* __restrict__ in, uint2* __restrict__ out, size_t n,
                                              unsigned* __restrict__ cur, unsigned tiles_per_cta) {
  constexpr int RL = T / NB;
  __shared__ unsigned s_run[NB];
  const size_t tiles = n / T;
  for (unsigned k = 0; k < tiles_per_cta; k++) {
    const size_t tile = (size_t)blockIdx.x * tiles_per_cta + k;
    if (tile >= tiles) break;
    for (int b = threadIdx.x; b < NB; b += NT) s_run[b] = atomicAdd(&cur[b], (unsigned)RL);
    __syncthreads();
    const uint2* src = in + tile * T;
#pragma unroll 4
    for (int i = threadIdx.x; i < T; i += NT) {
      const uint2 v = src[i];
      const int b = i / RL, o = i - b * RL;
      out[(size_t)s_run[b] + o] = v;
    }
    __syncthreads();
  }
}

// the same runs, but lane i of a warp writes bucket (i % NB): every store
// instruction touches 32 buckets (the pattern of a scatter without the
// shared-memory reorder); the runs still complete inside the tile
template <int NT, int T, int NB>
__global__ void __launch_bounds__(NT) k_direct(const uint2* __restrict__ in, uint2* __restrict__ out, size_t n,
                                                unsigned* __restrict__ cur, unsigned tiles_per_cta) {
  constexpr int RL = T / NB;
  __shared__ unsigned s_run[NB];
  const size_t tiles = n / T;
  for (unsigned k = 0; k < tiles_per_cta; k++) {
    const size_t tile = (size_t)blockIdx.x * tiles_per_cta + k;
    if (tile >= tiles) break;
    for (int b = threadIdx.x; b < NB; b += NT) s_run[b] = atomicAdd(&cur[b], (unsigned)RL);
    __syncthreads();
    const uint2* src = in + tile * T;
#pragma unroll 4
    for (int i = threadIdx.x; i < T; i += NT) {
      const uint2 v = src[i];
      const int b = i % NB, o = i / NB;
      out[(size_t)s_run[b] + o] = v;
    }
    __syncthreads();
  }
}

template <class F>
float timeit(F f, int reps) {
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  f();
  cudaDeviceSynchronize();
  cudaEventRecord(a);
  for (int r = 0; r < reps; r++) f();
  cudaEventRecord(b);
  cudaEventSynchronize(b);
  float ms;
  cudaEventElapsedTime(&ms, a, b);
  return ms / reps;
}

template <int NT, int T, int NB, bool DIRECT = false>
int run_pattern(const uint2* in, uint2* out, size_t n, unsigned* cur, int sms, int per_sm, const char* name) {
  const size_t tiles = n / T;
  const unsigned grid = sms * per_sm;
  const unsigned tpc = (unsigned)((tiles + grid - 1) / grid);
  // bucket b region starts at b * (n/NB): cursors reset before each launch
  unsigned h[NB];
  for (int b = 0; b < NB; b++) h[b] = (unsigned)((size_t)b * (n / NB));
  auto f = [&] {
    cudaMemcpyAsync(cur, h, sizeof(h), cudaMemcpyHostToDevice);
    if (DIRECT) k_direct<NT, T, NB><<<grid, NT>>>(in, out, tiles * T, cur, tpc);
    else k_runs<NT, T, NB><<<grid, NT>>>(in, out, tiles * T, cur, tpc);
  };
  float ms = timeit(f, 10);
  const double bytes = 2.0 * tiles * T * 8;
  printf("{\"kernel\": \"%s\", \"T\": %d, \"buckets\": %d, \"run_tuples\": %d, \"ctas_per_sm\": %d, \"ms\": %.4f, \"GB/s\": %.1f}\n",
         name, T, NB, T / NB, per_sm, ms, bytes / ms / 1e6);
  return 0;
}

int main() {
  int sms;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const size_t n = (size_t)1 << 28;  // 8-byte tuples: 2 GiB in, 2 GiB out (one pass over R+S of C2)
  uint2 *in, *out;
  unsigned* cur;
  CK(cudaMalloc(&in, n * 8));
  CK(cudaMalloc(&out, n * 8));
  CK(cudaMalloc(&cur, 4096 * 4));
  CK(cudaMemset(in, 1, n * 8));
  CK(cudaMemset(out, 0, n * 8));
  const size_t n4 = n * 8 / 16;
  for (int per : {2, 4, 8}) {
    float ms = timeit([&] { k_copy<<<sms * per, 512>>>((const uint4*)in, (uint4*)out, n4); }, 10);
    printf("{\"kernel\": \"copy\", \"ctas_per_sm\": %d, \"ms\": %.4f, \"GB/s\": %.1f}\n", per, ms, 2.0 * n * 8 / ms / 1e6);
  }
  for (int per : {2, 4, 8}) {
    float ms = timeit([&] { k_read<<<sms * per, 512>>>((const uint4*)in, n4, cur); }, 10);
    printf("{\"kernel\": \"read\", \"ctas_per_sm\": %d, \"ms\": %.4f, \"GB/s\": %.1f}\n", per, ms, 1.0 * n * 8 / ms / 1e6);
  }
  run_pattern<512, 6656, 256>(in, out, n, cur, sms, 2, "runs");
  run_pattern<512, 6656, 256>(in, out, n, cur, sms, 4, "runs");
  run_pattern<512, 13312, 256>(in, out, n, cur, sms, 2, "runs");
  run_pattern<512, 3328, 256>(in, out, n, cur, sms, 4, "runs");
  run_pattern<1024, 12288, 1024>(in, out, n, cur, sms, 2, "runs");
  run_pattern<512, 6144, 1024>(in, out, n, cur, sms, 4, "runs");
  run_pattern<512, 8192, 64>(in, out, n, cur, sms, 4, "runs");
  run_pattern<512, 6656, 256, true>(in, out, n, cur, sms, 2, "direct");
  run_pattern<512, 6656, 256, true>(in, out, n, cur, sms, 4, "direct");
  run_pattern<512, 13312, 256, true>(in, out, n, cur, sms, 2, "direct");
  run_pattern<1024, 12288, 1024, true>(in, out, n, cur, sms, 2, "direct");
  return 0;
}
