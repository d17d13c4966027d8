// Random gather + scatter (config 3's ADD_C pattern, n = 2^24, len_A = 2^24) --
// does separating the gathers from the scatters in time pay, and at which grain?
//   k_inter   : per thread Q iterations: Q gathers, then Q dependent stores (the flow / quad kernels' shape)
//   k_ctaphase: the CTA gathers its Q*T iterations, __syncthreads, then scatters them
//   k_disjoint: as k_inter but the gathers read [len_A, 2 len_A) (a read-only half, config3_waw's shape)
//   k_gridphase: persistent grid, phases of P iterations: gather -> coalesced buffer, grid barrier, scatter
//   two kernels: gather all (buffer), then scatter all
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o rand_phase rand_phase.cu && ./rand_phase
#include <cooperative_groups.h>
#include <cstdio>
#include <cstdint>
#include <vector>
#include <cuda_runtime.h>
namespace cg = cooperative_groups;

template <int Q>
__global__ void __launch_bounds__(256) k_inter(const int *r, const int *w, uint32_t *A, int64_t n, int64_t roff) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x * Q;
  for (int64_t i0 = (int64_t)blockIdx.x * blockDim.x * Q + threadIdx.x; i0 < n; i0 += stride) {
    int ri[Q], wi[Q];
    uint32_t g[Q];
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + (int64_t)u * blockDim.x;
      if (i < n) { ri[u] = __ldcs(r + i); wi[u] = __ldcs(w + i); }
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + (int64_t)u * blockDim.x;
      if (i < n) g[u] = __ldcg(A + roff + ri[u]);
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + (int64_t)u * blockDim.x;
      if (i < n) __stcg(A + wi[u], g[u] + 1);
    }
  }
}

template <int Q>
__global__ void __launch_bounds__(256) k_ctaphase(const int *r, const int *w, uint32_t *A, int64_t n) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x * Q;
  for (int64_t i0 = (int64_t)blockIdx.x * blockDim.x * Q + threadIdx.x; i0 < n; i0 += stride) {
    int ri[Q], wi[Q];
    uint32_t g[Q];
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + (int64_t)u * blockDim.x;
      if (i < n) { ri[u] = __ldcs(r + i); wi[u] = __ldcs(w + i); }
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + (int64_t)u * blockDim.x;
      if (i < n) g[u] = __ldcg(A + ri[u]);
    }
    __syncthreads();
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + (int64_t)u * blockDim.x;
      if (i < n) __stcg(A + wi[u], g[u] + 1);
    }
    __syncthreads();
  }
}

__global__ void __launch_bounds__(512) k_gridphase(const int *r, const int *w, uint32_t *A, uint32_t *o, int64_t n,
                                                   int64_t P) {
  cg::grid_group grid = cg::this_grid();
  const int64_t G = (int64_t)gridDim.x * blockDim.x, g = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  for (int64_t p0 = 0; p0 < n; p0 += P) {
    const int64_t p1 = p0 + P < n ? p0 + P : n;
    for (int64_t i = p0 + g; i < p1; i += 4 * G) {
      uint32_t v[4];
#pragma unroll
      for (int u = 0; u < 4; u++) if (i + u * G < p1) v[u] = __ldcg(A + __ldcs(r + i + u * G));
#pragma unroll
      for (int u = 0; u < 4; u++) if (i + u * G < p1) __stcg(o + i + u * G, v[u] + 1);
    }
    grid.sync();
    for (int64_t i = p0 + g; i < p1; i += 4 * G) {
      int wi[4]; uint32_t v[4];
#pragma unroll
      for (int u = 0; u < 4; u++) if (i + u * G < p1) { wi[u] = __ldcs(w + i + u * G); v[u] = __ldcg(o + i + u * G); }
#pragma unroll
      for (int u = 0; u < 4; u++) if (i + u * G < p1) __stcg(A + wi[u], v[u]);
    }
    grid.sync();
  }
}

__global__ void k_gather(const int *r, const uint32_t *A, uint32_t *o, int64_t n) {
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    __stcs(o + i, __ldcg(A + __ldcs(r + i)) + 1);
}
__global__ void k_scatter(const int *w, const uint32_t *o, uint32_t *A, int64_t n) {
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    __stcg(A + __ldcs(w + i), __ldcs(o + i));
}

template <typename F> float best_of(F f) {
  cudaEvent_t a, b;
  cudaEventCreate(&a); cudaEventCreate(&b);
  f(); cudaDeviceSynchronize();
  float best = 1e9;
  for (int k = 0; k < 7; k++) {
    cudaEventRecord(a); f(); cudaEventRecord(b); cudaEventSynchronize(b);
    float ms; cudaEventElapsedTime(&ms, a, b);
    if (ms < best) best = ms;
  }
  cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) printf("error %s\n", cudaGetErrorString(e));
  return best * 1e3f;
}

int main() {
  const int64_t n = 1 << 24, lenA = 1 << 24;
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  int *r, *w; uint32_t *A, *o;
  cudaMalloc(&r, 4 * n); cudaMalloc(&w, 4 * n); cudaMalloc(&o, 4 * n); cudaMalloc(&A, 8 * lenA);
  // r: uniform random; w: a permutation (config 3: w = pi, r mostly = w, here independent)
  std::vector<int> h(n), hw(n);
  uint64_t s = 12345;
  for (int64_t i = 0; i < n; i++) { s = s * 6364136223846793005ull + 1442695040888963407ull; h[i] = (int)((s >> 33) % lenA); hw[i] = (int)i; }
  for (int64_t i = n - 1; i > 0; i--) { s = s * 6364136223846793005ull + 1442695040888963407ull; int64_t j = (s >> 33) % (i + 1); std::swap(hw[i], hw[j]); }
  cudaMemcpy(r, h.data(), 4 * n, cudaMemcpyHostToDevice);
  cudaMemcpy(w, hw.data(), 4 * n, cudaMemcpyHostToDevice);
  for (int bps : {4, 8}) {
    const int grid = sms * bps;
    printf("grid %d: inter Q4 %.1f Q8 %.1f | ctaphase Q4 %.1f Q8 %.1f Q16 %.1f | disjoint Q8 %.1f us\n", grid,
           best_of([&] { k_inter<4><<<grid, 256>>>(r, w, A, n, 0); }), best_of([&] { k_inter<8><<<grid, 256>>>(r, w, A, n, 0); }),
           best_of([&] { k_ctaphase<4><<<grid, 256>>>(r, w, A, n); }), best_of([&] { k_ctaphase<8><<<grid, 256>>>(r, w, A, n); }),
           best_of([&] { k_ctaphase<16><<<grid, 256>>>(r, w, A, n); }), best_of([&] { k_inter<8><<<grid, 256>>>(r, w, A, n, lenA); }));
  }
  printf("two kernels: %.1f us (gather %.1f, scatter %.1f)\n",
         best_of([&] { k_gather<<<sms * 8, 256>>>(r, A, o, n); k_scatter<<<sms * 8, 256>>>(w, o, A, n); }),
         best_of([&] { k_gather<<<sms * 8, 256>>>(r, A, o, n); }), best_of([&] { k_scatter<<<sms * 8, 256>>>(w, o, A, n); }));
  // config 3's shape: r = w = pi (each iteration updates one address in place)
  cudaMemcpy(r, w, 4 * n, cudaMemcpyDeviceToDevice);
  printf("r = w (in-place update): inter Q8 %.1f | two kernels %.1f us (gather %.1f, scatter %.1f)\n",
         best_of([&] { k_inter<8><<<sms * 8, 256>>>(r, w, A, n, 0); }),
         best_of([&] { k_gather<<<sms * 8, 256>>>(r, A, o, n); k_scatter<<<sms * 8, 256>>>(w, o, A, n); }),
         best_of([&] { k_gather<<<sms * 8, 256>>>(r, A, o, n); }), best_of([&] { k_scatter<<<sms * 8, 256>>>(w, o, A, n); }));
  cudaMemcpy(r, h.data(), 4 * n, cudaMemcpyHostToDevice);
  int mb = 0; cudaOccupancyMaxActiveBlocksPerMultiprocessor(&mb, k_gridphase, 512, 0);
  for (int64_t P : {1ll << 20, 1ll << 21, 1ll << 22, 1ll << 24}) {
    printf("gridphase P=2^%d: %.1f us\n", __builtin_ctzll(P), best_of([&] {
      int64_t nn = n, PP = P; void *args[] = {&r, &w, &A, &o, &nn, &PP};
      cudaLaunchCooperativeKernel((void *)k_gridphase, dim3(sms * mb), dim3(512), args, 0, 0); }));
  }
  return 0;
}
