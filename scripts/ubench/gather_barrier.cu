// Micro-benchmark (not product code): the two costs of one on-chip TLS window on
// the grid path -- K random 4-byte gathers per thread from a 64 MiB array, and a
// software grid barrier -- measured separately and together.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gb gather_barrier.cu && /tmp/gb
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ void gsync(unsigned *count, unsigned target) {
  asm volatile("barrier.sync 0;" ::: "memory");
  if (threadIdx.x == 0) {
    asm volatile("fence.acq_rel.gpu;\n\tred.relaxed.gpu.global.add.u32 [%0], 1;" ::"l"(count) : "memory");
    unsigned v;
    do { asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(count) : "memory"); } while (v < target);
    asm volatile("fence.acq_rel.gpu;" ::: "memory");
  }
  asm volatile("barrier.sync 0;" ::: "memory");
}

template <int K, bool GATHER, bool BAR>
__global__ void __launch_bounds__(512, 1) kern(const uint32_t *A, const int32_t *idx, int rounds, unsigned *bar,
                                               uint32_t *sink) {
  const uint32_t G = gridDim.x * 512, g = blockIdx.x * 512 + threadIdx.x;
  uint32_t acc = 0;
  for (int rd = 0; rd < rounds; rd++) {
    if (GATHER) {
      uint32_t v[K];
#pragma unroll
      for (int k = 0; k < K; k++) v[k] = __ldcg(A + __ldg(idx + ((uint32_t)rd * K * G + k * G + g) % (1u << 24)));
#pragma unroll
      for (int k = 0; k < K; k++) acc += v[k];
    }
    if (BAR) gsync(bar, gridDim.x * (rd + 1));
  }
  if (acc == 0x12345678) sink[g] = acc;
}

template <int K, bool GATHER, bool BAR>
float run(const uint32_t *A, const int32_t *idx, unsigned *bar, uint32_t *sink, int grid, int rounds) {
  cudaMemset(bar, 0, 8);
  cudaEvent_t a, b;
  cudaEventCreate(&a); cudaEventCreate(&b);
  void *args[] = {(void *)&A, (void *)&idx, (void *)&rounds, (void *)&bar, (void *)&sink};
  cudaLaunchCooperativeKernel((void *)kern<K, GATHER, BAR>, grid, 512, args, 0, 0);
  cudaMemset(bar, 0, 8);
  cudaEventRecord(a);
  cudaLaunchCooperativeKernel((void *)kern<K, GATHER, BAR>, grid, 512, args, 0, 0);
  cudaEventRecord(b);
  cudaEventSynchronize(b);
  float ms; cudaEventElapsedTime(&ms, a, b);
  return ms * 1000.f / rounds;   // us per round
}

int main() {
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const size_t n = 1u << 24;
  uint32_t *A; int32_t *idx; unsigned *bar; uint32_t *sink;
  cudaMalloc(&A, 4 * n); cudaMalloc(&idx, 4 * n); cudaMalloc(&bar, 8); cudaMalloc(&sink, 4 * 148 * 512);
  // random indices (LCG on the host)
  int32_t *h = new int32_t[n];
  uint64_t x = 88172645463325252ull;
  for (size_t i = 0; i < n; i++) { x ^= x << 13; x ^= x >> 7; x ^= x << 17; h[i] = (int32_t)(x % n); }
  cudaMemcpy(idx, h, 4 * n, cudaMemcpyHostToDevice);
  cudaMemset(A, 1, 4 * n);
  const int rounds = 200;
  printf("grid %d CTAs x 512 threads\n", sms);
  printf("barrier only            : %.2f us/round\n", run<4, false, true>(A, idx, bar, sink, sms, rounds));
  printf("gather K=4 only         : %.2f us/round\n", run<4, true, false>(A, idx, bar, sink, sms, rounds));
  printf("gather K=4 + barrier    : %.2f us/round\n", run<4, true, true>(A, idx, bar, sink, sms, rounds));
  printf("gather K=8 only         : %.2f us/round\n", run<8, true, false>(A, idx, bar, sink, sms, rounds));
  printf("gather K=8 + barrier    : %.2f us/round\n", run<8, true, true>(A, idx, bar, sink, sms, rounds));
  printf("gather K=16 only        : %.2f us/round\n", run<16, true, false>(A, idx, bar, sink, sms, rounds));
  printf("barrier only, 16 CTAs   : %.2f us/round\n", run<4, false, true>(A, idx, bar, sink, 16, rounds));
  cudaError_t e = cudaGetLastError();
  printf("%s\n", cudaGetErrorString(e));
  return 0;
}
