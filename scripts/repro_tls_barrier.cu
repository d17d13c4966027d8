// Stand-alone reproduction of the TLS CTA barrier finding.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -DV_BAR=0 -DV_C=0 -DV_RESET_START=0 -DV_EARLY=1 -DV_REDUX=1 -o r0 repro_tls_barrier.cu  -> fails intermittently
// same with -DV_BAR=2 (explicit barrier.sync + memory clobber)                                             -> 0/40 failures

// Minimal CTA-TLS kernel for bisecting; same harness/data as h5.
#include <cstdio>
#include <cstdint>
#include <vector>
#include <algorithm>
#include <random>
#if V_BAR == 1
#define SYNC() do { if (__syncthreads_or(0)) asm volatile("trap;"); } while (0)
#elif V_BAR == 2
#define SYNC() asm volatile("barrier.sync 0;" ::: "memory")
#else
#define SYNC() __syncthreads()
#endif
constexpr int LOG = 13, H = 1 << LOG, T = 1024, IPT = 4;
constexpr uint32_t E = 0xFFFFFFFFu;
__device__ __forceinline__ uint32_t home(uint32_t k) { return (k * 0x9E3779B1u) >> (32 - LOG); }
__device__ __forceinline__ int hins(uint32_t* hk, uint32_t* hmin, uint32_t key, uint32_t off) {
  uint32_t h = home(key);
  while (true) { uint32_t p = atomicCAS(&hk[h], E, key); if (p == E || p == key) break; h = (h + 1) & (H - 1); }
  atomicMin(&hmin[h], off); return h;
}
__device__ __forceinline__ int hfind(const uint32_t* hk, uint32_t key) {
  uint32_t h = home(key);
  while (true) { uint32_t k = hk[h]; if (k == key) return h; if (k == E) return -1; h = (h + 1) & (H - 1); }
}
struct Args { long n; const int *r, *w; uint32_t* A; int W; };
__global__ void __launch_bounds__(T, 1) kern(Args a, long long* st) {
  extern __shared__ uint32_t sm[];
  uint32_t *hk0 = sm, *hmin0 = sm + H;
  __shared__ int s_fv[2];
  for (int k = threadIdx.x; k < (V_C == 1 ? 2 : 1) * H; k += T) { sm[k] = E; sm[k + (V_C == 1 ? 2 : 1) * H] = E; }
  if (threadIdx.x == 0) { s_fv[0] = s_fv[1] = INT32_MAX; }
  SYNC();
  long ws = 0; long long windows = 0; int par = 0;
  while (ws < a.n) {
    const int span = (int)min((long)a.W, a.n - ws);
#if V_RESET_START
    if (threadIdx.x == 0) s_fv[par] = INT32_MAX;
    SYNC();
#else
    if (threadIdx.x == 0) s_fv[par ^ 1] = INT32_MAX;
#endif
    uint32_t *hk = hk0, *hmin = hmin0;
    if (V_C == 1) { hk = sm + (windows & 1) * H; hmin = sm + 2 * H + (windows & 1) * H; }
    int sl[IPT], ra[IPT], wa[IPT]; uint32_t va[IPT];
#pragma unroll
    for (int k = 0; k < IPT; k++) {
      int off = k * T + threadIdx.x;
      if (off < span) { long i = ws + off; ra[k] = a.r[i]; wa[k] = a.w[i]; va[k] = a.A[ra[k]] + 7u; sl[k] = hins(hk, hmin, (uint32_t)wa[k] << 1, off); }
    }
    SYNC();
    int my = INT32_MAX;
#pragma unroll
    for (int k = 0; k < IPT; k++) {
      int off = k * T + threadIdx.x;
#if V_EARLY
      if (off < span && my == INT32_MAX) {
        int h = hfind(hk, (uint32_t)ra[k] << 1);
        if (h >= 0 && hmin[h] < (uint32_t)off) my = off;
      }
#else
      if (off < span) {
        int h = hfind(hk, (uint32_t)ra[k] << 1);
        if (my == INT32_MAX && h >= 0 && hmin[h] < (uint32_t)off) my = off;
      }
#endif
    }
#if V_REDUX
    my = __reduce_min_sync(0xffffffffu, my);
    if ((threadIdx.x & 31) == 0 && my != INT32_MAX) atomicMin(&s_fv[par], my);
#else
    atomicMin(&s_fv[par], my);
#endif
    SYNC();
    const int fv = min(s_fv[par], span);
#pragma unroll
    for (int k = 0; k < IPT; k++) {
      int off = k * T + threadIdx.x;
      if (off < fv) a.A[wa[k]] = va[k];
    }
#pragma unroll
    for (int k = 0; k < IPT; k++) {
      int off = k * T + threadIdx.x;
      if (off < span) { hk[sl[k]] = E; hmin[sl[k]] = E; }
    }
    if (V_C == 2) __threadfence_block();
    windows++; ws += fv; par ^= 1;
    SYNC();
  }
  if (threadIdx.x == 0) st[0] = windows;
}
int main() {
  long n = 131083; double d = 0.1; int W = 4096;
  std::mt19937_64 g(7);
  std::vector<int> w(n), r(n); std::vector<uint32_t> A(n), S(n);
  for (long i = 0; i < n; i++) { w[i] = i; A[i] = g() & 0xFFFFF; }
  std::shuffle(w.begin(), w.end(), g);
  for (long i = 0; i < n; i++) r[i] = w[i];
  for (long i = 1; i < n; i++) if (std::uniform_real_distribution<double>(0, 1)(g) < d) { long dl = 1 + g() % std::min<long>(i, 1024); r[i] = w[i - dl]; }
  S = A; for (long i = 0; i < n; i++) S[w[i]] = S[r[i]] + 7u;
  int *dr, *dw; uint32_t* dA; long long* st;
  cudaMalloc(&dr, n * 4); cudaMalloc(&dw, n * 4); cudaMalloc(&dA, n * 4); cudaMalloc(&st, 64);
  cudaMemcpy(dr, r.data(), n * 4, cudaMemcpyHostToDevice); cudaMemcpy(dw, w.data(), n * 4, cudaMemcpyHostToDevice);
  size_t smem = (V_C == 1 ? 4 : 2) * H * 4;
  cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  int fails = 0;
  for (int rep = 0; rep < 20; rep++) {
    cudaMemcpy(dA, A.data(), n * 4, cudaMemcpyHostToDevice);
    kern<<<1, T, smem>>>(Args{n, dr, dw, dA, W}, st);
    long long h; cudaMemcpy(&h, st, 8, cudaMemcpyDeviceToHost);
    std::vector<uint32_t> G(n); cudaMemcpy(G.data(), dA, n * 4, cudaMemcpyDeviceToHost);
    long bad = 0; for (long i = 0; i < n; i++) bad += G[i] != S[i];
    if (bad || h != 1035) { fails++; printf("  rep %d windows=%lld badA=%ld\n", rep, h, bad); }
  }
  printf("BAR=%d C=%d RESET_START=%d EARLY=%d REDUX=%d fails=%d/20 (%s)\n", V_BAR, V_C, V_RESET_START, V_EARLY, V_REDUX, fails, cudaGetErrorString(cudaGetLastError()));
}
