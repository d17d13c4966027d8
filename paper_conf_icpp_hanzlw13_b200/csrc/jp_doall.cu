// jp_doall.cu -- DOALL kernels (loops "determined to be
// dependency-free during the static analysis phase or profiling phase could be
// safely parallelized without any software protection").
//
// k_doall_affine_vec: all index arrays NULL (the "determined DOALL" mode A of
//   P:L361-362; config 2).  Pure HBM streaming: 16-byte vector lanes, UNROLL
//   independent vectors in flight per thread, streaming cache hints
//   (ld.global.cs / st.global.cs: touched once), persistent grid sized to a
//   multiple of the SM count.  12 B/iteration for SAXPY (X 4 + Y 4 read, Y 4 written).
// k_doall_generic: indirect bodies (config 1 at 0%, the config-5 head):
//   coalesced index streams, gathered/scattered element accesses.
#include "jp_host.h"

namespace jp {

template <int OP, int DT>
__device__ __forceinline__ void vec_body(const uint4 &x, uint4 &a, uint4 &t, uint32_t c0, uint32_t c1) {
  uint32_t *pa = &a.x, *pt = &t.x;
  const uint32_t *px = &x.x;
#pragma unroll
  for (int k = 0; k < 4; k++) {
    if constexpr (OP == JP_OP_ADD_C) pa[k] = op_add<DT>(pa[k], c0);
    else if constexpr (OP == JP_OP_SAXPY) pa[k] = op_add<DT>(op_mul<DT>(c0, px[k]), pa[k]);
    else if constexpr (OP == JP_OP_PRIV_TMP) { pt[k] = op_mul<DT>(c0, px[k]); pa[k] = op_add<DT>(pt[k], c1); }
    else pa[k] = op_mul<DT>(op_add<DT>(pa[k], pa[k]), c0);
  }
}

constexpr int kAffUnroll = 4;
constexpr int kAffThreads = 256;

template <int OP, int DT>
__global__ void __launch_bounds__(kAffThreads) k_doall_affine_vec(DLoop L, int64_t nvec) {
  constexpr bool readsA = OP != JP_OP_PRIV_TMP;
  constexpr bool readsX = OP == JP_OP_SAXPY || OP == JP_OP_PRIV_TMP;
  const uint4 *X4 = reinterpret_cast<const uint4 *>(L.X);
  uint4 *A4 = reinterpret_cast<uint4 *>(L.A);
  uint4 *T4 = reinterpret_cast<uint4 *>(L.T);
  const int64_t step = (int64_t)gridDim.x * kAffThreads * kAffUnroll;
  for (int64_t v0 = (int64_t)blockIdx.x * kAffThreads * kAffUnroll + threadIdx.x; v0 < nvec; v0 += step) {
    uint4 a[kAffUnroll], x[kAffUnroll], t[kAffUnroll];
#pragma unroll
    for (int u = 0; u < kAffUnroll; u++) {
      const int64_t v = v0 + (int64_t)u * kAffThreads;
      if (v < nvec) {
        if constexpr (readsA) a[u] = __ldcs(A4 + v);
        if constexpr (readsX) x[u] = __ldcs(X4 + v);
      }
    }
#pragma unroll
    for (int u = 0; u < kAffUnroll; u++) {
      const int64_t v = v0 + (int64_t)u * kAffThreads;
      if (v < nvec) {
        vec_body<OP, DT>(x[u], a[u], t[u], L.c0, L.c1);
        __stcs(A4 + v, a[u]);
        if constexpr (OP == JP_OP_PRIV_TMP) __stcs(T4 + v, t[u]);
      }
    }
  }
  // scalar tail [4*nvec, n)
  if (blockIdx.x == 0) {
    for (int64_t i = 4 * nvec + threadIdx.x; i < L.n; i += kAffThreads) {
      uint32_t va = 0, vt = 0;
      body_values<OP, DT>(L, i, L.A, va, vt);
      if constexpr (OP == JP_OP_PRIV_TMP) L.T[i] = vt;
      L.A[i] = va;
    }
  }
}

template <int OP, int DT>
__global__ void __launch_bounds__(256) k_doall_generic(DLoop L) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < L.n; i += stride) {
    uint32_t va = 0, vt = 0;
    body_values<OP, DT>(L, i, L.A, va, vt);
    if constexpr (OP == JP_OP_PRIV_TMP) L.T[ixl(L, L.s, i)] = vt;
    L.A[ixl(L, L.w, i)] = va;
  }
}

static bool aligned16(const void *p) { return ((uintptr_t)p & 15) == 0; }

template <int OP, int DT>
static void run_doall(const DLoop &d, cudaStream_t st, int max_ctas) {
  const bool affine = !d.r && !d.r2 && !d.w && !d.s && d.ioff == 0;
  int sms = num_sms();
  if (affine && aligned16(d.A) && (!d.X || aligned16(d.X)) && (!d.T || aligned16(d.T))) {
    int64_t nvec = d.n / 4;
    int64_t need = (nvec + kAffThreads * kAffUnroll - 1) / (kAffThreads * kAffUnroll);
    int64_t cap = (int64_t)sms * 8;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
    k_doall_affine_vec<OP, DT><<<grid, kAffThreads, 0, st>>>(d, nvec);
  } else {
    int64_t need = (d.n + 255) / 256;
    int64_t cap = (int64_t)sms * 8;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
    k_doall_generic<OP, DT><<<grid, 256, 0, st>>>(d);
  }
  note_launch();
}

cudaError_t launch_doall(const Job &j, cudaStream_t st, int max_ctas) {
  if (j.d.n == 0) return cudaSuccess;
  JP_DISPATCH(j.op, j.dt, run_doall, j.d, st, max_ctas);
  return launch_check();
}

}  // namespace jp
