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
#include <atomic>
#include <chrono>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <vector>
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

// k_doall_affine_tma: the same affine loop staged through shared memory with
// bulk copies (cp.async.bulk, the TMA engine's 1-D mode): one CTA per SM, a
// kTmaStages-deep ring of 16 KiB tiles per stream, mbarrier completion for the
// loads (one elected thread arms expect_tx and issues both copies), the body
// computed in place in shared memory by all threads, then one bulk store per
// tile (bulk_group; a stage is reloaded once its store has finished reading).
// Measured against k_doall_affine_vec in DESIGN.md Sec.6 (the faster one is
// the default).
constexpr int kTmaTile = 4096;                 // elements per tile per stream (16 KiB)
constexpr int kTmaStages = 4;
constexpr int kTmaThreads = 256;

template <int OP, int DT>
__global__ void __launch_bounds__(kTmaThreads, 1) k_doall_affine_tma(DLoop L, int64_t ntiles) {
  constexpr bool readsA = OP != JP_OP_PRIV_TMP;
  constexpr bool readsX = OP == JP_OP_SAXPY || OP == JP_OP_PRIV_TMP;
  constexpr int NB = 2;   // buffers per stage: A (in/out) and X (PRIV_TMP: T out, X in)
  extern __shared__ __align__(128) uint32_t tsm[];   // [stage][NB][kTmaTile]
  __shared__ __align__(8) unsigned long long full[kTmaStages];
  const int tid = threadIdx.x;
  const uint32_t bytes_in = (uint32_t)(((readsA ? 1 : 0) + (readsX ? 1 : 0)) * kTmaTile * 4);
  // this CTA's tiles: t = blockIdx.x + k * gridDim.x
  const int64_t my = ntiles > blockIdx.x ? (ntiles - 1 - blockIdx.x) / gridDim.x + 1 : 0;
  auto tile_of = [&](int64_t k) { return (int64_t)blockIdx.x + k * gridDim.x; };
  auto issue = [&](int64_t k) {
    const int s = (int)(k % kTmaStages);
    const int64_t e0 = tile_of(k) * kTmaTile;
    uint32_t *bA = tsm + (size_t)s * NB * kTmaTile, *bX = bA + kTmaTile;
    mbar_expect_tx(&full[s], bytes_in);
    if constexpr (readsA) bulk_load(bA, L.A + e0, kTmaTile * 4, &full[s]);
    if constexpr (readsX) bulk_load(bX, L.X + e0, kTmaTile * 4, &full[s]);
  };
  if (tid == 0) {
    for (int s = 0; s < kTmaStages; s++) mbar_init(&full[s], 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  if (tid == 0)
    for (int64_t k = 0; k < kTmaStages - 1 && k < my; k++) issue(k);
  for (int64_t k = 0; k < my; k++) {
    const int s = (int)(k % kTmaStages);
    const uint32_t parity = (uint32_t)((k / kTmaStages) & 1);
    uint32_t *bA = tsm + (size_t)s * NB * kTmaTile, *bX = bA + kTmaTile;
    mbar_wait(&full[s], parity);
    uint4 *A4 = reinterpret_cast<uint4 *>(bA);
    uint4 *X4 = reinterpret_cast<uint4 *>(bX);
#pragma unroll
    for (int v = tid; v < kTmaTile / 4; v += kTmaThreads) {
      uint4 a = readsA ? A4[v] : make_uint4(0, 0, 0, 0), x = readsX ? X4[v] : make_uint4(0, 0, 0, 0), t;
      vec_body<OP, DT>(x, a, t, L.c0, L.c1);
      A4[v] = a;
      if constexpr (OP == JP_OP_PRIV_TMP) X4[v] = t;   // X is consumed: its buffer carries T out
    }
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");   // generic writes -> async proxy
    __syncthreads();
    if (tid == 0) {
      const int64_t e0 = tile_of(k) * kTmaTile;
      bulk_store(L.A + e0, bA, kTmaTile * 4);
      if constexpr (OP == JP_OP_PRIV_TMP) bulk_store(L.T + e0, bX, kTmaTile * 4);
      asm volatile("cp.async.bulk.commit_group;" ::: "memory");
      // refill the stage used one iteration ago once its store has read smem
      if (k + kTmaStages - 1 < my) {
        asm volatile("cp.async.bulk.wait_group.read 1;" ::: "memory");
        issue(k + kTmaStages - 1);
      }
    }
  }
  if (tid == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
  // element tail [ntiles * kTmaTile, n): CTA 0, plain accesses
  if (blockIdx.x == 0) {
    for (int64_t i = ntiles * kTmaTile + tid; i < L.n; i += kTmaThreads) {
      uint32_t va = 0, vt = 0;
      body_values<OP, DT>(L, i, L.A, va, vt);
      if constexpr (OP == JP_OP_PRIV_TMP) L.T[i] = vt;
      L.A[i] = va;
    }
  }
}

template <int OP, int DT>
__global__ void __launch_bounds__(256) k_doall_generic(DLoop L) {
  if (aborted(L)) return;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < L.n; i += stride) {
    uint32_t va = 0, vt = 0;
    body_values<OP, DT>(L, i, L.A, va, vt);
    if constexpr (OP == JP_OP_PRIV_TMP) L.T[ixl(L, L.s, i)] = vt;
    L.A[ixl(L, L.w, i)] = va;
  }
}

// k_doall_quad: the indirect DOALL body with more random accesses in flight --
// each thread takes two quads of 4 consecutive iterations per trip (16-byte
// index loads when aligned), issues all 8 iterations' gathers, then computes
// and scatters.  The loop carries no dependence (d_raw = d_war = d_waw = 0), so
// reading A in place and storing in any order is the sequential result.
__device__ __forceinline__ int4 q_idx(const DLoop &L, const int32_t *p, int64_t i, bool vec) {
  if (!p) {
    const int32_t b = (int32_t)(L.ioff + i);
    return make_int4(b, b + 1, b + 2, b + 3);
  }
  if (vec && i + 4 <= L.n) return __ldcs(reinterpret_cast<const int4 *>(p + i));
  int4 r;
  r.x = p[i];
  r.y = i + 1 < L.n ? p[i + 1] : 0;
  r.z = i + 2 < L.n ? p[i + 2] : 0;
  r.w = i + 3 < L.n ? p[i + 3] : 0;
  return r;
}
__device__ __forceinline__ int q_get(const int4 &v, int k) { return k == 0 ? v.x : k == 1 ? v.y : k == 2 ? v.z : v.w; }

template <int OP, int DT>
__global__ void __launch_bounds__(256) k_doall_quad(DLoop L, int vec) {
  if (aborted(L)) return;
  constexpr int Q = 2;   // quads per thread per trip
  const int64_t nq = (L.n + 3) >> 2, B = blockDim.x;
  for (int64_t q0 = (int64_t)blockIdx.x * B * Q + threadIdx.x; q0 < nq; q0 += (int64_t)gridDim.x * B * Q) {
    int4 ra[Q], wa[Q], xa[Q];
    uint32_t g0[Q][4], g1[Q][4];
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t q = q0 + u * B;
      if (q >= nq) continue;
      const int64_t i = q << 2;
      ra[u] = q_idx(L, L.r, i, vec);
      wa[u] = q_idx(L, L.w, i, vec);
      if constexpr (OP == JP_OP_STENCIL2) xa[u] = q_idx(L, L.r2, i, vec);
      if constexpr (OP == JP_OP_PRIV_TMP) xa[u] = q_idx(L, L.s, i, vec);
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {   // every gather of the trip issued before any use
      const int64_t q = q0 + u * B;
      if (q >= nq) continue;
      const int kn = L.n - (q << 2) < 4 ? (int)(L.n - (q << 2)) : 4;
#pragma unroll
      for (int k = 0; k < 4; k++) {
        if (k >= kn) break;
        if constexpr (OP == JP_OP_ADD_C) g0[u][k] = L.A[q_get(ra[u], k)];
        else if constexpr (OP == JP_OP_SAXPY) { g0[u][k] = L.X[q_get(ra[u], k)]; g1[u][k] = L.A[q_get(wa[u], k)]; }
        else if constexpr (OP == JP_OP_PRIV_TMP) g0[u][k] = L.X[q_get(ra[u], k)];
        else { g0[u][k] = L.A[q_get(ra[u], k)]; g1[u][k] = L.A[q_get(xa[u], k)]; }
      }
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t q = q0 + u * B;
      if (q >= nq) continue;
      const int kn = L.n - (q << 2) < 4 ? (int)(L.n - (q << 2)) : 4;
#pragma unroll
      for (int k = 0; k < 4; k++) {
        if (k >= kn) break;
        if constexpr (OP == JP_OP_ADD_C) L.A[q_get(wa[u], k)] = op_add<DT>(g0[u][k], L.c0);
        else if constexpr (OP == JP_OP_SAXPY) L.A[q_get(wa[u], k)] = op_add<DT>(op_mul<DT>(L.c0, g0[u][k]), g1[u][k]);
        else if constexpr (OP == JP_OP_PRIV_TMP) {
          const uint32_t t = op_mul<DT>(L.c0, g0[u][k]);
          L.T[q_get(xa[u], k)] = t;
          L.A[q_get(wa[u], k)] = op_add<DT>(t, L.c1);
        } else L.A[q_get(wa[u], k)] = op_mul<DT>(op_add<DT>(g0[u][k], g1[u][k]), L.c0);
      }
    }
  }
}

// Phased indirect DOALL: every iteration's value into a scratch array first (all
// the loop's random reads), then every scatter.  On B200 a random in-place update
// over an L2-resident A runs at 273-283 us for 2^24 iterations interleaved and
// at 192 us as a gather kernel then a scatter kernel (scripts/ubench/
// rand_phase.cu); the split is legal because a DOALL loop reads no element
// another iteration writes.  Not for PRIV_TMP (two outputs per iteration).
template <int OP, int DT>
__global__ void __launch_bounds__(256) k_doall_gath(DLoop L, uint32_t *o) {
  if (aborted(L)) return;
  constexpr int Q = 4;
  const int64_t G = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i0 = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i0 < L.n; i0 += G * Q) {
    int32_t ra[Q], wa[Q];
    uint32_t g0[Q], g1[Q];
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + u * G;
      if (i >= L.n) continue;
      ra[u] = L.r ? __ldcs(L.r + i) : (int32_t)(L.ioff + i);
      if constexpr (OP == JP_OP_SAXPY) wa[u] = L.w ? __ldcs(L.w + i) : (int32_t)(L.ioff + i);
      if constexpr (OP == JP_OP_STENCIL2) wa[u] = L.r2 ? __ldcs(L.r2 + i) : (int32_t)(L.ioff + i);
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + u * G;
      if (i >= L.n) continue;
      if constexpr (OP == JP_OP_ADD_C) g0[u] = __ldcg(L.A + ra[u]);
      else if constexpr (OP == JP_OP_SAXPY) { g0[u] = __ldcg(L.X + ra[u]); g1[u] = __ldcg(L.A + wa[u]); }
      else { g0[u] = __ldcg(L.A + ra[u]); g1[u] = __ldcg(L.A + wa[u]); }
    }
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + u * G;
      if (i >= L.n) continue;
      uint32_t v;
      if constexpr (OP == JP_OP_ADD_C) v = op_add<DT>(g0[u], L.c0);
      else if constexpr (OP == JP_OP_SAXPY) v = op_add<DT>(op_mul<DT>(L.c0, g0[u]), g1[u]);
      else v = op_mul<DT>(op_add<DT>(g0[u], g1[u]), L.c0);
      __stcs(o + i, v);
    }
  }
}
__global__ void __launch_bounds__(256) k_doall_scat(DLoop L, const uint32_t *o) {
  if (aborted(L)) return;
  constexpr int Q = 4;
  const int64_t G = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i0 = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i0 < L.n; i0 += G * Q) {
    int32_t wa[Q];
    uint32_t v[Q];
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + u * G;
      if (i >= L.n) continue;
      wa[u] = L.w ? __ldcs(L.w + i) : (int32_t)(L.ioff + i);
      v[u] = __ldcs(o + i);
    }
#pragma unroll
    for (int u = 0; u < Q; u++)
      if (i0 + u * G < L.n) __stcg(L.A + wa[u], v[u]);
  }
}

__host__ __device__ static inline bool aligned16(const void *p) { return ((uintptr_t)p & 15) == 0; }

// affine DOALL kernel choice (jp_doall_kernel): 0 LDG/STG.128 grid-stride, 1 bulk-copy (TMA) staged
// (default: config 2 measured 6.48 vs 6.25 TB/s)
static std::atomic<int> g_doall_kernel{-1};
int doall_kernel_choice() {
  int v = g_doall_kernel.load();
  if (v < 0) {
    const char *e = getenv("JP_DOALL_KERNEL");   // default: bulk-copy staged (measured faster)
    v = e && e[0] == '0' ? 0 : 1;
    g_doall_kernel.store(v);
  }
  return v;
}
void set_doall_kernel_choice(int v) { g_doall_kernel.store(v); }

template <int OP, int DT>
static void run_doall(const DLoop &d, cudaStream_t st, int max_ctas) {
  const bool affine = !d.r && !d.r2 && !d.w && !d.s && d.ioff == 0;
  int sms = num_sms();
  if (doall_kernel_choice() == 1 && affine && aligned16(d.A) && (!d.X || aligned16(d.X)) && (!d.T || aligned16(d.T))) {
    const int64_t ntiles = d.n / kTmaTile;
    const size_t smem = (size_t)kTmaStages * 2 * kTmaTile * 4;
    set_smem_once((const void *)k_doall_affine_tma<OP, DT>, (int)smem);
    int64_t cap = sms;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    const int grid = (int)(ntiles < 1 ? 1 : ntiles < cap ? ntiles : cap);
    k_doall_affine_tma<OP, DT><<<grid, kTmaThreads, smem, st>>>(d, ntiles);
  } else if (affine && aligned16(d.A) && (!d.X || aligned16(d.X)) && (!d.T || aligned16(d.T))) {
    int64_t nvec = d.n / 4;
    int64_t need = (nvec + kAffThreads * kAffUnroll - 1) / (kAffThreads * kAffUnroll);
    int64_t cap = (int64_t)sms * 8;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
    k_doall_affine_vec<OP, DT><<<grid, kAffThreads, 0, st>>>(d, nvec);
  } else if (!getenv("JP_DOALL_GENERIC")) {
    auto al = [](const int32_t *q) { return q == nullptr || ((uintptr_t)q & 15) == 0; };
    const int vec = al(d.r) && al(d.w) && al(d.r2) && al(d.s);
    int64_t need = ((d.n + 3) / 4 + 511) / 512;
    int64_t cap = (int64_t)sms * 8;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
    k_doall_quad<OP, DT><<<grid, 256, 0, st>>>(d, vec);
  } else {
    int64_t need = (d.n + 255) / 256;
    int64_t cap = (int64_t)sms * 8;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
    k_doall_generic<OP, DT><<<grid, 256, 0, st>>>(d);
  }
  note_launch();
}

// ---------------------------------------------------------------------------
// k_doall_spill: task sharing with cross-boundary spill (M1; C8).
// Every rank's range is cut into uniform chunks.  Rank k's chunk counter
// ctr[k] packs (tail claims << 32 | head claims); one system-scope 64-bit
// atomicAdd claims a chunk and sees both counts at once, so a chunk c is taken
// exactly once: the owner claims ascending (head h valid iff h + t < nch),
// an idle rank claims descending from the tail (chunk nch-1-t, same test).
// Once its own range is exhausted a CTA steals from the rank with the most
// unclaimed chunks, ties to the lowest rank (reading A18).  The views are the
// ranks' shards with pointers valid in this process (peer memory mapped over
// NVLink through CUDA IPC on a multi-GPU node), so a stolen chunk is read and
// written where it lives.
// ---------------------------------------------------------------------------
constexpr int kSpillMaxRanks = 8;
struct SpillArgs {
  DLoop v[kSpillMaxRanks];
  int64_t nch[kSpillMaxRanks];
  unsigned long long *ctr;
  int64_t *stats;   // [0] own iterations, [1] stolen iterations, [2] stolen chunks (this executor)
  int64_t chunk;
  int world, me;
};

__device__ __forceinline__ bool spill_claim(unsigned long long *ctr, int64_t nch, bool tail, int64_t &c) {
  const unsigned long long old = atomicAdd_system(ctr, tail ? (1ull << 32) : 1ull);
  const int64_t h = (uint32_t)old, t = (uint32_t)(old >> 32);
  if (h + t >= nch) return false;
  c = tail ? nch - 1 - t : h;
  return true;
}

template <int OP, int DT>
__device__ __forceinline__ void spill_chunk(const DLoop &L, int64_t s, int64_t e) {
  constexpr bool readsA = OP != JP_OP_PRIV_TMP;
  constexpr bool readsX = OP == JP_OP_SAXPY || OP == JP_OP_PRIV_TMP;
  int64_t v_end = 0;
  if (aligned16(L.A + s) && (!readsX || aligned16(L.X + s)) && (OP != JP_OP_PRIV_TMP || aligned16(L.T + s))) {
    const int64_t nvec = (e - s) >> 2;
    v_end = nvec << 2;
    const uint4 *X4 = reinterpret_cast<const uint4 *>(L.X + s);
    uint4 *A4 = reinterpret_cast<uint4 *>(L.A + s);
    uint4 *T4 = reinterpret_cast<uint4 *>(L.T + s);
    for (int64_t v0 = threadIdx.x; v0 < nvec; v0 += kAffThreads * kAffUnroll) {
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
  }
  for (int64_t i = s + v_end + threadIdx.x; i < e; i += kAffThreads) {
    uint32_t va = 0, vt = 0;
    body_values<OP, DT>(L, i, L.A, va, vt);
    if constexpr (OP == JP_OP_PRIV_TMP) L.T[i] = vt;
    L.A[i] = va;
  }
}

template <int OP, int DT>
__global__ void __launch_bounds__(kAffThreads) k_doall_spill(const __grid_constant__ SpillArgs P) {
  __shared__ int s_rank;
  __shared__ long long s_chunk;
  int64_t own = 0, stolen = 0, nst = 0;
  bool mine = true;
  for (;;) {
    if (threadIdx.x == 0) {
      int rk = -1;
      int64_t c = 0;
      if (mine && spill_claim(&P.ctr[P.me], P.nch[P.me], false, c)) rk = P.me;
      else mine = false;
      while (rk < 0) {   // steal: the rank with the most unclaimed chunks, ties to the lowest
        int best = -1;
        int64_t most = 0;
        for (int k = 0; k < P.world; k++) {
          if (k == P.me) continue;
          const unsigned long long v = *(volatile unsigned long long *)&P.ctr[k];
          const int64_t left = P.nch[k] - (int64_t)(uint32_t)v - (int64_t)(uint32_t)(v >> 32);
          if (left > most) { most = left; best = k; }
        }
        if (best < 0) break;
        if (spill_claim(&P.ctr[best], P.nch[best], true, c)) rk = best;
      }
      s_rank = rk;
      s_chunk = c;
    }
    __syncthreads();
    const int rk = s_rank;
    const int64_t c = s_chunk;
    __syncthreads();
    if (rk < 0) break;
    const DLoop &L = P.v[rk];
    const int64_t s = c * P.chunk, e = s + P.chunk < L.n ? s + P.chunk : L.n;
    spill_chunk<OP, DT>(L, s, e);
    if (threadIdx.x == 0) {
      if (rk == P.me) own += e - s;
      else { stolen += e - s; nst++; }
    }
  }
  if (threadIdx.x == 0 && P.stats) {
    if (own) atomicAdd(reinterpret_cast<unsigned long long *>(&P.stats[0]), (unsigned long long)own);
    if (stolen) {
      atomicAdd(reinterpret_cast<unsigned long long *>(&P.stats[1]), (unsigned long long)stolen);
      atomicAdd(reinterpret_cast<unsigned long long *>(&P.stats[2]), (unsigned long long)nst);
    }
  }
}

template <int OP, int DT>
static void run_spill(const SpillArgs &P, int grid, cudaStream_t st) {
  k_doall_spill<OP, DT><<<grid, kAffThreads, 0, st>>>(P);
  note_launch();
}

cudaError_t launch_doall_spill(const Job *views, int world, int me, int64_t chunk, unsigned long long *ctr,
                               int64_t *stats, int max_ctas, cudaStream_t st) {
  SpillArgs P;
  memset(&P, 0, sizeof P);
  for (int k = 0; k < world; k++) {
    P.v[k] = views[k].d;
    P.nch[k] = (views[k].d.n + chunk - 1) / chunk;
  }
  P.ctr = ctr;
  P.stats = stats;
  P.chunk = chunk;
  P.world = world;
  P.me = me;
  int grid = num_sms() * 4;   // 256-thread CTAs, 4 per SM resident
  if (max_ctas > 0 && grid > max_ctas) grid = max_ctas;
  JP_DISPATCH(views[0].op, views[0].dt, run_spill, P, grid, st);
  return launch_check();
}

template <int OP, int DT>
static void run_doall_phased(const DLoop &d, uint32_t *o, cudaStream_t st, int max_ctas) {
  if constexpr (OP == JP_OP_PRIV_TMP) {
    run_doall<OP, DT>(d, st, max_ctas);
  } else {
    int64_t cap = (int64_t)num_sms() * 8;
    if (max_ctas > 0 && cap > max_ctas) cap = max_ctas;
    const int64_t need = (d.n + 255) / 256;
    const int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
    k_doall_gath<OP, DT><<<grid, 256, 0, st>>>(d, o);
    k_doall_scat<<<grid, 256, 0, st>>>(d, o);
    note_launch(2);
  }
}

cudaError_t launch_doall(const Job &j, cudaStream_t st, int max_ctas, uint32_t *o) {
  if (j.d.n == 0) return cudaSuccess;
  const bool affine = !j.d.r && !j.d.r2 && !j.d.w && !j.d.s;
  const char *e = getenv("JP_DOALL_PHASED");
  if (o && !affine && j.op != JP_OP_PRIV_TMP && !(e && e[0] == '0')) {
    JP_DISPATCH(j.op, j.dt, run_doall_phased, j.d, o, st, max_ctas);
  } else {
    JP_DISPATCH(j.op, j.dt, run_doall, j.d, st, max_ctas);
  }
  return launch_check();
}

}  // namespace jp
