// jp_sched.cu -- inter-task dependence for the task-stealing scheme (Sec. V.B,
// "Inter-loop dependencies are analyzed to compose the PDG ... the
// task scheduler gets a batch of data-independent tasks from the pool by
// topological sort").  Here a task is a maximal run of same-mode chunks of one
// loop (reading A19); two tasks depend on each other iff they touch a common
// address and at least one of them writes it (RAW, WAR or WAW at element
// granularity).  Exact for up to 64 tasks: every address carries a 64-bit
// write mask and read mask of the tasks touching it.
#include "jp_host.h"

namespace jp {

// only addresses in the pass's window [lo, lo + span): mask tables larger than
// L2 are built in several passes, each with an L2-resident working set
__device__ __forceinline__ void setbit(unsigned long long *m, int64_t a, unsigned long long b, uint32_t lo,
                                       uint32_t span) {
  if (m && (uint32_t)a - lo < span && (m[a] & b) == 0) atomicOr(&m[a], b);   // check first: most addresses see one task
}
// byte masks (<= 8 tasks): the mask of address a is byte a & 3 of 32-bit word a >> 2
__device__ __forceinline__ void setbit8(unsigned long long *m, int64_t a, unsigned long long b, uint32_t lo,
                                        uint32_t span) {
  if (!m || (uint32_t)a - lo >= span) return;
  uint32_t *w = reinterpret_cast<uint32_t *>(m) + (a >> 2);
  const uint32_t bb = (uint32_t)b << (8 * (a & 3));
  if ((*w & bb) == 0) atomicOr(w, bb);
}
__device__ __forceinline__ unsigned long long getmask8(const unsigned long long *m, int64_t a) {
  return (reinterpret_cast<const uint32_t *>(m)[a >> 2] >> (8 * (a & 3))) & 0xFFu;
}

// index of 4 consecutive local iterations (one 16-byte load when aligned)
__device__ __forceinline__ int4 tm_idx4(const DLoop &L, const int32_t *p, int64_t i, bool vec) {
  if (!p) {
    const int b = (int)(L.ioff + i);
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
__device__ __forceinline__ int tm_q4(const int4 &v, int k) { return k == 0 ? v.x : k == 1 ? v.y : k == 2 ? v.z : v.w; }

// 4 consecutive iterations per thread (chunk_iters is a multiple of 32, so a
// quad never straddles two tasks), 32-bit index math
template <int OP, bool B8>
__global__ void __launch_bounds__(256) k_task_masks(DLoop L, const int32_t *chunk_task, uint32_t chunk,
                                                    unsigned long long *wmA, unsigned long long *rmA,
                                                    unsigned long long *wmT, unsigned long long *rmT, uint32_t lo,
                                                    uint32_t span, int vec) {
  const int64_t nq = (L.n + 3) >> 2;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t q = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; q < nq; q += stride) {
    const int64_t i = q << 2;
    const unsigned long long b = 1ull << chunk_task[(uint32_t)i / chunk];
    const int kn = L.n - i < 4 ? (int)(L.n - i) : 4;
    auto setbit = [&](unsigned long long *m, int32_t a) {
      if constexpr (B8) setbit8(m, a, b, lo, span); else jp::setbit(m, a, b, lo, span);
    };
    if constexpr (OP == JP_OP_ADD_C) {
      const int4 w = tm_idx4(L, L.w, i, vec), r = tm_idx4(L, L.r, i, vec);
      for (int k = 0; k < kn; k++) { setbit(wmA, tm_q4(w, k)); setbit(rmA, tm_q4(r, k)); }
    } else if constexpr (OP == JP_OP_SAXPY) {
      const int4 w = tm_idx4(L, L.w, i, vec);
      for (int k = 0; k < kn; k++) { setbit(wmA, tm_q4(w, k)); setbit(rmA, tm_q4(w, k)); }
    } else if constexpr (OP == JP_OP_PRIV_TMP) {
      const int4 sv = tm_idx4(L, L.s, i, vec), w = tm_idx4(L, L.w, i, vec);
      for (int k = 0; k < kn; k++) { setbit(wmT, tm_q4(sv, k)); setbit(rmT, tm_q4(sv, k)); setbit(wmA, tm_q4(w, k)); }
    } else {
      const int4 w = tm_idx4(L, L.w, i, vec), r = tm_idx4(L, L.r, i, vec), r2 = tm_idx4(L, L.r2, i, vec);
      for (int k = 0; k < kn; k++) { setbit(wmA, tm_q4(w, k)); setbit(rmA, tm_q4(r, k)); setbit(rmA, tm_q4(r2, k)); }
    }
  }
}

template <bool B8>
__global__ void __launch_bounds__(256) k_task_conf(const unsigned long long *wm, const unsigned long long *rm,
                                                   int64_t len, unsigned long long *conf) {
  __shared__ unsigned long long sc[kMaxTasks];
  if (threadIdx.x < kMaxTasks) sc[threadIdx.x] = 0;
  JP_CTA_SYNC();
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t a = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; a < len; a += stride) {
    const unsigned long long mw = B8 ? getmask8(wm, a) : wm[a], mr = rm ? (B8 ? getmask8(rm, a) : rm[a]) : 0ull,
                             all = mw | mr;
    if (mw && (all & (all - 1))) {
      unsigned long long rest = all;
      while (rest) {
        const int t = __ffsll((long long)rest) - 1;
        rest &= rest - 1;
        const unsigned long long c = (((mw >> t) & 1ull) ? all : mw) & ~(1ull << t);
        if (c && (sc[t] & c) != c) atomicOr(&sc[t], c);
      }
    }
  }
  JP_CTA_SYNC();
  if (threadIdx.x < kMaxTasks && sc[threadIdx.x]) atomicOr(&conf[threadIdx.x], sc[threadIdx.x]);
}

// Address range of every task per array (A, T): [min, max] over the elements
// its iterations touch.  Tasks whose ranges are disjoint in every array cannot
// touch a common address, so when no two ranges overlap the task PDG has no
// edge and the per-address masks pass is skipped (one streaming pass over the
// index arrays instead of two random atomics per access).  A warp's 32
// iterations lie in one chunk (chunk % 32 == 0), hence in one task.
template <int OP>
__global__ void __launch_bounds__(256) k_task_ranges(DLoop L, const int32_t *ct, uint32_t chunk, uint32_t *rg) {
  __shared__ uint32_t s[4][kMaxTasks];   // minA, maxA, minT, maxT
  for (int t = threadIdx.x; t < kMaxTasks; t += blockDim.x) {
    s[0][t] = s[2][t] = 0xFFFFFFFFu;
    s[1][t] = s[3][t] = 0u;
  }
  __syncthreads();
  const int lane = threadIdx.x & 31;
  // each warp streams a contiguous run of 32-iteration tiles, keeping its
  // min / max in registers while the task stays the same (one warp reduction
  // per task change instead of one per tile)
  const int64_t tiles = (L.n + 31) / 32, nw = (int64_t)gridDim.x * (blockDim.x >> 5);
  const int64_t wg = (int64_t)blockIdx.x * (blockDim.x >> 5) + (threadIdx.x >> 5);
  const int64_t t0 = tiles * wg / nw, t1 = tiles * (wg + 1) / nw;
  uint32_t amin = 0xFFFFFFFFu, amax = 0u, tmin = 0xFFFFFFFFu, tmax = 0u;
  int cur = t0 < t1 ? ct[(t0 * 32) / chunk] : -1;
  auto flush = [&]() {
    const uint32_t a0 = __reduce_min_sync(0xffffffffu, amin), a1 = __reduce_max_sync(0xffffffffu, amax);
    const uint32_t b0 = __reduce_min_sync(0xffffffffu, tmin), b1 = __reduce_max_sync(0xffffffffu, tmax);
    if (lane == 0 && cur >= 0) {
      atomicMin(&s[0][cur], a0); atomicMax(&s[1][cur], a1);
      atomicMin(&s[2][cur], b0); atomicMax(&s[3][cur], b1);
    }
    amin = tmin = 0xFFFFFFFFu;
    amax = tmax = 0u;
  };
  constexpr int U = 8;   // tiles whose loads are in flight together
  auto tile_acc = [&](int64_t tile0, int nt) {
    uint32_t w[U], r[U], x[U];
#pragma unroll
    for (int u = 0; u < U; u++) {   // all loads first
      const int64_t i = (tile0 + u) * 32 + lane;
      w[u] = r[u] = x[u] = 0;
      if (u < nt && i < L.n) {
        w[u] = (uint32_t)ixl(L, L.w, i);
        if constexpr (OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2) r[u] = (uint32_t)ixl(L, L.r, i);
        if constexpr (OP == JP_OP_STENCIL2 || OP == JP_OP_PRIV_TMP)
          x[u] = (uint32_t)ixl(L, OP == JP_OP_STENCIL2 ? L.r2 : L.s, i);
      }
    }
#pragma unroll
    for (int u = 0; u < U; u++) {
      const int64_t i = (tile0 + u) * 32 + lane;
      if (u < nt && i < L.n) {
        amin = min(amin, w[u]); amax = max(amax, w[u]);
        if constexpr (OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2) { amin = min(amin, r[u]); amax = max(amax, r[u]); }
        if constexpr (OP == JP_OP_STENCIL2) { amin = min(amin, x[u]); amax = max(amax, x[u]); }
        if constexpr (OP == JP_OP_PRIV_TMP) { tmin = min(tmin, x[u]); tmax = max(tmax, x[u]); }
      }
    }
  };
  for (int64_t tile = t0; tile < t1;) {
    const int task = ct[(tile * 32) / chunk];   // warp-uniform (chunk % 32 == 0)
    if (task != cur) { flush(); cur = task; }
    // U tiles at once when they all lie in this task (tasks are runs of chunks)
    int nt = 1;
    if (tile + U <= t1 && ct[((tile + U - 1) * 32) / chunk] == task) nt = U;
    tile_acc(tile, nt);
    tile += nt;
  }
  flush();
  __syncthreads();
  for (int t = threadIdx.x; t < kMaxTasks; t += blockDim.x) {
    if (s[0][t] != 0xFFFFFFFFu) { atomicMin(&rg[t], s[0][t]); atomicMax(&rg[kMaxTasks + t], s[1][t]); }
    if (s[2][t] != 0xFFFFFFFFu) { atomicMin(&rg[2 * kMaxTasks + t], s[2][t]); atomicMax(&rg[3 * kMaxTasks + t], s[3][t]); }
  }
}

template <int OP, int DT>
static void run_ranges(const DLoop &d, const int32_t *ct, int64_t chunk, uint32_t *rg, cudaStream_t st) {
  (void)DT;
  int64_t need = (d.n + 255) / 256, cap = (int64_t)num_sms() * 8;
  k_task_ranges<OP><<<(int)(need < cap ? (need < 1 ? 1 : need) : cap), 256, 0, st>>>(d, ct, (uint32_t)chunk, rg);
  note_launch();
}

cudaError_t launch_task_ranges(const Job &j, const int32_t *chunk_task, int64_t chunk, uint32_t *rg, cudaStream_t st) {
  cudaMemsetAsync(rg, 0xFF, 4 * kMaxTasks, st);
  cudaMemsetAsync(rg + kMaxTasks, 0, 4 * kMaxTasks, st);
  cudaMemsetAsync(rg + 2 * kMaxTasks, 0xFF, 4 * kMaxTasks, st);
  cudaMemsetAsync(rg + 3 * kMaxTasks, 0, 4 * kMaxTasks, st);
  if (j.d.n == 0) return launch_check();
  JP_DISPATCH(j.op, j.dt, run_ranges, j.d, chunk_task, chunk, rg, st);
  return launch_check();
}

template <int OP, int DT>
static void run_masks(const DLoop &d, const int32_t *ct, int64_t chunk, unsigned long long *wmA,
                      unsigned long long *rmA, unsigned long long *wmT, unsigned long long *rmT, bool b8,
                      cudaStream_t st) {
  (void)DT;
  int64_t need = ((d.n + 3) / 4 + 255) / 256, cap = (int64_t)num_sms() * 8;
  auto al = [](const int32_t *q) { return q == nullptr || ((uintptr_t)q & 15) == 0; };
  const int vec = al(d.r) && al(d.w) && al(d.r2) && al(d.s);
  // ~48 MB of mask tables per pass (a third of L2)
  const int64_t bytes = (b8 ? 1 : 8) * ((wmA ? d.lenA : 0) + (rmA ? d.lenA : 0) + (wmT ? d.lenT : 0) + (rmT ? d.lenT : 0));
  const int np = (int)((bytes + (48ll << 20) - 1) / (48ll << 20));
  const int64_t amax = d.lenA > d.lenT ? d.lenA : d.lenT;
  const int64_t step = np > 1 ? (amax + np - 1) / np : 0;
  for (int p = 0; p < (np > 1 ? np : 1); p++) {
    const uint32_t lo = np > 1 ? (uint32_t)(p * step) : 0u, span = np > 1 ? (uint32_t)step : 0xFFFFFFFFu;
    const int g = (int)(need < cap ? (need < 1 ? 1 : need) : cap);
    if (b8) k_task_masks<OP, true><<<g, 256, 0, st>>>(d, ct, (uint32_t)chunk, wmA, rmA, wmT, rmT, lo, span, vec);
    else k_task_masks<OP, false><<<g, 256, 0, st>>>(d, ct, (uint32_t)chunk, wmA, rmA, wmT, rmT, lo, span, vec);
    note_launch();
  }
}

static void run_conf(const unsigned long long *wm, const unsigned long long *rm, int64_t len,
                     unsigned long long *conf, bool b8, cudaStream_t st) {
  if (!wm || !len) return;
  int64_t need = (len + 255) / 256, cap = (int64_t)num_sms() * 8;
  if (b8) k_task_conf<true><<<(int)(need < cap ? need : cap), 256, 0, st>>>(wm, rm, len, conf);
  else k_task_conf<false><<<(int)(need < cap ? need : cap), 256, 0, st>>>(wm, rm, len, conf);
  note_launch();
}

cudaError_t launch_task_conflicts(const Job &j, const int32_t *chunk_task, int64_t chunk, int n_tasks,
                                  unsigned long long *wmA, unsigned long long *rmA, unsigned long long *wmT,
                                  unsigned long long *rmT, unsigned long long *conf, cudaStream_t st) {
  // <= 8 tasks: one byte of mask per address (a single L2-resident pass for
  // tens of millions of addresses); else 64-bit masks
  const bool b8 = n_tasks <= 8;
  const size_t mb = b8 ? 1 : 8;
  if (wmA) cudaMemsetAsync(wmA, 0, mb * j.d.lenA + 4, st);
  if (rmA) cudaMemsetAsync(rmA, 0, mb * j.d.lenA + 4, st);
  if (wmT) cudaMemsetAsync(wmT, 0, mb * j.d.lenT + 4, st);
  if (rmT) cudaMemsetAsync(rmT, 0, mb * j.d.lenT + 4, st);
  cudaMemsetAsync(conf, 0, 8 * kMaxTasks, st);
  if (j.d.n == 0) return launch_check();
  JP_DISPATCH(j.op, j.dt, run_masks, j.d, chunk_task, chunk, wmA, rmA, wmT, rmT, b8, st);
  run_conf(wmA, rmA, j.d.lenA, conf, b8, st);
  run_conf(wmT, rmT, j.d.lenT, conf, b8, st);
  return launch_check();
}

}  // namespace jp
