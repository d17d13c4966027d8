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

__device__ __forceinline__ void setbit(unsigned long long *m, int64_t a, unsigned long long b) {
  if (m && (m[a] & b) == 0) atomicOr(&m[a], b);   // check first: most addresses see one task
}

template <int OP>
__global__ void __launch_bounds__(256) k_task_masks(DLoop L, const int32_t *chunk_task, int64_t chunk,
                                                    unsigned long long *wmA, unsigned long long *rmA,
                                                    unsigned long long *wmT, unsigned long long *rmT) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < L.n; i += stride) {
    const unsigned long long b = 1ull << chunk_task[i / chunk];
    if constexpr (OP == JP_OP_ADD_C) {
      setbit(wmA, ixl(L, L.w, i), b);
      setbit(rmA, ixl(L, L.r, i), b);
    } else if constexpr (OP == JP_OP_SAXPY) {
      const int64_t a = ixl(L, L.w, i);
      setbit(wmA, a, b);
      setbit(rmA, a, b);
    } else if constexpr (OP == JP_OP_PRIV_TMP) {
      const int64_t t = ixl(L, L.s, i);
      setbit(wmT, t, b);
      setbit(rmT, t, b);
      setbit(wmA, ixl(L, L.w, i), b);
    } else {
      setbit(wmA, ixl(L, L.w, i), b);
      setbit(rmA, ixl(L, L.r, i), b);
      setbit(rmA, ixl(L, L.r2, i), b);
    }
  }
}

__global__ void __launch_bounds__(256) k_task_conf(const unsigned long long *wm, const unsigned long long *rm,
                                                   int64_t len, unsigned long long *conf) {
  __shared__ unsigned long long sc[kMaxTasks];
  if (threadIdx.x < kMaxTasks) sc[threadIdx.x] = 0;
  JP_CTA_SYNC();
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t a = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; a < len; a += stride) {
    const unsigned long long mw = wm[a], mr = rm ? rm[a] : 0ull, all = mw | mr;
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

template <int OP, int DT>
static void run_masks(const DLoop &d, const int32_t *ct, int64_t chunk, unsigned long long *wmA,
                      unsigned long long *rmA, unsigned long long *wmT, unsigned long long *rmT, cudaStream_t st) {
  (void)DT;
  int64_t need = (d.n + 255) / 256, cap = (int64_t)num_sms() * 8;
  k_task_masks<OP><<<(int)(need < cap ? (need < 1 ? 1 : need) : cap), 256, 0, st>>>(d, ct, chunk, wmA, rmA, wmT, rmT);
  note_launch();
}

static void run_conf(const unsigned long long *wm, const unsigned long long *rm, int64_t len,
                     unsigned long long *conf, cudaStream_t st) {
  if (!wm || !len) return;
  int64_t need = (len + 255) / 256, cap = (int64_t)num_sms() * 8;
  k_task_conf<<<(int)(need < cap ? need : cap), 256, 0, st>>>(wm, rm, len, conf);
  note_launch();
}

cudaError_t launch_task_conflicts(const Job &j, const int32_t *chunk_task, int64_t chunk, unsigned long long *wmA,
                                  unsigned long long *rmA, unsigned long long *wmT, unsigned long long *rmT,
                                  unsigned long long *conf, cudaStream_t st) {
  if (wmA) cudaMemsetAsync(wmA, 0, 8 * j.d.lenA, st);
  if (rmA) cudaMemsetAsync(rmA, 0, 8 * j.d.lenA, st);
  if (wmT) cudaMemsetAsync(wmT, 0, 8 * j.d.lenT, st);
  if (rmT) cudaMemsetAsync(rmT, 0, 8 * j.d.lenT, st);
  cudaMemsetAsync(conf, 0, 8 * kMaxTasks, st);
  if (j.d.n == 0) return launch_check();
  JP_DISPATCH(j.op, j.dt, run_masks, j.d, chunk_task, chunk, wmA, rmA, wmT, rmT, st);
  run_conf(wmA, rmA, j.d.lenA, conf, st);
  run_conf(wmT, rmT, j.d.lenT, conf, st);
  return launch_check();
}

}  // namespace jp
