// jp_serial.cu -- mode C on the device: the loop run in program order by one
// warp (second half).
//
// Fig. 2(b) sends a loop whose true-dependence density is high to sequential
// execution ("high TD density -> dispatched to CPU"; P:L370-373:
// warps whose profile shows TD run "on CPU sequentially").  There is no CPU
// path here (north_star): a single warp executes the iteration space in
// batches of 32 consecutive iterations, exactly in program order:
//   * in-batch RAW: lane j's exposed A read takes the value of the LATEST
//     earlier lane k < j that writes the same element (32 shuffle rounds find
//     it), resolved in dependence order: one-source bodies (ADD_C, SAXPY) get
//     their depth by pointer jumping and run max-depth + 1 vote-free shuffle
//     rounds; STENCIL2 (two sources) polls readiness one round per link;
//   * in-batch WAW: only the last writer of an element stores it
//     (__match_any_sync groups, highest lane);
//   * the next batch's operands (and the indices of the batch after it) are
//     loaded before this batch stores (latency hidden behind the resolve),
//     then patched from this batch's writes (same shuffle compare), so every
//     read sees the value the sequential loop would see.
// Speculation never fails, so nothing is re-executed; stats report windows =
// batches and violations = in-batch RAW reads that were forwarded.
#include "jp_host.h"

namespace jp {

namespace {
constexpr unsigned kFull = 0xffffffffu;

template <int OP>
struct SerBatch {
  int32_t ra, wa, xa;   // read / write / (r2 | s) element, -1 when the lane is past n
  uint32_t o0, o1;      // exposed operands
};

// indices of iteration i (a batch ahead of its gathers, so that the gathers
// never wait for an index load)
template <int OP>
__device__ __forceinline__ void ser_idx(const DLoop &L, int64_t i, SerBatch<OP> &b) {
  b.ra = b.wa = b.xa = -1;
  b.o0 = b.o1 = 0;
  if (i >= L.n) return;
  b.ra = (int32_t)ixl(L, L.r, i);
  b.wa = (int32_t)ixl(L, L.w, i);
  if constexpr (OP == JP_OP_STENCIL2) b.xa = (int32_t)ixl(L, L.r2, i);
  if constexpr (OP == JP_OP_PRIV_TMP) b.xa = (int32_t)ixl(L, L.s, i);
}
template <int OP, int DT>
__device__ __forceinline__ void ser_gather(const DLoop &L, SerBatch<OP> &b) {
  if (b.wa < 0) return;
  if constexpr (OP == JP_OP_ADD_C) b.o0 = __ldcg(L.A + b.ra);
  else if constexpr (OP == JP_OP_SAXPY) { b.o0 = __ldg(L.X + b.ra); b.o1 = __ldcg(L.A + b.wa); }
  else if constexpr (OP == JP_OP_PRIV_TMP) b.o0 = __ldg(L.X + b.ra);
  else { b.o0 = __ldcg(L.A + b.ra); b.o1 = __ldcg(L.A + b.xa); }
}

// A elements read by operand 0 / 1 (-2: the operand is not an A read)
template <int OP>
__device__ __forceinline__ int32_t a_read0(const SerBatch<OP> &b) {
  return (OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2) && b.wa >= 0 ? b.ra : -2;
}
template <int OP>
__device__ __forceinline__ int32_t a_read1(const SerBatch<OP> &b) {
  if (b.wa < 0) return -2;
  return OP == JP_OP_SAXPY ? b.wa : OP == JP_OP_STENCIL2 ? b.xa : -2;
}

template <int OP, int DT>
__device__ __forceinline__ uint32_t ser_body(const DLoop &L, uint32_t a0, uint32_t a1, uint32_t &vt) {
  if constexpr (OP == JP_OP_ADD_C) return op_add<DT>(a0, L.c0);
  else if constexpr (OP == JP_OP_SAXPY) return op_add<DT>(op_mul<DT>(L.c0, a0), a1);
  else if constexpr (OP == JP_OP_PRIV_TMP) { vt = op_mul<DT>(L.c0, a0); return op_add<DT>(vt, L.c1); }
  else return op_mul<DT>(op_add<DT>(a0, a1), L.c0);
}
}  // namespace

template <int OP, int DT>
__global__ void __launch_bounds__(32, 1) k_serial_warp(DLoop L, int64_t *stats) {
  const int lane = threadIdx.x;
  SerBatch<OP> c, nx, nn;
  ser_idx<OP>(L, lane, c);
  ser_gather<OP, DT>(L, c);
  ser_idx<OP>(L, 32 + lane, nx);
  int64_t fwd = 0;
  for (int64_t base = 0; base < L.n; base += 32) {
    // the next batch's operands (its indices arrived a batch ago) and the
    // indices of the batch after it, issued before this batch stores
    ser_gather<OP, DT>(L, nx);
    ser_idx<OP>(L, base + 64 + lane, nn);
    // in-batch sources: the latest earlier lane writing the element read
    const int32_t r0 = a_read0<OP>(c), r1 = a_read1<OP>(c);
    int s0 = -1, s1 = -1;
#pragma unroll
    for (int k = 0; k < 31; k++) {
      const int32_t wk = __shfl_sync(kFull, c.wa, k);
      if (k < lane && wk >= 0) {
        if (wk == r0) s0 = k;
        if (wk == r1) s1 = k;
      }
    }
    fwd += (s0 >= 0 || s1 >= 0);
    // resolve in dependence order: one round per chain link; a lane's state
    // travels as one 64-bit word (value | done << 32)
    bool done = c.wa < 0;
    uint32_t va = 0, vt = 0;
    if constexpr (OP == JP_OP_ADD_C || OP == JP_OP_SAXPY) {
      // one source per lane: its depth in the dependence forest by pointer
      // jumping (5 rounds), then exactly max-depth + 1 value rounds, no votes
      const int src = OP == JP_OP_ADD_C ? s0 : s1;
      int dep = src >= 0, p = src;
      for (int k = 0; k < 5 && __any_sync(kFull, p >= 0); k++) {
        const int q = p < 0 ? lane : p;
        const int pd = __shfl_sync(kFull, dep, q), pp = __shfl_sync(kFull, p, q);
        if (p >= 0) { dep += pd; p = pp; }
      }
      const int maxd = (int)__reduce_max_sync(kFull, (unsigned)(done ? 0 : dep));
      const int q = src < 0 ? lane : src;
      for (int rd = 0; rd <= maxd; rd++) {
        const uint32_t v = __shfl_sync(kFull, va, q);
        if (!done && dep == rd) {
          if (src >= 0) { if (OP == JP_OP_ADD_C) c.o0 = v; else c.o1 = v; }
          va = ser_body<OP, DT>(L, c.o0, c.o1, vt);
        }
      }
    } else if (!__all_sync(kFull, s0 < 0 && s1 < 0)) {
      for (;;) {
        const unsigned long long me = (unsigned long long)done << 32 | va;
        constexpr bool has0 = OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2;   // operand 0 may be an A read
        constexpr bool has1 = OP == JP_OP_SAXPY || OP == JP_OP_STENCIL2;   // operand 1 may be an A read
        unsigned long long u0 = 1ull << 32, u1 = 1ull << 32;
        if constexpr (has0) u0 = __shfl_sync(kFull, me, s0 < 0 ? lane : s0);
        if constexpr (has1) u1 = __shfl_sync(kFull, me, s1 < 0 ? lane : s1);
        if (!done && (s0 < 0 || (u0 >> 32)) && (s1 < 0 || (u1 >> 32))) {
          if (s0 >= 0) c.o0 = (uint32_t)u0;
          if (s1 >= 0) c.o1 = (uint32_t)u1;
          va = ser_body<OP, DT>(L, c.o0, c.o1, vt);
          done = true;
        }
        if (__all_sync(kFull, done)) break;
      }
    } else if (!done) {
      va = ser_body<OP, DT>(L, c.o0, c.o1, vt);
    }
    // stores: last writer of each element within the batch
    const unsigned gw = __match_any_sync(kFull, c.wa);
    if (c.wa >= 0 && 31 - __clz(gw) == lane) __stcg(L.A + c.wa, va);
    if constexpr (OP == JP_OP_PRIV_TMP) {
      const unsigned gs = __match_any_sync(kFull, c.xa);
      if (c.xa >= 0 && 31 - __clz(gs) == lane) __stcg(L.T + c.xa, vt);
    }
    // patch the next batch's operands from this batch's writes (latest writer last)
    const int32_t n0 = a_read0<OP>(nx), n1 = a_read1<OP>(nx);
#pragma unroll
    for (int k = 0; k < 32; k++) {
      const int32_t wk = __shfl_sync(kFull, c.wa, k);
      const uint32_t vk = __shfl_sync(kFull, va, k);
      if (wk >= 0) {
        if (wk == n0) nx.o0 = vk;
        if (wk == n1) nx.o1 = vk;
      }
    }
    __syncwarp();   // this batch's stores are ordered before the next batch's loads of any lane
    c = nx;
    nx = nn;
  }
  fwd = __reduce_add_sync(kFull, (unsigned)fwd);
  if (lane == 0 && stats) {
    const int64_t nb = (L.n + 31) / 32;
    stats[0] = L.n;
    stats[1] = L.n;
    stats[2] = nb;
    stats[3] = fwd;
  }
}

template <int OP, int DT>
static void run_serial(const DLoop &d, int64_t *stats, cudaStream_t st) {
  k_serial_warp<OP, DT><<<1, 32, 0, st>>>(d, stats);
  note_launch();
}

cudaError_t launch_serial(const Job &j, int64_t *stats, cudaStream_t st) {
  if (j.d.n == 0) {
    if (stats) cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
    return launch_check();
  }
  JP_DISPATCH(j.op, j.dt, run_serial, j.d, stats, st);
  return launch_check();
}

}  // namespace jp
