// jp_exchange.cu -- owner-partitioned sparse exchange (SURVEY §8(f) NEXT-2,
// §8(e) "an owner-partitioned sparse all-to-all").
//
// The partitioned profile (C1) and the partitioned merges (C4) reduce dense
// per-address tables across ranks (privatized values are written
// back "after all the iterations finish"; the profile needs the first writer /
// first reader of every address over the whole loop, reading A1).  A dense
// all_reduce moves len entries per rank whatever the loop touched; these
// kernels turn a table into (address, value...) rows bucketed by the address's
// owner rank so that dist.py's all_to_all moves only the touched entries:
//
//   pack    dense table(s) -> rows [m][1+ntab], column 0 the address, sorted by
//           address, hence grouped by owner (owner(a) = a / ceil(len/world))
//   reduce  rows -> table(s): atomicMax (the owner folds every rank's entries)
//   gather  table(s) -> rows: the owner answers each received row with the
//           reduced value (the C1 response)
//   scatter rows -> table(s): a rank installs the answers / the owners' finals
//
// Rows whose address lies outside [0, len) are ignored by reduce / gather /
// scatter (dist.py pads all_gather buffers with address -1).
#include "jp_host.h"

namespace jp {

constexpr int kXThreads = 256, kXPer = 16, kXTile = kXThreads * kXPer;

struct XTiles {
  int64_t lo, hi, slice, tpo;   // tile t: owner k = t / tpo, j = t % tpo
  int world;
  __host__ __device__ void range(int64_t t, int64_t &b, int64_t &e) const {
    const int64_t k = t / tpo, j = t % tpo;
    int64_t s0 = k * slice, s1 = s0 + slice;
    if (s0 < lo) s0 = lo;
    if (s1 > hi) s1 = hi;
    b = s0 + j * kXTile;
    e = b + kXTile < s1 ? b + kXTile : s1;
    if (b > e) b = e;
  }
};

// Warp w of a tile owns the kXPer * 32 consecutive entries starting at
// b + w * kXPer * 32; round q reads entry (q, lane) = base + q * 32 + lane
// (coalesced).  Returns the warp's ballots packed as per-lane flag bits
// (bit q = flag of entry (q, lane)) and the warp's total.
template <typename E, int NT>
__device__ __forceinline__ uint32_t x_flags(const E *t0, const E *t1, E empty, int64_t b, int64_t e, int &wtot) {
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  const int64_t a0 = b + (int64_t)wid * kXPer * 32 + lane;
  uint32_t f = 0;
  E v0[kXPer], v1[kXPer];
#pragma unroll
  for (int q = 0; q < kXPer; q++) {   // all loads first (16 in flight per lane)
    const int64_t a = a0 + q * 32;
    v0[q] = a < e ? t0[a] : empty;
    if constexpr (NT == 2) v1[q] = a < e ? t1[a] : empty;
  }
  int tot = 0;
#pragma unroll
  for (int q = 0; q < kXPer; q++) {
    bool full = v0[q] != empty;
    if constexpr (NT == 2) full = full || v1[q] != empty;
    f |= (uint32_t)full << q;
    tot += __popc(__ballot_sync(0xffffffffu, full));
  }
  wtot = tot;
  return f;
}

// exclusive prefix of the warps' totals (one value per warp); *total = sum
__device__ __forceinline__ int x_warp_scan(int wtot, int *total) {
  __shared__ int ws[kXThreads / 32];
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  if (lane == 0) ws[wid] = wtot;
  __syncthreads();
  int pre = 0, tot = 0;
#pragma unroll
  for (int w = 0; w < kXThreads / 32; w++) {
    const int s = ws[w];
    if (w < wid) pre += s;
    tot += s;
  }
  *total = tot;
  return pre;
}

template <typename E, int NT>
__global__ void __launch_bounds__(kXThreads) k_x_count(const E *t0, const E *t1, E empty, XTiles X, int64_t *cnt) {
  int64_t b, e;
  X.range(blockIdx.x, b, e);
  int wtot, tot;
  x_flags<E, NT>(t0, t1, empty, b, e, wtot);
  x_warp_scan(wtot, &tot);
  if (threadIdx.x == 0) cnt[blockIdx.x] = tot;
}

// one CTA: off[t] = sum cnt[<t], off[tiles] = total, counts[k] = rows of owner k
__global__ void __launch_bounds__(1024) k_x_scan(const int64_t *cnt, int64_t tiles, int64_t tpo, int world,
                                                 int64_t *off, int64_t *counts) {
  __shared__ int64_t part[1024];
  const int tid = threadIdx.x;
  const int64_t per = (tiles + 1023) / 1024, t0 = tid * per;
  int64_t s = 0;
  for (int64_t t = t0; t < t0 + per && t < tiles; t++) s += cnt[t];
  part[tid] = s;
  __syncthreads();
  for (int d = 1; d < 1024; d <<= 1) {   // Hillis-Steele over 1024 partials
    const int64_t y = tid >= d ? part[tid - d] : 0;
    __syncthreads();
    part[tid] += y;
    __syncthreads();
  }
  int64_t run = part[tid] - s;
  for (int64_t t = t0; t < t0 + per && t < tiles; t++) {
    off[t] = run;
    run += cnt[t];
  }
  if (tid == 1023) off[tiles] = part[1023];
  __syncthreads();
  for (int k = tid; k < world; k += 1024) counts[k] = off[(k + 1) * tpo] - off[k * tpo];
}

template <typename E, int NT>
__global__ void __launch_bounds__(kXThreads) k_x_emit(const E *t0, const E *t1, E empty, XTiles X, const int64_t *off,
                                                      E *rows, int64_t cap) {
  int64_t b, e;
  X.range(blockIdx.x, b, e);
  int wtot, tot;
  const uint32_t f = x_flags<E, NT>(t0, t1, empty, b, e, wtot);
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  int64_t r = off[blockIdx.x] + x_warp_scan(wtot, &tot);
  const int64_t a0 = b + (int64_t)wid * kXPer * 32 + lane;
  const uint32_t lt = (1u << lane) - 1u;
#pragma unroll
  for (int q = 0; q < kXPer; q++) {
    const bool full = (f >> q) & 1u;
    const uint32_t bal = __ballot_sync(0xffffffffu, full);
    const int64_t ri = r + __popc(bal & lt);
    if (full && ri < cap) {
      const int64_t a = a0 + q * 32;
      E *row = rows + ri * (1 + NT);
      row[0] = (E)a;
      row[1] = t0[a];
      if constexpr (NT == 2) row[2] = t1[a];
    }
    r += __popc(bal);
  }
}

__device__ __forceinline__ void x_max(int32_t *p, int32_t v) { atomicMax(p, v); }
__device__ __forceinline__ void x_max(unsigned long long *p, unsigned long long v) { atomicMax(p, v); }
__device__ __forceinline__ int64_t x_addr(int32_t v) { return v; }
__device__ __forceinline__ int64_t x_addr(unsigned long long v) { return (int64_t)v; }

// what: 0 reduce (atomicMax), 1 gather (row <- table), 2 scatter (table <- row)
template <typename E, int NT>
__global__ void __launch_bounds__(kXThreads) k_x_rows(E *t0, E *t1, int64_t len, E *rows, int64_t m, int what) {
  const int64_t stride = (int64_t)gridDim.x * kXThreads;
  for (int64_t i = (int64_t)blockIdx.x * kXThreads + threadIdx.x; i < m; i += stride) {
    E *row = rows + i * (1 + NT);
    const int64_t a = x_addr(row[0]);
    if (a < 0 || a >= len) continue;
    if (what == 0) {
      x_max(&t0[a], row[1]);
      if constexpr (NT == 2) x_max(&t1[a], row[2]);
    } else if (what == 1) {
      row[1] = __ldcg(&t0[a]);
      if constexpr (NT == 2) row[2] = __ldcg(&t1[a]);
    } else {
      t0[a] = row[1];
      if constexpr (NT == 2) t1[a] = row[2];
    }
  }
}

static XTiles x_tiles(int64_t len, int64_t lo, int64_t hi, int world) {
  XTiles X;
  X.lo = lo;
  X.hi = hi;
  X.world = world;
  X.slice = (len + world - 1) / world;
  if (X.slice < 1) X.slice = 1;
  int64_t seg = X.slice < hi - lo ? X.slice : hi - lo;
  X.tpo = seg > 0 ? (seg + kXTile - 1) / kXTile : 1;
  return X;
}

size_t sparse_scratch_bytes(int64_t len, int world) {
  const int64_t tiles = (int64_t)world * ((((len + world - 1) / world) + kXTile - 1) / kXTile + 1);
  return (size_t)(2 * tiles + 2 + world) * sizeof(int64_t);
}

template <typename E, int NT>
static void pack_t(const void *t0, const void *t1, int64_t empty, const XTiles &X, int64_t tiles, int64_t *cnt,
                   int64_t *off, int64_t *counts, void *rows, int64_t cap, cudaStream_t st) {
  const E em = (E)empty;
  k_x_count<E, NT><<<(unsigned)tiles, kXThreads, 0, st>>>((const E *)t0, (const E *)t1, em, X, cnt);
  k_x_scan<<<1, 1024, 0, st>>>(cnt, tiles, X.tpo, X.world, off, counts);
  k_x_emit<E, NT><<<(unsigned)tiles, kXThreads, 0, st>>>((const E *)t0, (const E *)t1, em, X, off, (E *)rows, cap);
  note_launch(3);
}

cudaError_t launch_sparse_pack(const void *t0, const void *t1, int elem, int64_t len, int64_t lo, int64_t hi,
                               int64_t empty, int world, void *rows, int64_t cap, int64_t *counts_dev, void *scratch,
                               cudaStream_t st) {
  const XTiles X = x_tiles(len, lo, hi, world);
  const int64_t tiles = (int64_t)world * X.tpo;
  int64_t *cnt = static_cast<int64_t *>(scratch), *off = cnt + tiles;
  if (elem == 4) {
    if (t1) pack_t<int32_t, 2>(t0, t1, empty, X, tiles, cnt, off, counts_dev, rows, cap, st);
    else pack_t<int32_t, 1>(t0, t1, empty, X, tiles, cnt, off, counts_dev, rows, cap, st);
  } else {
    if (t1) pack_t<unsigned long long, 2>(t0, t1, empty, X, tiles, cnt, off, counts_dev, rows, cap, st);
    else pack_t<unsigned long long, 1>(t0, t1, empty, X, tiles, cnt, off, counts_dev, rows, cap, st);
  }
  return launch_check();
}

int64_t sparse_pack_tiles(int64_t len, int64_t lo, int64_t hi, int world) {
  return (int64_t)world * x_tiles(len, lo, hi, world).tpo;
}

cudaError_t launch_sparse_rows(void *t0, void *t1, int elem, int64_t len, void *rows, int64_t m, int what,
                               cudaStream_t st) {
  if (m <= 0) return cudaSuccess;
  int64_t g = (m + kXThreads - 1) / kXThreads;
  const int64_t gmax = (int64_t)num_sms() * 8;
  if (g > gmax) g = gmax;
  if (elem == 4) {
    if (t1) k_x_rows<int32_t, 2><<<(unsigned)g, kXThreads, 0, st>>>((int32_t *)t0, (int32_t *)t1, len, (int32_t *)rows, m, what);
    else k_x_rows<int32_t, 1><<<(unsigned)g, kXThreads, 0, st>>>((int32_t *)t0, nullptr, len, (int32_t *)rows, m, what);
  } else {
    using U = unsigned long long;
    if (t1) k_x_rows<U, 2><<<(unsigned)g, kXThreads, 0, st>>>((U *)t0, (U *)t1, len, (U *)rows, m, what);
    else k_x_rows<U, 1><<<(unsigned)g, kXThreads, 0, st>>>((U *)t0, nullptr, len, (U *)rows, m, what);
  }
  note_launch(1);
  return launch_check();
}

}  // namespace jp
