// jp_static.cu -- static analysis lite: "Loops
// determined as DOALL by static analysis are executed in mode A";
// the translator's rule 1 asks whether array indices are affine in the loop
// variable.  There is no compiler here, so the index arrays
// themselves are examined: one streaming pass decides, per index array,
// whether p[i] == p[0] + (p[1] - p[0]) * i for every i; the host then runs an
// exact two-variable dependence test on every (write, access) pair of the same
// array (an integer solution i != j in [0, n) of alpha_f i + beta_f ==
// alpha_g j + beta_g).  A loop whose accesses are all affine and pairwise
// conflict-free is DOALL without profiling; its index range is checked from
// the endpoints (reading A13).  Anything else is left to the profiler.
#include <cstdint>
#include "jp_host.h"

namespace jp {

// flags[q] stays 1 while index array q is affine; p[0], p[1] give alpha, beta
__global__ void __launch_bounds__(256) k_affine(int64_t n, const int32_t *p0, const int32_t *p1, const int32_t *p2,
                                                const int32_t *p3, int *flags) {
  const int32_t *ps[4] = {p0, p1, p2, p3};
  bool ok[4];
  int64_t a[4], b[4];
#pragma unroll
  for (int q = 0; q < 4; q++) {
    ok[q] = true;
    if (ps[q]) { b[q] = __ldg(ps[q]); a[q] = n > 1 ? (int64_t)__ldg(ps[q] + 1) - b[q] : 0; }
  }
  const int64_t stride = (int64_t)gridDim.x * blockDim.x * 4;
  for (int64_t i0 = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) * 4; i0 < n; i0 += stride) {
#pragma unroll
    for (int q = 0; q < 4; q++) {
      if (!ps[q] || !ok[q]) continue;
      const bool vec = ((uintptr_t)ps[q] & 15) == 0 && i0 + 4 <= n;
      int32_t v[4];
      if (vec) {
        const int4 x = __ldcs(reinterpret_cast<const int4 *>(ps[q] + i0));
        v[0] = x.x; v[1] = x.y; v[2] = x.z; v[3] = x.w;
      } else {
        for (int k = 0; k < 4; k++) v[k] = i0 + k < n ? __ldg(ps[q] + i0 + k) : 0;
      }
      for (int k = 0; k < 4 && i0 + k < n; k++) ok[q] = ok[q] && (int64_t)v[k] == b[q] + a[q] * (i0 + k);
    }
  }
#pragma unroll
  for (int q = 0; q < 4; q++) {
    if (!ps[q]) continue;
    const bool all = __all_sync(0xffffffffu, ok[q]);
    if ((threadIdx.x & 31) == 0 && !all) atomicAnd(&flags[q], 0);
  }
}

cudaError_t launch_affine(const Job &j, int *flags, cudaStream_t st) {
  cudaMemsetAsync(flags, 0, 4 * sizeof(int), st);
  const int32_t *ps[4] = {j.d.r, j.d.r2, j.d.w, j.d.s};
  int one[4];
  for (int q = 0; q < 4; q++) one[q] = ps[q] ? 1 : 0;
  cudaMemcpyAsync(flags, one, sizeof one, cudaMemcpyHostToDevice, st);   // pageable: ordered on st
  if (j.d.n == 0) return launch_check();
  const int64_t need = ((j.d.n + 3) / 4 + 255) / 256, cap = (int64_t)num_sms() * 8;
  k_affine<<<(int)(need < 1 ? 1 : need < cap ? need : cap), 256, 0, st>>>(j.d.n, j.d.r, j.d.r2, j.d.w, j.d.s, flags);
  note_launch();
  return launch_check();
}

// One warp: are the first m entries of every index array affine?  The verdict
// goes to mapped host words (mir[0]), then the call's sequence number
// (mir[1]): the host polls it instead of a device-to-host copy and a sync.
__global__ void __launch_bounds__(32) k_prefix_affine(const int32_t *p0, const int32_t *p1, const int32_t *p2,
                                                      const int32_t *p3, int m, long long *mir,
                                                      unsigned long long seq) {
  const int32_t *ps[4] = {p0, p1, p2, p3};
  bool ok = true;
#pragma unroll
  for (int q = 0; q < 4; q++) {
    if (!ps[q]) continue;
    const int64_t b = __ldg(ps[q]), a = (int64_t)__ldg(ps[q] + 1) - b;
    for (int k = threadIdx.x; k < m; k += 32) ok = ok && (int64_t)__ldg(ps[q] + k) == b + a * k;
  }
  ok = __all_sync(0xffffffffu, ok);
  if (threadIdx.x == 0) {
    mir[0] = ok ? 1 : 0;
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(mir + 1), "l"(seq) : "memory");
  }
}

cudaError_t launch_prefix_affine(const Job &j, int m, long long *mir, unsigned long long seq, cudaStream_t st) {
  k_prefix_affine<<<1, 32, 0, st>>>(j.d.r, j.d.r2, j.d.w, j.d.s, m, mir, seq);
  note_launch();
  return launch_check();
}

// ---------------------------------------------------------------------------
// host: exact dependence test of two affine accesses f(i) = af*i + bf (a write)
// and g(j) = ag*j + bg of the same array, i, j in [0, n), i != j
// ---------------------------------------------------------------------------
static int64_t egcd(int64_t a, int64_t b, int64_t &x, int64_t &y) {
  if (b == 0) { x = a >= 0 ? 1 : -1; y = 0; return a >= 0 ? a : -a; }
  int64_t x1, y1;
  const int64_t g = egcd(b, a % b, x1, y1);
  x = y1;
  y = x1 - (a / b) * y1;
  return g;
}

bool affine_conflict(int64_t af, int64_t bf, int64_t ag, int64_t bg, int64_t n) {
  if (n < 2) return false;
  const int64_t c = bg - bf;   // af*i - ag*j = c
  if (af == 0 && ag == 0) return c == 0;                       // one address, touched by every iteration
  if (af == ag) {                                              // i - j = c / a
    if (c % af) return false;
    const int64_t d = c / af;
    return d != 0 && (d < 0 ? -d : d) <= n - 1;
  }
  // general: af*i + (-ag)*j = c, solutions i = i0 + (ag/g) t, j = j0 + (af/g) t
  int64_t x, y;
  const int64_t g = egcd(af, -ag, x, y);
  if (c % g) return false;
  const __int128 i0 = (__int128)x * (c / g), j0 = (__int128)y * (c / g);
  const int64_t si = ag / g, sj = af / g;   // i = i0 + si t, j = j0 + sj t (note -(-ag)/g = ag/g)
  // t range with 0 <= i, j <= n-1
  __int128 lo = -((__int128)1 << 100), hi = (__int128)1 << 100;
  auto bound = [&](__int128 v0, int64_t s) {
    if (s == 0) {
      if (v0 < 0 || v0 > n - 1) { lo = 1; hi = 0; }
      return;
    }
    // 0 <= v0 + s t <= n - 1
    const __int128 a1 = -v0, a2 = (__int128)(n - 1) - v0;
    __int128 l, h;
    if (s > 0) { l = a1 >= 0 ? (a1 + s - 1) / s : -((-a1) / s); h = a2 >= 0 ? a2 / s : -((-a2 + s - 1) / s); }
    else {
      const int64_t m = -s;   // 0 <= v0 - m t <= n-1  ->  (v0 - (n-1))/m <= t <= v0/m
      const __int128 b1 = v0 - (__int128)(n - 1), b2 = v0;
      l = b1 >= 0 ? (b1 + m - 1) / m : -((-b1) / m);
      h = b2 >= 0 ? b2 / m : -((-b2 + m - 1) / m);
    }
    if (l > lo) lo = l;
    if (h < hi) hi = h;
  };
  bound(i0, si);
  bound(j0, sj);
  if (lo > hi) return false;
  // every solution with i == j lies at one t (si != sj since af != ag): excluded
  const __int128 cnt = hi - lo + 1;
  if (cnt >= 2) return true;
  const __int128 ii = i0 + (__int128)si * lo, jj = j0 + (__int128)sj * lo;
  return ii != jj;
}

}  // namespace jp
