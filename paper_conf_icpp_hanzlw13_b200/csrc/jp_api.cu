// jp_api.cu -- the extern "C" entry points of libjp.so (include/jp.h).
// Host logic only: argument checks, workspace layout, the Fig. 2(b) decision,
// the task-sharing / task-stealing plans and the one-GPU scheduler.  Every
// step of the loop itself runs in the kernels of jp_*.cu.
#include <algorithm>
#include <atomic>
#include <cmath>
#include <cstdarg>
#include <cstdio>
#include <cstring>
#include <functional>
#include <mutex>
#include <string>
#include <vector>

#include "jp_host.h"

namespace jp {

static std::atomic<long long> g_launches{0};
void note_launch(int k) { g_launches.fetch_add(k, std::memory_order_relaxed); }

static thread_local std::string g_err;

static jp_status fail(jp_status s, const char *fmt, ...) {
  char buf[512];
  va_list ap;
  va_start(ap, fmt);
  vsnprintf(buf, sizeof buf, fmt, ap);
  va_end(ap);
  g_err = buf;
  return s;
}

int num_sms() {
  static int cache[64] = {0};
  int dev = 0;
  cudaGetDevice(&dev);
  if (dev < 0 || dev >= 64) dev = 0;
  if (!cache[dev]) {
    int v = 0;
    cudaDeviceGetAttribute(&v, cudaDevAttrMultiProcessorCount, dev);
    cache[dev] = v > 0 ? v : 1;
  }
  return cache[dev];
}

cudaError_t launch_check() { return cudaGetLastError(); }

static jp_status cuda_fail(cudaError_t e, const char *where) {
  return fail(JP_ERR_CUDA, "%s: %s", where, cudaGetErrorString(e));
}

static bool have_device() {
  int n = 0;
  if (cudaGetDeviceCount(&n) != cudaSuccess || n == 0) {
    cudaGetLastError();
    return false;
  }
  return true;
}

static size_t al256(size_t x) { return (x + 255) & ~(size_t)255; }

// index arrays the opcode actually uses
static void used_idx(int op, bool &r, bool &r2, bool &w, bool &s) {
  r = true; w = true;
  r2 = op == JP_OP_STENCIL2;
  s = op == JP_OP_PRIV_TMP;
}

Job make_job(const jp_loop *L) {
  Job j;
  bool ur, ur2, uw, us;
  used_idx(L->op, ur, ur2, uw, us);
  j.op = L->op;
  j.dt = L->dtype;
  DLoop &d = j.d;
  d.n = L->n;
  d.base = L->iter_base;
  d.ioff = L->ident_off;
  d.r = ur ? L->r : nullptr;
  d.r2 = ur2 ? L->r2 : nullptr;
  d.w = uw ? L->w : nullptr;
  d.s = us ? L->s : nullptr;
  d.A = static_cast<uint32_t *>(L->A);
  d.lenA = L->len_A;
  d.X = static_cast<const uint32_t *>(L->X);
  d.lenX = L->len_X;
  d.T = static_cast<uint32_t *>(L->T);
  d.lenT = L->len_T;
  d.c0 = (uint32_t)L->c0.i;
  d.c1 = (uint32_t)L->c1.i;
  return j;
}

static bool has_idx(const Job &j) { return j.d.r || j.d.r2 || j.d.w || j.d.s; }

SchedLayout sched_layout(const jp_loop *L) {
  SchedLayout s{};
  Job j = make_job(L);
  const bool aI = a_indirect(j.op, j.d.r, j.d.r2, j.d.w), tI = t_indirect(j.op, j.d.s);
  const int64_t nck = (L->n + kSchedMinChunk - 1) / kSchedMinChunk + 1;
  size_t o = 0;
  s.counts = o; o = al256(o + 24 * (size_t)nck);
  s.chunk_task = o; o = al256(o + 4 * (size_t)nck);
  s.wmA = aI ? o : SIZE_MAX; if (aI) o = al256(o + 8 * (size_t)L->len_A);
  s.rmA = aI && a_has_reads(j.op) ? o : SIZE_MAX; if (s.rmA != SIZE_MAX) o = al256(o + 8 * (size_t)L->len_A);
  s.wmT = tI ? o : SIZE_MAX; if (tI) o = al256(o + 8 * (size_t)L->len_T);
  s.rmT = tI ? o : SIZE_MAX; if (tI) o = al256(o + 8 * (size_t)L->len_T);
  s.conf = o; o = al256(o + 8 * kMaxTasks);
  s.tstats = o; o = al256(o + 32 * kMaxTasks);
  s.ranges = o; o = al256(o + 16 * kMaxTasks);
  s.crange = o; o = al256(o + 8 * (size_t)nck);
  s.total = o;
  return s;
}

Layout layout(const jp_loop *L) {
  Layout lo;
  memset(&lo, 0, sizeof lo);
  Job j = make_job(L);
  const bool aI = a_indirect(j.op, j.d.r, j.d.r2, j.d.w), tI = t_indirect(j.op, j.d.s);
  size_t off = 0;
  auto add = [&](int r, size_t bytes) {
    off = al256(off);
    lo.off[r] = off;
    lo.bytes[r] = bytes;
    off += bytes;
  };
  add(R_HEADER, kHeaderBytes);
  add(R_MINW_A, aI ? 4 * (size_t)L->len_A : 0);
  add(R_MINR_A, aI && a_has_reads(j.op) ? 4 * (size_t)L->len_A : 0);
  add(R_MINW_T, tI ? 4 * (size_t)L->len_T : 0);
  add(R_MINR_T, tI ? 4 * (size_t)L->len_T : 0);
  add(R_KEYS_A, aI ? 8 * (size_t)L->len_A : 0);
  add(R_KEYS_T, tI ? 8 * (size_t)L->len_T : 0);
  add(R_TLS_S_A, aI && j.op != JP_OP_PRIV_TMP ? 8 * (size_t)L->len_A : 0);
  add(R_TLS_C_A, aI ? 8 * (size_t)L->len_A : 0);
  add(R_TLS_S_T, 0);
  add(R_TLS_C_T, tI ? 8 * (size_t)L->len_T : 0);
  add(R_SCHED, sched_layout(L).total);
  const bool rx = aI && j.op != JP_OP_PRIV_TMP;   // A has exposed reads through an index
  add(R_MAXRX_A, rx ? 4 * (size_t)L->len_A : 0);
  add(R_GUIDE, rx ? 8 * (size_t)((L->n + 31) / 32) : 0);
  lo.total = al256(off);
  return lo;
}

size_t layout_end(const Layout &lo, int uses) {
  int last = R_HEADER;
  if (uses & JP_WS_PROFILE) last = R_MINR_T;
  if (uses & JP_WS_PRIV) last = std::max(last, (int)R_KEYS_T);
  if (uses & JP_WS_TLS) last = std::max(last, (int)R_TLS_C_T);
  if (uses & JP_WS_SCHED) last = R_SCHED;
  if (uses & JP_WS_GUIDE) last = R_GUIDE;
  return al256(lo.off[last] + lo.bytes[last]);
}

}  // namespace jp

using namespace jp;

// ---------------------------------------------------------------------------
// argument checks
// ---------------------------------------------------------------------------
static jp_status check_loop(const jp_loop *L) {
  if (!L) return fail(JP_ERR_ARG, "loop descriptor is NULL");
  if (L->op < JP_OP_ADD_C || L->op > JP_OP_STENCIL2) return fail(JP_ERR_UNSUPPORTED, "opcode %d is not templated", L->op);
  if (L->dtype != JP_I32 && L->dtype != JP_F32) return fail(JP_ERR_UNSUPPORTED, "dtype %d is not templated", L->dtype);
  if (L->n < 0 || L->iter_base < 0 || L->iter_base + L->n > 2147483646LL || L->ident_off < 0)
    return fail(JP_ERR_ARG, "need 0 <= n, 0 <= iter_base, 0 <= ident_off, iter_base + n <= 2^31-2 (n=%lld base=%lld)",
                (long long)L->n, (long long)L->iter_base);
  const int64_t lmax = 2147483647LL;
  if (L->len_A < 0 || L->len_X < 0 || L->len_T < 0 || L->len_A > lmax || L->len_X > lmax || L->len_T > lmax)
    return fail(JP_ERR_ARG, "array lengths must be in [0, 2^31-1]");
  if (L->n == 0) return JP_OK;
  if (!L->A) return fail(JP_ERR_ARG, "A/Y is NULL");
  const bool usesX = L->op == JP_OP_SAXPY || L->op == JP_OP_PRIV_TMP;
  if (usesX && !L->X) return fail(JP_ERR_ARG, "X is NULL");
  if (L->op == JP_OP_PRIV_TMP && !L->T) return fail(JP_ERR_ARG, "T is NULL");
  // identity accesses must stay inside their arrays (reading A13)
  auto idn = [&](const int32_t *p, int64_t len, const char *what) -> jp_status {
    if (!p && L->ident_off + L->n > len)
      return fail(JP_ERR_INDEX, "identity index of %s exceeds its length (%lld > %lld)", what,
                  (long long)(L->ident_off + L->n), (long long)len);
    return JP_OK;
  };
  jp_status s = JP_OK;
  switch (L->op) {
    case JP_OP_ADD_C: if ((s = idn(L->r, L->len_A, "r"))) return s; if ((s = idn(L->w, L->len_A, "w"))) return s; break;
    case JP_OP_SAXPY: if ((s = idn(L->r, L->len_X, "r"))) return s; if ((s = idn(L->w, L->len_A, "w"))) return s; break;
    case JP_OP_PRIV_TMP:
      if ((s = idn(L->r, L->len_X, "r"))) return s;
      if ((s = idn(L->s, L->len_T, "s"))) return s;
      if ((s = idn(L->w, L->len_A, "w"))) return s;
      break;
    default:
      if ((s = idn(L->r, L->len_A, "r"))) return s;
      if ((s = idn(L->r2, L->len_A, "r2"))) return s;
      if ((s = idn(L->w, L->len_A, "w"))) return s;
  }
  return JP_OK;
}

static jp_status check_ws(const jp_loop *L, void *ws, size_t ws_bytes, int uses, Layout &lo) {
  lo = layout(L);
  const size_t need = layout_end(lo, uses);
  if (!ws || ws_bytes < need)
    return fail(JP_ERR_WORKSPACE, "workspace of %zu bytes is smaller than the %zu bytes needed", ws ? ws_bytes : 0,
                need);
  if ((uintptr_t)ws & 255) return fail(JP_ERR_WORKSPACE, "workspace must be 256-byte aligned");
  return JP_OK;
}

#define JP_TRY(expr)                  \
  do {                                \
    jp_status _s = (expr);            \
    if (_s != JP_OK) return _s;       \
  } while (0)
#define JP_CUDA(expr, where)                        \
  do {                                              \
    cudaError_t _e = (expr);                        \
    if (_e != cudaSuccess) return cuda_fail(_e, where); \
  } while (0)

static jp_status need_device() {
  if (!have_device()) return fail(JP_ERR_CUDA, "no CUDA device (libjp.so has no CPU fallback)");
  return JP_OK;
}

// Small device->host reads of results (a few hundred bytes) go through a
// per-thread pinned staging buffer: a pageable destination would add a staged
// copy to every jp_schedule / profile / TLS call (latency-bound config 1).
static cudaError_t d2h_small_sync(void *dst, const void *src, size_t bytes, cudaStream_t st) {
  thread_local void *pin = nullptr;
  thread_local size_t pin_bytes = 0;
  if (bytes > pin_bytes) {
    if (pin) cudaFreeHost(pin);
    pin_bytes = bytes < 4096 ? 4096 : bytes;
    cudaError_t e = cudaMallocHost(&pin, pin_bytes);
    if (e != cudaSuccess) { pin = nullptr; pin_bytes = 0; return e; }
  }
  cudaError_t e = cudaMemcpyAsync(pin, src, bytes, cudaMemcpyDeviceToHost, st);
  if (e == cudaSuccess) e = cudaStreamSynchronize(st);
  if (e == cudaSuccess) memcpy(dst, pin, bytes);
  return e;
}

// Per-thread mapped pinned words for the tiny path (config 1): the kernel writes
// its results and a sequence flag there; NULL host when the allocation fails
// (then the D2H copy path is used).
struct TinyMirror {
  int64_t *host = nullptr, *dev = nullptr;
  unsigned long long seq = 0;
};
static TinyMirror &tiny_mirror() {
  thread_local TinyMirror m;
  thread_local bool tried = false;
  if (!tried) {
    tried = true;
    void *p = nullptr;
    if (!getenv("JP_TINY_NO_MIRROR") &&
        cudaHostAlloc(&p, 32 * sizeof(int64_t), cudaHostAllocMapped | cudaHostAllocPortable) == cudaSuccess) {
      void *d = nullptr;
      if (cudaHostGetDevicePointer(&d, p, 0) == cudaSuccess) {
        memset(p, 0, 32 * sizeof(int64_t));
        m.host = static_cast<int64_t *>(p);
        m.dev = static_cast<int64_t *>(d);
      } else {
        cudaFreeHost(p);
      }
    }
    cudaGetLastError();
  }
  return m;
}

// validate indices on the device, syncs; JP_ERR_INDEX when any is out of range
static jp_status validate_sync(const Job &j, void *ws, const Layout &lo, cudaStream_t st, int64_t *bad_out) {
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  JP_CUDA(launch_validate(j, hdr, st), "validate");
  int64_t bad = 0;
  JP_CUDA(d2h_small_sync(&bad, &hdr[H_BAD], sizeof bad, st), "validate D2H");
  if (bad_out) *bad_out = bad;
  if (bad) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)bad);
  return JP_OK;
}

extern "C" {

const char *jp_last_error(void) { return g_err.c_str(); }
const char *jp_version(void) { return "jp-b200 0.1 (sm_100a)"; }
int64_t jp_launch_count(void) { return g_launches.load(); }
int64_t jp_tls_grid_window(void) { return have_device() ? tls_fwd_grid_wcap() : 0; }

int32_t jp_doall_kernel(int32_t which) {
  if (which == 0 || which == 1) set_doall_kernel_choice(which);
  return doall_kernel_choice();
}

size_t jp_workspace_bytes(const jp_loop *L, int32_t uses) {
  if (!L || check_loop(L) == JP_ERR_ARG) return 0;
  return layout_end(layout(L), uses);
}

jp_status jp_ws_region(const jp_loop *L, int32_t region, size_t *offset, size_t *bytes) {
  JP_TRY(check_loop(L));
  if (region < 0 || region >= R_COUNT) return fail(JP_ERR_ARG, "bad region id %d", region);
  Layout lo = layout(L);
  if (offset) *offset = lo.off[region];
  if (bytes) *bytes = lo.bytes[region];
  return JP_OK;
}

jp_status jp_validate(const jp_loop *L, void *ws, size_t ws_bytes, int64_t *bad, jp_stream_t st) {
  jp_status s = check_loop(L);
  if (s == JP_ERR_INDEX) { if (bad) *bad = -1; return s; }
  JP_TRY(s);
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, 0, lo));
  return validate_sync(make_job(L), ws, lo, (cudaStream_t)st, bad);
}

jp_status jp_profile_stamp(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st) {
  JP_TRY(check_loop(L));
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PROFILE, lo));
  JP_CUDA(launch_prof_stamp(make_job(L), ws, lo, (cudaStream_t)st), "profile stamp");
  return JP_OK;
}

static void fill_profile(jp_profile *out, int64_t n, const int64_t *h) {
  out->n = n;
  out->raw_iters = h[H_RAW];
  out->war_iters = h[H_WAR];
  out->waw_iters = h[H_WAW];
  out->first_raw_iter = h[H_FIRST_RAW];   // -1 (all ones) when none
  out->d_raw = n ? (double)out->raw_iters / (double)n : 0.0;
  out->d_war = n ? (double)out->war_iters / (double)n : 0.0;
  out->d_waw = n ? (double)out->waw_iters / (double)n : 0.0;
}

jp_status jp_profile_classify(const jp_loop *L, void *ws, size_t ws_bytes, uint32_t *raw_bits, int64_t chunk_iters,
                              int64_t *chunk_counts, jp_profile *out, jp_stream_t stp) {
  JP_TRY(check_loop(L));
  if (!out) return fail(JP_ERR_ARG, "profile output is NULL");
  if (chunk_counts && (chunk_iters <= 0 || chunk_iters % 32))
    return fail(JP_ERR_ARG, "chunk_iters must be a positive multiple of 32");
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PROFILE, lo));
  cudaStream_t st = (cudaStream_t)stp;
  JP_CUDA(launch_prof_classify(make_job(L), ws, lo, raw_bits, chunk_iters, chunk_counts, st), "profile classify");
  int64_t h[8];
  JP_CUDA(d2h_small_sync(h, at<int64_t>(ws, lo, R_HEADER), sizeof h, st), "profile D2H");
  if (h[H_BAD]) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)h[H_BAD]);
  fill_profile(out, L->n, h);
  return JP_OK;
}

jp_status jp_profile_density(const jp_loop *L, void *ws, size_t ws_bytes, uint32_t *raw_bits, int64_t chunk_iters,
                             int64_t *chunk_counts, jp_profile *out, jp_stream_t st) {
  JP_TRY(jp_profile_stamp(L, ws, ws_bytes, st));
  return jp_profile_classify(L, ws, ws_bytes, raw_bits, chunk_iters, chunk_counts, out, st);
}

// the largest raw count whose density is not above tau (select_mode_counts: mode B, not C)
static int64_t raw_max_for(int64_t n, double tau) {
  if (n <= 0) return 0;
  int64_t r = (int64_t)std::floor(tau * (double)n);
  if (r > n) r = n;
  while (r + 1 <= n && (double)(r + 1) / (double)n <= tau) r++;
  while (r >= 0 && (double)r / (double)n > tau) r--;
  return r;
}

static int32_t select_mode_counts(int64_t n, int64_t raw, int64_t war, int64_t waw, double tau) {
  const double d_raw = n ? (double)raw / (double)n : 0.0;
  if (d_raw > tau) return JP_MODE_SEQ_RECOMMENDED;   // mode C
  if (raw > 0) return JP_MODE_TLS;                    // mode B
  if (war > 0 || waw > 0) return JP_MODE_PRIVATIZED;  // mode D
  return JP_MODE_DOALL;                               // mode D'
}

int32_t jp_select_mode(const jp_loop *L, const jp_profile *p, double tau_high) {
  if (check_loop(L) == JP_ERR_ARG || check_loop(L) == JP_ERR_UNSUPPORTED) return -1;
  Job j = make_job(L);
  if (!has_idx(j)) return JP_MODE_DOALL;   // "determined DOALL" (mode A), no profile needed
  if (!p) { fail(JP_ERR_ARG, "a profile is required when index arrays are present"); return -1; }
  return select_mode_counts(p->n, p->raw_iters, p->war_iters, p->waw_iters, tau_high);
}

// ---------------------------------------------------------------------------
// static analysis lite (jp_static.cu)
// ---------------------------------------------------------------------------
// after_sample (nullable): called right after the prefix sample is launched,
// before the host waits for it (jp_schedule queues side-stream work there)
static jp_status static_check(const jp_loop *L, const Job &j, void *ws, const Layout &lo, jp_static *out,
                              cudaStream_t st, const std::function<void()> *after_sample = nullptr,
                              bool skip_prefix = false) {
  bool kicked = false;
  auto kick = [&]() {
    if (after_sample && !kicked) (*after_sample)();
    kicked = true;
  };
  memset(out, 0, sizeof *out);
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  int *flags = reinterpret_cast<int *>(&hdr[H_AFFINE]);
  if (!skip_prefix) {
    // a 64-entry prefix of each index array first: an array that is not affine
    // there is not affine at all, and the full pass (a read of every index
    // array) is skipped -- the common case of indirect loops
    constexpr int kS = 64;
    const int m = (int)std::min<int64_t>(L->n, kS);
    TinyMirror &mm = tiny_mirror();
    if (m >= 3 && mm.host) {
      // verdict through mapped host words (tiny mirror [19], sequence [20]): one
      // warp-sized kernel and a poll instead of copies and a stream sync
      const unsigned long long seq = ++mm.seq;
      JP_CUDA(launch_prefix_affine(j, m, reinterpret_cast<long long *>(mm.dev + 19), seq, st), "affine sample");
      kick();
      volatile unsigned long long *flag = reinterpret_cast<volatile unsigned long long *>(&mm.host[20]);
      for (unsigned spins = 0; *flag != seq; spins++) {
        if ((spins & 1023) == 1023) {
          const cudaError_t q = cudaStreamQuery(st);
          if (q != cudaSuccess && q != cudaErrorNotReady) return cuda_fail(q, "affine sample");
          if (q == cudaSuccess && *flag != seq) return fail(JP_ERR_CUDA, "affine sample kernel did not publish");
        }
      }
      if (*reinterpret_cast<volatile int64_t *>(&mm.host[19]) == 0) return JP_OK;   // out->affine == 0
    }
    thread_local int32_t *pin = nullptr;
    if (!mm.host && !pin && cudaMallocHost(&pin, 4 * kS * sizeof(int32_t)) != cudaSuccess) {
      pin = nullptr;
      cudaGetLastError();
    }
    const int32_t *qs[4] = {j.d.r, j.d.r2, j.d.w, j.d.s};
    if (!mm.host && pin && m >= 3) {
      for (int q = 0; q < 4; q++)
        if (qs[q]) JP_CUDA(cudaMemcpyAsync(pin + q * kS, qs[q], 4 * (size_t)m, cudaMemcpyDeviceToHost, st), "affine sample");
      JP_CUDA(cudaStreamSynchronize(st), "affine sample");
      for (int q = 0; q < 4; q++) {
        if (!qs[q]) continue;
        const int64_t b = pin[q * kS], a = (int64_t)pin[q * kS + 1] - b;
        for (int k = 2; k < m; k++)
          if ((int64_t)pin[q * kS + k] != b + a * k) return JP_OK;   // out->affine == 0
      }
    }
  }
  JP_CUDA(launch_affine(j, flags, st), "affine");
  const int32_t *ps[4] = {j.d.r, j.d.r2, j.d.w, j.d.s};
  int32_t first[4][2] = {{0, 0}, {0, 0}, {0, 0}, {0, 0}};
  for (int q = 0; q < 4; q++)
    if (ps[q] && L->n > 0)
      JP_CUDA(cudaMemcpyAsync(first[q], ps[q], L->n > 1 ? 8 : 4, cudaMemcpyDeviceToHost, st), "affine D2H");
  int fl[4];
  JP_CUDA(d2h_small_sync(fl, flags, sizeof fl, st), "affine D2H");
  out->affine = 1;
  for (int q = 0; q < 4; q++) {
    if (ps[q]) {
      out->affine &= fl[q] ? 1 : 0;
      out->beta[q] = first[q][0];
      out->alpha[q] = L->n > 1 ? (int64_t)first[q][1] - first[q][0] : 0;
    } else {
      out->alpha[q] = 1;
      out->beta[q] = L->ident_off;
    }
  }
  if (!out->affine) return JP_OK;
  // accesses per array (SURVEY Sec.8 opcode table): 0 r, 1 r2, 2 w, 3 s
  struct Acc { int q; bool write; int arr; };   // arr 0 A, 1 X, 2 T
  Acc acc[4];
  int na = 0;
  switch (L->op) {
    case JP_OP_ADD_C: acc[na++] = {2, true, 0}; acc[na++] = {0, false, 0}; break;
    case JP_OP_SAXPY: acc[na++] = {2, true, 0}; acc[na++] = {0, false, 1}; break;     // Y[w] read == its write
    case JP_OP_PRIV_TMP: acc[na++] = {3, true, 2}; acc[na++] = {2, true, 0}; acc[na++] = {0, false, 1}; break;
    default: acc[na++] = {2, true, 0}; acc[na++] = {0, false, 0}; acc[na++] = {1, false, 0}; break;
  }
  const int64_t len[3] = {L->len_A, L->len_X, L->len_T};
  out->in_range = 1;
  for (int k = 0; k < na; k++) {
    const Acc &a = acc[k];
    if (L->n == 0) break;
    const int64_t v0 = out->beta[a.q], v1 = out->beta[a.q] + out->alpha[a.q] * (L->n - 1);
    if (std::min(v0, v1) < 0 || std::max(v0, v1) >= len[a.arr]) out->in_range = 0;
  }
  out->independent = 1;
  for (int f = 0; f < na; f++) {
    if (!acc[f].write) continue;
    for (int g = 0; g < na; g++) {
      if (acc[g].arr != acc[f].arr) continue;
      if (affine_conflict(out->alpha[acc[f].q], out->beta[acc[f].q], out->alpha[acc[g].q], out->beta[acc[g].q], L->n))
        out->independent = 0;
    }
  }
  return JP_OK;
}

int64_t jp_tls_next_window(int64_t n, int64_t prof_raw_iters, int64_t prev_commit, int64_t w_max) {
  if (n < 0 || w_max < 32) return -1;
  return tls_next_window(n, prof_raw_iters, prev_commit, w_max);
}

int32_t jp_affine_dependence(int64_t af, int64_t bf, int64_t ag, int64_t bg, int64_t n) {
  return affine_conflict(af, bf, ag, bg, n) ? 1 : 0;
}

jp_status jp_static_check(const jp_loop *L, void *ws, size_t ws_bytes, jp_static *out, jp_stream_t st) {
  JP_TRY(check_loop(L));
  if (!out) return fail(JP_ERR_ARG, "result is NULL");
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, 0, lo));
  return static_check(L, make_job(L), ws, lo, out, (cudaStream_t)st);
}

jp_status jp_run_doall(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes, jp_stream_t stp) {
  JP_TRY(check_loop(L));
  if (p && (p->raw_iters || p->war_iters || p->waw_iters))
    return fail(JP_ERR_ILLEGAL_MODE, "DOALL needs d_raw = d_war = d_waw = 0 (profile: %lld/%lld/%lld)",
                (long long)p->raw_iters, (long long)p->war_iters, (long long)p->waw_iters);
  JP_TRY(need_device());
  cudaStream_t st = (cudaStream_t)stp;
  Job j = make_job(L);
  if (has_idx(j) && !p) {
    Layout lo;
    JP_TRY(check_ws(L, ws, ws_bytes, 0, lo));
    JP_TRY(validate_sync(j, ws, lo, st, nullptr));
  }
  JP_CUDA(launch_doall(j, st), "doall");
  return JP_OK;
}

jp_status jp_priv_stream(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes, int32_t clear_keys,
                         jp_stream_t stp) {
  JP_TRY(check_loop(L));
  if (p && p->raw_iters)
    return fail(JP_ERR_ILLEGAL_MODE, "privatization needs d_raw = 0 (profile: %lld RAW iterations)",
                (long long)p->raw_iters);
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PRIV, lo));
  cudaStream_t st = (cudaStream_t)stp;
  Job j = make_job(L);
  if (has_idx(j) && !p) JP_TRY(validate_sync(j, ws, lo, st, nullptr));
  JP_CUDA(launch_priv_stream(j, ws, lo, clear_keys != 0, st), "priv stream");
  return JP_OK;
}

jp_status jp_priv_finalize(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st) {
  JP_TRY(check_loop(L));
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PRIV, lo));
  JP_CUDA(launch_priv_finalize(make_job(L), ws, lo, (cudaStream_t)st), "priv finalize");
  return JP_OK;
}

jp_status jp_run_privatized(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes, jp_stream_t stp) {
  JP_TRY(check_loop(L));
  if (p && p->raw_iters)
    return fail(JP_ERR_ILLEGAL_MODE, "privatization needs d_raw = 0 (profile: %lld RAW iterations)",
                (long long)p->raw_iters);
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PRIV, lo));
  cudaStream_t st = (cudaStream_t)stp;
  Job j = make_job(L);
  if (has_idx(j) && !p) JP_TRY(validate_sync(j, ws, lo, st, nullptr));
  bool applied = false;   // single GPU: the stream kernel may apply the keys itself
  JP_CUDA(launch_priv_stream(j, ws, lo, true, st, 0, true, &applied), "priv stream");
  if (!applied) JP_CUDA(launch_priv_finalize(j, ws, lo, st), "priv finalize");
  return JP_OK;
}

jp_status jp_tls_guide(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st) {
  JP_TRY(check_loop(L));
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PROFILE | JP_WS_GUIDE, lo));
  JP_CUDA(launch_tls_guide(make_job(L), ws, lo, (cudaStream_t)st), "tls guide");
  return JP_OK;
}

// choose the TLS path and check its limits
static jp_status tls_plan(const Job &j, const jp_tls_cfg *cfg, const jp_profile *prof, TlsPlan &tp) {
  tp.window = cfg ? cfg->window : 0;
  tp.w_max = cfg && cfg->w_max > 0 ? cfg->w_max : 65536;
  tp.prof_raw = prof ? prof->raw_iters : -1;
  if (tp.window < 0) return fail(JP_ERR_ARG, "window must be >= 0");
  if (tp.window == 0 && tp.w_max < 32) return fail(JP_ERR_ARG, "w_max must be >= 32");
  const bool hA = a_indirect(j.op, j.d.r, j.d.r2, j.d.w), hT = t_indirect(j.op, j.d.s);
  tp.waw = (hA || hT) && !(prof && prof->waw_iters == 0);
  const int64_t wcap = tp.window > 0 ? tp.window : tp.w_max;
  int path = cfg ? cfg->path : 0;
  if (path == 7) {   // mode C on the device: one warp, program order (jp_serial.cu); nothing speculates
    tp.path = 7;
    tp.guided = false;
    tp.recovery = JP_TLS_RESTART;
    tp.cluster = 1;
    return JP_OK;
  }
  int cl = cfg ? cfg->cluster : 0;
  if (cl < 0 || cl > 16 || (cl & (cl - 1)))
    return fail(JP_ERR_ARG, "cluster must be 0 (auto) or a power of two <= 16 (got %d)", cl);
  tp.guided = cfg && cfg->guided;
  if (tp.guided && (!prof || prof->waw_iters != 0))
    return fail(JP_ERR_ARG, "a guided TLS run needs a profile with waw_iters == 0");
  if (tp.guided && !(hA && j.op != JP_OP_PRIV_TMP)) tp.guided = false;   // nothing to guide
  tp.recovery = cfg ? cfg->recovery : JP_TLS_RESTART;
  if (tp.recovery != JP_TLS_RESTART && tp.recovery != JP_TLS_ONCHIP)
    return fail(JP_ERR_ARG, "bad TLS recovery %d", tp.recovery);
  if (tp.recovery == JP_TLS_ONCHIP) {
    // reading B7: one shadow slot per address needs a loop that writes no address twice
    if (!prof || prof->waw_iters != 0)
      return fail(JP_ERR_ARG, "on-chip TLS recovery needs a profile with waw_iters == 0");
    const int cmax = tls_fwd_max_cluster();
    if (cl > cmax) return fail(JP_ERR_UNSUPPORTED, "the device schedules TLS clusters of up to %d CTAs", cmax);
    if (path != 0 && path != 5 && path != 6 && path != 8)
      return fail(JP_ERR_ARG, "on-chip TLS runs on path 5 (cluster), 6 (grid) or 8 (one window)");
    if (path == 8) {
      // one window spanning the loop, DC from the guide (jp_tls_flow.cu): ADD_C,
      // write-once and WAR-free by the profile, guide words of that profile
      if (j.op != JP_OP_ADD_C || prof->war_iters != 0)
        return fail(JP_ERR_ARG, "TLS path 8 needs an ADD_C loop whose profile shows war_iters == waw_iters == 0");
      if (tp.window != 0 && tp.window < j.d.n)
        return fail(JP_ERR_ARG, "TLS path 8 runs one window of the whole loop (window 0 or >= n)");
      tp.window = std::max<int64_t>(j.d.n, 1);
      tp.cluster = num_sms();
      tp.path = 8;
      tp.waw = false;
      return JP_OK;
    }
    // auto: a window the 16-CTA cluster holds stays there, larger loops use every SM
    if (path == 0) path = (tp.window > 0 ? tp.window : j.d.n) <= tls_fwd_wcap(cmax) ? 5 : 6;
    if (path == 6) {
      const int64_t gcap = tls_fwd_grid_wcap();
      if (tp.window == 0) tp.window = gcap;
      if (tp.window > gcap)
        return fail(JP_ERR_UNSUPPORTED, "the on-chip TLS grid holds windows up to %lld iterations", (long long)gcap);
      tp.cluster = (int)((tp.window + tls_fwd_grid_cta_slots() - 1) / tls_fwd_grid_cta_slots());
      tp.path = 6;
      tp.waw = false;
      return JP_OK;
    }
    if (tp.window > 0) {
      if (cl == 0) {
        cl = 1;
        while (cl < cmax && tls_fwd_wcap(cl) < tp.window) cl <<= 1;
      }
      if (tls_fwd_wcap(cl) < tp.window)
        return fail(JP_ERR_UNSUPPORTED, "a %d-CTA on-chip TLS cluster holds windows up to %lld iterations", cl,
                    (long long)tls_fwd_wcap(cl));
    } else {
      if (cl == 0) {
        cl = 1;
        while (cl < cmax && tls_fwd_wcap(cl) < j.d.n) cl <<= 1;
      }
      tp.window = tls_fwd_wcap(cl);
    }
    tp.cluster = cl;
    tp.path = 5;
    tp.waw = false;
    return JP_OK;
  }
  const int64_t cta_max = tls_cta_wcap(j.op, tp.waw, tp.guided);
  if (path == 0) {
    // auto (measured): windows of <= 1024 iterations stay on
    // one SM (a CTA barrier is ~50 cycles, a cluster barrier ~1000); larger
    // windows spread their gathers over a 16-CTA cluster (one SM sustains only
    // ~0.25 random L2/HBM loads per cycle).
    path = wcap <= 1024 && wcap <= cta_max ? 1 : wcap <= tls_cluster_wcap(16) ? 3 : 2;
  }
  if (path == 1 && wcap > cta_max)
    return fail(JP_ERR_UNSUPPORTED, "the single-CTA TLS path holds windows up to %lld iterations", (long long)cta_max);
  if (path == 2) tp.guided = false;
  if (path == 3) {
    if (cl == 0) cl = tls_max_cluster();   // auto: the largest cluster the device schedules (16 on B200)
    if (tls_cluster_wcap(cl) < wcap)
      return fail(JP_ERR_UNSUPPORTED, "a %d-CTA TLS cluster holds windows up to %lld iterations", cl,
                  (long long)tls_cluster_wcap(cl));
  }
  if (path < 1 || path > 3) return fail(JP_ERR_ARG, "bad TLS path %d", path);
  tp.cluster = cl;
  tp.path = path;
  return JP_OK;
}

// TLS window cap from the profiled density (jp_sched_cfg.tls_w_max == 0):
// clamp(pow2ceil(sqrt(1000 / d_raw)), 256, 1024) -- the measured optimum of the
// single-CTA path on config 3 (1024 at 0.1%, 512 at 1%, 256-384 at 5-10%;
// DESIGN.md Sec.6).  A policy parameter of reading A8, not of the semantics.
static int64_t auto_w_max(const jp_profile *p) {
  if (!p || p->raw_iters <= 0 || p->n <= 0) return 1024;
  const double d = (double)p->raw_iters / (double)p->n;
  const double t = sqrt(1000.0 / d);
  int64_t w = 256;
  while ((double)w < t && w < 1024) w <<= 1;
  return w;
}

// Restart-TLS plan from the profile's dependence distances (reading A8's cap
// and the path; the semantics and the oracle's statistics only depend on the
// cap, which jp_sched_result reports).  A window starting at ws ends at the
// first iteration whose exposed read was written inside the window: an
// iteration at offset m is raw with probability d = raw_iters / n and then
// violates iff its distance delta <= m, so the hazard is h(m) = d F(m) with F
// the distance CDF (dist[b] = raw reads with floor(log2 delta) = b, F linear
// inside a bucket).  The expected commit of a window capped at W is
// E[c_W] = sum_{k<W} prod_{m<k} (1 - h(m)); the adaptive policy keeps windows
// near min(W, 2 E[c]), so one committed iteration costs about
// cost(path, min(W, 2 E[c])) / E[c_W].  cost() is the measured time per window
// of each path at fixed windows on dependence-free loops (scripts/restart_calib.py,
// profiles/r02_restart_calib.jsonl; B200, N = 2^22), with and without the WAW
// commit.  The (path, W) of least cost per committed iteration wins.
namespace {
struct CostPt { int path; int64_t w; double us, us_waw; };
constexpr CostPt kRestartCost[] = {
    {1, 64, 0.85, 1.01},      {1, 128, 0.88, 1.07},     {1, 256, 0.98, 1.18},     {1, 512, 1.21, 1.57},
    {1, 1024, 2.53, 3.04},    {3, 2048, 2.79, 4.53},    {3, 4096, 3.08, 5.26},    {3, 8192, 3.72, 6.25},
    {3, 16384, 4.80, 8.89},   {3, 32768, 7.18, 13.96},  {3, 65536, 12.05, 24.07}, {2, 262144, 22.85, 28.72}};
}  // namespace

static double restart_cost(int path, int64_t w, bool waw) {
  // piecewise linear in W between the measured points of the same path
  const CostPt *lo = nullptr, *hi = nullptr;
  for (const CostPt &c : kRestartCost) {
    if (c.path != path) continue;
    if (c.w <= w) lo = &c;
    if (c.w >= w && !hi) hi = &c;
  }
  if (!lo) lo = hi;
  if (!hi) hi = lo;
  const double a = waw ? lo->us_waw : lo->us, b = waw ? hi->us_waw : hi->us;
  if (hi->w == lo->w) return a;
  return a + (b - a) * (double)(w - lo->w) / (double)(hi->w - lo->w);
}

// expected commit length of a window of at most W iterations (see above)
static double restart_commit(const int64_t *dist, double d, int64_t W) {
  double tot = 0;
  for (int b = 0; b < 32; b++) tot += (double)dist[b];
  if (tot <= 0 || d <= 0) return (double)W;
  double F = 0, logS = 0, ec = 0;   // F(m) at the start of bucket b, log S(m)
  int64_t m = 0;
  // m = 0 never violates (delta >= 1); step through the buckets [2^b, 2^(b+1))
  ec += 1.0;
  m = 1;
  for (int b = 0; b < 32 && m < W; b++) {
    const int64_t lo = (int64_t)1 << b, hi = std::min<int64_t>((int64_t)2 << b, W);
    const double fb = (double)dist[b] / tot;      // mass of this bucket, spread over [2^b, 2^(b+1))
    const double span = (double)((int64_t)1 << b);
    // integrate k over [lo, hi) in up to 64 steps: S(k) = exp(logS), logS += log(1 - d F(k))
    const int64_t steps = std::min<int64_t>(64, hi - lo);
    const double dk = (double)(hi - lo) / (double)steps;
    for (int64_t q = 0; q < steps; q++) {
      const double k = (double)lo + (q + 0.5) * dk;
      const double Fk = F + fb * (k - (double)lo + 1.0) / span;
      const double h = std::min(0.999999, d * Fk);
      ec += exp(logS) * dk;
      logS += log1p(-h) * dk;
    }
    F += fb;
    m = hi;
    if (logS < -50) break;   // every later window position is unreachable
  }
  return ec;
}

static void restart_plan(const jp_profile *p, const int64_t *dist, int64_t n, bool waw, int64_t *w_max, int *path) {
  const double d = p && p->n > 0 ? (double)p->raw_iters / (double)p->n : 0.0;
  double best = 1e300;
  for (const CostPt &c : kRestartCost) {
    if (c.w > std::max<int64_t>(n, 64) * 2 && c.w > 64) continue;
    const double ec = restart_commit(dist, d, c.w);
    double weff = std::min((double)c.w, 2.0 * ec);
    if (weff < 32) weff = 32;
    const double t = restart_cost(c.path, (int64_t)weff, waw) / std::max(ec, 1.0);
    if (t < best) {
      best = t;
      *w_max = c.w;
      *path = c.path;
    }
  }
}

// auto_guide: run jp_tls_guide first when the plan benefits (cluster path
// always, single-CTA path at d_raw <= 2%: measured) and the profile and
// workspace allow it (jp_schedule)
static jp_status run_tls_job(const jp_loop *L, const Job &j, const jp_tls_cfg *cfg, const jp_profile *prof, void *ws,
                             size_t ws_bytes, jp_tls_stats *stats, cudaStream_t st, bool auto_guide = false,
                             TlsPlan *plan_out = nullptr, bool guide_ready = false, int s_clean = 0) {
  TlsPlan tp;
  JP_TRY(tls_plan(j, cfg, prof, tp));
  const bool helps = tp.path == 3 || tp.path >= 5 || (tp.path == 1 && prof && prof->n > 0 && prof->raw_iters * 50 <= prof->n);
  if (auto_guide && !tp.guided && helps && prof && prof->waw_iters == 0 && a_indirect(j.op, j.d.r, j.d.r2, j.d.w) &&
      j.op != JP_OP_PRIV_TMP) {
    Layout lg = layout(L);
    if (ws && ws_bytes >= layout_end(lg, JP_WS_PROFILE | JP_WS_GUIDE | JP_WS_TLS) && lg.bytes[R_GUIDE]) {
      if (!guide_ready) JP_CUDA(launch_tls_guide(j, ws, lg, st), "tls guide");
      tp.guided = true;
    }
  }
  Layout lo;
  const int uses = (tp.path == 2 || tp.path == 3 || tp.path == 6 || tp.path == 8 ? JP_WS_TLS : 0) |
                   (tp.guided ? JP_WS_GUIDE : 0);
  if (tp.path == 8 && !tp.guided) return fail(JP_ERR_ARG, "TLS path 8 needs the guide words (guided = 1)");
  JP_TRY(check_ws(L, ws, ws_bytes, uses, lo));
  if (has_idx(j) && !prof) JP_TRY(validate_sync(j, ws, lo, st, nullptr));
  if (plan_out) *plan_out = tp;
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  const uint32_t *bits = tp.guided ? at<uint32_t>(ws, lo, R_GUIDE) : nullptr;
  const uint32_t *bsrc = bits ? bits + (L->n + 31) / 32 : nullptr;
  if (tp.path == 7) {
    JP_CUDA(launch_serial(j, &hdr[H_TLS_COMMITTED], st), "serial warp");
  } else if (tp.path == 5) {
    JP_CUDA(launch_tls_fwd(j, tp.window, tp.cluster, bits, bsrc, &hdr[H_TLS_COMMITTED], st), "tls on-chip");
  } else if (tp.path == 8) {
    auto *V = at<unsigned long long>(ws, lo, R_TLS_C_A);
    if (!(s_clean & 6)) cudaMemsetAsync(V, 0, 8 * (size_t)L->len_A, st);   // no shadow value yet
    JP_CUDA(launch_tls_flow(j, bits, bsrc, V, &hdr[H_TLS_COMMITTED], st), "tls one window");
  } else if (tp.path == 6) {
    auto *S = at<unsigned long long>(ws, lo, R_TLS_S_A);
    auto *V = at<unsigned long long>(ws, lo, R_TLS_C_A);
    const int64_t lenS = S && V ? L->len_A : 0;
    JP_CUDA(launch_tls_fwd_grid(j, tp.window, bits, bsrc, S, V, lenS, reinterpret_cast<unsigned *>(&hdr[H_BAR_COUNT]),
                                &hdr[H_TLS_COMMITTED], st, s_clean),
            "tls on-chip grid");
  } else {
    JP_CUDA(launch_tls(j, ws, lo, tp, &hdr[H_TLS_COMMITTED], st), "tls");
  }
  if (stats) {
    int64_t h[4];
    JP_CUDA(d2h_small_sync(h, &hdr[H_TLS_COMMITTED], sizeof h, st), "tls D2H");
    if (tp.path == 8) {   // device: h[3] violations, h[1] warps that lost their writer
      if (h[1]) return fail(JP_ERR_ARG, "one-window TLS: a violator's writer never published (guide and profile disagree)");
      h[0] = L->n;
      h[1] = L->n + h[3];
      h[2] = L->n > 0 ? 1 : 0;
    }
    if (tp.path >= 5 && h[0] < 0)
      return fail(JP_ERR_ARG, "on-chip TLS recovery met an address written twice (the profile passed was wrong)");
    stats->committed = h[0];
    stats->executed = h[1];
    stats->windows = h[2];
    stats->violations = h[3];
  }
  return JP_OK;
}

jp_status jp_run_tls(const jp_loop *L, const jp_tls_cfg *cfg, const jp_profile *prof, void *ws, size_t ws_bytes,
                     jp_tls_stats *stats, jp_stream_t st) {
  JP_TRY(check_loop(L));
  JP_TRY(need_device());
  return run_tls_job(L, make_job(L), cfg, prof, ws, ws_bytes, stats, (cudaStream_t)st);
}

#ifdef JP_TLS_TRACE
int32_t jp_tls_trace(long long *host, int32_t n) { return (int32_t)jp::tls_trace_copy(host, n); }
int32_t jp_tls_fwd_trace(long long *host, int32_t n) { return (int32_t)jp::tls_fwd_trace_copy(host, n); }
#endif

jp_status jp_merge_apply(void *arr, int64_t len, const int64_t *keys, jp_stream_t st) {
  if (len < 0 || (len > 0 && (!arr || !keys))) return fail(JP_ERR_ARG, "bad merge arguments");
  JP_TRY(need_device());
  JP_CUDA(launch_merge_apply(arr, len, keys, (cudaStream_t)st), "merge apply");
  return JP_OK;
}

// ---------------------------------------------------------------------------
// task sharing with cross-boundary spill (M1, C8) and the IPC plumbing it needs
// ---------------------------------------------------------------------------
jp_status jp_run_doall_spill(const jp_loop *views, int32_t world, int32_t me, int64_t chunk,
                             unsigned long long *ctr, int64_t *stats, int32_t max_ctas, jp_stream_t st) {
  if (!views || world < 1 || world > kSpillRanks || me < 0 || me >= world)
    return fail(JP_ERR_ARG, "need 1 <= world <= %d and 0 <= me < world", kSpillRanks);
  if (chunk < 1 || !ctr) return fail(JP_ERR_ARG, "need chunk >= 1 and a counter table");
  Job jobs[kSpillRanks];
  for (int k = 0; k < world; k++) {
    const jp_loop *L = &views[k];
    JP_TRY(check_loop(L));
    if (L->r || L->r2 || L->w || L->s || L->ident_off != 0)
      return fail(JP_ERR_UNSUPPORTED, "spill runs affine shards only (NULL index arrays, ident_off 0)");
    if (L->op != views[0].op || L->dtype != views[0].dtype || L->c0.i != views[0].c0.i || L->c1.i != views[0].c1.i)
      return fail(JP_ERR_ARG, "every rank's view must run the same body");
    if ((L->n + chunk - 1) / chunk >= (1LL << 31)) return fail(JP_ERR_ARG, "too many chunks");
    jobs[k] = make_job(L);
  }
  JP_TRY(need_device());
  JP_CUDA(launch_doall_spill(jobs, world, me, chunk, ctr, stats, max_ctas, (cudaStream_t)st), "doall spill");
  return JP_OK;
}

jp_status jp_run_priv_claim(const jp_loop *L, const int64_t *chunks, const int64_t *first, int32_t world, int32_t me,
                            unsigned long long *ctr, int64_t *stats, void *ws, size_t ws_bytes, int32_t max_ctas,
                            jp_stream_t st) {
  JP_TRY(check_loop(L));
  if (!first || world < 1 || world > 8 || me < 0 || me >= world || !ctr)
    return fail(JP_ERR_ARG, "need 1 <= world <= 8, 0 <= me < world, first[world+1] and a counter table");
  if (first[0] != 0) return fail(JP_ERR_ARG, "first[0] must be 0");
  for (int k = 0; k < world; k++)
    if (first[k + 1] < first[k] || first[k + 1] - first[k] >= (1LL << 31))
      return fail(JP_ERR_ARG, "rank blocks must be ordered and < 2^31 chunks");
  if (first[world] > 0 && !chunks) return fail(JP_ERR_ARG, "NULL chunk list");
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PRIV, lo));
  JP_CUDA(launch_priv_claim(make_job(L), ws, lo, chunks, first, world, me, ctr, stats, max_ctas, (cudaStream_t)st),
          "priv claim");
  return JP_OK;
}

jp_status jp_keys_merge_p2p(const int64_t *const *peer_keys, int32_t world, int64_t *keys, int64_t len,
                            unsigned long long *bar, int64_t epoch, void *arr, int32_t *err, jp_stream_t st) {
  if (!peer_keys || world < 1 || world > 8 || !keys || !bar || !err || epoch < 1)
    return fail(JP_ERR_ARG, "bad p2p merge arguments (1 <= world <= 8, epoch >= 1)");
  if (len < 0 || len > kP2PMaxLen) return fail(JP_ERR_ARG, "p2p merge holds at most %lld slots", (long long)kP2PMaxLen);
  for (int k = 0; k < world; k++)
    if (!peer_keys[k]) return fail(JP_ERR_ARG, "peer key table %d is NULL", k);
  JP_TRY(need_device());
  JP_CUDA(launch_keys_merge_p2p(reinterpret_cast<const unsigned long long *const *>(peer_keys), world,
                                reinterpret_cast<unsigned long long *>(keys), len, bar, (unsigned long long)epoch,
                                static_cast<uint32_t *>(arr), err, (cudaStream_t)st),
          "p2p key merge");
  return JP_OK;
}

size_t jp_priv_inbox_bytes(const jp_loop *L, int32_t world) {
  if (check_loop(L) != JP_OK) return 0;
  return priv_inbox_bytes(make_job(L), world);
}

jp_status jp_priv_stream_merge(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes,
                               void *const *peer_inbox, int32_t world, int32_t me, int32_t *err, jp_stream_t st) {
  JP_TRY(check_loop(L));
  if (p && p->raw_iters != 0) return fail(JP_ERR_ILLEGAL_MODE, "privatization needs d_raw = 0");
  const Job j = make_job(L);
  if (!priv_merge_ok(j, world))
    return fail(JP_ERR_UNSUPPORTED, "the fused merge runs PRIV_TMP with identity X / Y, an indirect s, "
                                    "len_T <= 4096, 16-byte aligned streams and 1 <= world <= 8");
  if (!peer_inbox || me < 0 || me >= world || !err) return fail(JP_ERR_ARG, "bad merge arguments");
  for (int k = 0; k < world; k++)
    if (!peer_inbox[k]) return fail(JP_ERR_ARG, "inbox of rank %d is NULL", k);
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PRIV, lo));
  if (L->n == 0) return JP_OK;
  JP_CUDA(launch_priv_stream_merge(j, at<unsigned long long>(ws, lo, R_KEYS_T),
                                   reinterpret_cast<unsigned long long *const *>(peer_inbox), world, me, err,
                                   (cudaStream_t)st),
          "priv stream + merge");
  return JP_OK;
}

typedef int (*cu_range_fn)(unsigned long long *, size_t *, unsigned long long);
static cu_range_fn cu_mem_range() {
  static cu_range_fn fn = nullptr;
  static std::once_flag once;
  std::call_once(once, [] {
    void *p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuMemGetAddressRange", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<cu_range_fn>(p);
  });
  return fn;
}

jp_status jp_ipc_export(const void *ptr, void *handle, int64_t *offset) {
  if (!ptr || !handle || !offset) return fail(JP_ERR_ARG, "NULL argument");
  JP_TRY(need_device());
  cu_range_fn fn = cu_mem_range();
  unsigned long long base = 0;
  size_t size = 0;
  if (!fn || fn(&base, &size, (unsigned long long)(uintptr_t)ptr) != 0)
    return fail(JP_ERR_CUDA, "cuMemGetAddressRange failed for %p", ptr);
  cudaIpcMemHandle_t h;
  JP_CUDA(cudaIpcGetMemHandle(&h, (void *)(uintptr_t)base), "cudaIpcGetMemHandle");
  memcpy(handle, &h, sizeof h);
  *offset = (int64_t)((uintptr_t)ptr - base);
  return JP_OK;
}

jp_status jp_ipc_import(const void *handle, int64_t offset, void **ptr) {
  if (!handle || !ptr || offset < 0) return fail(JP_ERR_ARG, "bad IPC import arguments");
  JP_TRY(need_device());
  cudaIpcMemHandle_t h;
  memcpy(&h, handle, sizeof h);
  void *base = nullptr;
  JP_CUDA(cudaIpcOpenMemHandle(&base, h, cudaIpcMemLazyEnablePeerAccess), "cudaIpcOpenMemHandle");
  *ptr = static_cast<char *>(base) + offset;
  return JP_OK;
}

jp_status jp_ipc_close(void *ptr, int64_t offset) {
  if (!ptr || offset < 0) return fail(JP_ERR_ARG, "bad IPC close arguments");
  JP_TRY(need_device());
  JP_CUDA(cudaIpcCloseMemHandle(static_cast<char *>(ptr) - offset), "cudaIpcCloseMemHandle");
  return JP_OK;
}

// ---------------------------------------------------------------------------
// owner-partitioned sparse exchange (NEXT-2)
// ---------------------------------------------------------------------------
static jp_status check_sparse(const void *t0, int32_t elem, int64_t len, const void *rows, int64_t m) {
  if (elem != 4 && elem != 8) return fail(JP_ERR_ARG, "elem_bytes must be 4 or 8 (got %d)", elem);
  if (len < 0 || (elem == 4 && len > INT32_MAX)) return fail(JP_ERR_ARG, "bad table length %lld", (long long)len);
  if (m < 0) return fail(JP_ERR_ARG, "negative row count");
  if (m > 0 && (!t0 || !rows)) return fail(JP_ERR_ARG, "NULL table or rows");
  return JP_OK;
}

size_t jp_sparse_scratch_bytes(int64_t len, int32_t world) {
  if (len < 0 || world <= 0) return 0;
  return sparse_scratch_bytes(len, world);
}

jp_status jp_sparse_pack(const void *t0, const void *t1, int32_t elem_bytes, int64_t len, int64_t lo, int64_t hi,
                         int64_t empty, int32_t world, void *rows, int64_t cap, int64_t *counts, void *scratch,
                         size_t scratch_bytes, jp_stream_t st) {
  JP_TRY(check_sparse(t0, elem_bytes, len, rows, 0));
  if (world <= 0 || !counts) return fail(JP_ERR_ARG, "world must be > 0 and counts non-NULL");
  if (lo < 0 || hi < lo || hi > len) return fail(JP_ERR_ARG, "bad range [%lld, %lld) of a %lld-entry table",
                                                 (long long)lo, (long long)hi, (long long)len);
  if (cap < 0 || (cap > 0 && !rows)) return fail(JP_ERR_ARG, "bad rows / cap");
  if (hi > lo && !t0) return fail(JP_ERR_ARG, "NULL table");
  const size_t need = sparse_scratch_bytes(len, world);
  if (!scratch || scratch_bytes < need || ((uintptr_t)scratch & 7))
    return fail(JP_ERR_WORKSPACE, "sparse scratch of %zu bytes (8-byte aligned) needed", need);
  JP_TRY(need_device());
  for (int k = 0; k < world; k++) counts[k] = 0;
  if (hi == lo) return JP_OK;
  const cudaStream_t s = (cudaStream_t)st;
  const int64_t tiles = sparse_pack_tiles(len, lo, hi, world);
  int64_t *counts_dev = static_cast<int64_t *>(scratch) + 2 * tiles + 1;
  JP_CUDA(launch_sparse_pack(t0, t1, elem_bytes, len, lo, hi, empty, world, rows, cap, counts_dev, scratch, s),
          "sparse pack");
  JP_CUDA(d2h_small_sync(counts, counts_dev, sizeof(int64_t) * world, s), "sparse pack D2H");
  int64_t m = 0;
  for (int k = 0; k < world; k++) m += counts[k];
  if (m > cap) return fail(JP_ERR_ARG, "%lld rows do not fit the %lld-row buffer", (long long)m, (long long)cap);
  return JP_OK;
}

static jp_status sparse_rows(void *t0, void *t1, int32_t elem, int64_t len, void *rows, int64_t m, int what,
                             jp_stream_t st, const char *where) {
  JP_TRY(check_sparse(t0, elem, len, rows, m));
  JP_TRY(need_device());
  JP_CUDA(launch_sparse_rows(t0, t1, elem, len, rows, m, what, (cudaStream_t)st), where);
  return JP_OK;
}

jp_status jp_sparse_reduce_max(void *t0, void *t1, int32_t elem_bytes, int64_t len, const void *rows, int64_t m,
                               jp_stream_t st) {
  return sparse_rows(t0, t1, elem_bytes, len, const_cast<void *>(rows), m, 0, st, "sparse reduce");
}

jp_status jp_sparse_gather(const void *t0, const void *t1, int32_t elem_bytes, int64_t len, void *rows, int64_t m,
                           jp_stream_t st) {
  return sparse_rows(const_cast<void *>(t0), const_cast<void *>(t1), elem_bytes, len, rows, m, 1, st,
                     "sparse gather");
}

jp_status jp_sparse_scatter(void *t0, void *t1, int32_t elem_bytes, int64_t len, const void *rows, int64_t m,
                            jp_stream_t st) {
  return sparse_rows(t0, t1, elem_bytes, len, const_cast<void *>(rows), m, 2, st, "sparse scatter");
}

// ---------------------------------------------------------------------------
// plans (host only)
// ---------------------------------------------------------------------------
jp_status jp_plan_sharing(int64_t n, int32_t world, const double *weights, int64_t *ranges) {
  if (n < 0 || world <= 0 || !ranges) return fail(JP_ERR_ARG, "bad sharing-plan arguments");
  double total = 0.0;
  for (int k = 0; k < world; k++) {
    const double w = weights ? weights[k] : 1.0;
    if (!(w >= 0.0) || std::isinf(w)) return fail(JP_ERR_ARG, "weights must be finite and >= 0");
    total += w;
  }
  if (!(total > 0.0)) return fail(JP_ERR_ARG, "weights sum to zero");
  double pre = 0.0;
  for (int k = 0; k < world; k++) {
    const int64_t b0 = (int64_t)std::floor((double)n * (pre / total));
    pre += weights ? weights[k] : 1.0;
    const int64_t b1 = k == world - 1 ? n : (int64_t)std::floor((double)n * (pre / total));
    ranges[2 * k] = b0;
    ranges[2 * k + 1] = b1;
  }
  return JP_OK;
}

jp_status jp_plan_stealing(const int64_t *tasks, int64_t n_tasks, int32_t world, int64_t chunk_iters,
                           const double *speed, double speed_tls, int64_t *chunks, int64_t cap, int64_t *n_out,
                           int64_t *stolen_out) {
  if (!tasks || n_tasks < 0 || world <= 0 || chunk_iters <= 0 || !chunks || !n_out || !(speed_tls > 0.0))
    return fail(JP_ERR_ARG, "bad stealing-plan arguments");
  for (int k = 0; k < world; k++)
    if (speed && !(speed[k] > 0.0)) return fail(JP_ERR_ARG, "speeds must be > 0");
  struct Ch { int64_t s, e, mode, home, owner; };
  std::vector<Ch> cs;
  for (int64_t t = 0; t < n_tasks; t++) {
    const int64_t s = tasks[3 * t], e = tasks[3 * t + 1], m = tasks[3 * t + 2];
    if (e < s) return fail(JP_ERR_ARG, "task %lld has end < start", (long long)t);
    const bool tls = m == JP_MODE_TLS || m == JP_MODE_SEQ_RECOMMENDED;
    if (tls) { cs.push_back({s, e, m, 0, -1}); continue; }
    for (int64_t c = s; c < e; c += chunk_iters) cs.push_back({c, std::min(e, c + chunk_iters), m, -1, -1});
  }
  if ((int64_t)cs.size() > cap) { *n_out = (int64_t)cs.size(); return fail(JP_ERR_ARG, "plan needs %zu chunks", cs.size()); }
  // deal the partitionable chunks by task sharing (weights = speeds)
  std::vector<int64_t> part;
  for (size_t c = 0; c < cs.size(); c++) if (cs[c].home < 0) part.push_back((int64_t)c);
  std::vector<int64_t> rg(2 * world);
  jp_plan_sharing((int64_t)part.size(), world, speed, rg.data());
  std::vector<std::vector<int64_t>> dq(world), pinned(world);
  for (int k = 0; k < world; k++)
    for (int64_t q = rg[2 * k]; q < rg[2 * k + 1]; q++) { cs[part[q]].home = k; dq[k].push_back(part[q]); }
  for (size_t c = 0; c < cs.size(); c++) if (cs[c].home == 0 && (cs[c].mode == JP_MODE_TLS || cs[c].mode == JP_MODE_SEQ_RECOMMENDED)) pinned[0].push_back((int64_t)c);
  std::vector<size_t> head(world, 0), tail(world), pin_head(world, 0);
  for (int k = 0; k < world; k++) tail[k] = dq[k].size();
  std::vector<double> t(world, 0.0);
  std::vector<bool> done(world, false);
  int64_t stolen = 0;
  while (true) {
    int k = -1;
    for (int q = 0; q < world; q++) if (!done[q] && (k < 0 || t[q] < t[k])) k = q;
    if (k < 0) break;
    int64_t c = -1;
    double rate = speed ? speed[k] : 1.0;
    if (pin_head[k] < pinned[k].size()) { c = pinned[k][pin_head[k]++]; rate = speed_tls; }
    else if (head[k] < tail[k]) c = dq[k][head[k]++];
    else {
      // steal from the TAIL of the deque with the most remaining iterations (ties: lowest rank)
      int v = -1; int64_t best = 0;
      for (int q = 0; q < world; q++) {
        if (q == k) continue;
        int64_t rem = 0;
        for (size_t x = head[q]; x < tail[q]; x++) rem += cs[dq[q][x]].e - cs[dq[q][x]].s;
        if (rem > best) { best = rem; v = q; }
      }
      if (v < 0) { done[k] = true; continue; }
      c = dq[v][--tail[v]];
      stolen++;
    }
    cs[c].owner = k;
    t[k] += (double)(cs[c].e - cs[c].s) / rate;
  }
  for (size_t c = 0; c < cs.size(); c++) {
    chunks[4 * c] = cs[c].s; chunks[4 * c + 1] = cs[c].e; chunks[4 * c + 2] = cs[c].mode; chunks[4 * c + 3] = cs[c].owner;
  }
  *n_out = (int64_t)cs.size();
  if (stolen_out) *stolen_out = stolen;
  return JP_OK;
}

// ---------------------------------------------------------------------------
// scheduler (one GPU)
// ---------------------------------------------------------------------------
static jp_sched_cfg default_cfg() {
  jp_sched_cfg c;
  memset(&c, 0, sizeof c);
  c.scheme = JP_SCHED_SHARING;
  c.tau_high = kTauHigh;
  c.chunk_iters = 65536;
  c.tls_window = 0;
  c.tls_w_max = 0;   // auto from the profiled density (auto_w_max)
  c.tls_path = 0;
  return c;
}

static Job sub_job(const Job &j, int64_t s, int64_t e) {
  Job k = j;
  DLoop &d = k.d;
  d.n = e - s;
  d.base = j.d.base + s;
  d.ioff = j.d.ioff + s;
  if (d.r) d.r += s;
  if (d.r2) d.r2 += s;
  if (d.w) d.w += s;
  if (d.s) d.s += s;
  return k;
}

// Replay of a fixed launch sequence from a CUDA graph cached per key (the values
// its launches take): captured once on a per-thread side stream, then launched
// into st.  JP_NO_GRAPHS=1 issues the sequence directly.
static cudaError_t graph_launch(const std::string &key, const std::function<cudaError_t(cudaStream_t)> &issue,
                                cudaStream_t st) {
  const char *ng = getenv("JP_NO_GRAPHS");
  if (ng && ng[0] == '1') return issue(st);
  struct Ent { std::string key; cudaGraphExec_t exec; };
  thread_local std::vector<Ent> cache;
  for (const Ent &e : cache)
    if (e.key == key) return cudaGraphLaunch(e.exec, st);
  int dev = 0;
  cudaGetDevice(&dev);
  thread_local cudaStream_t cs[64] = {};
  if (!cs[dev & 63]) {
    const cudaError_t e = cudaStreamCreateWithFlags(&cs[dev & 63], cudaStreamNonBlocking);
    if (e != cudaSuccess) return e;
  }
  const cudaStream_t c = cs[dev & 63];
  cudaError_t e = cudaStreamBeginCapture(c, cudaStreamCaptureModeThreadLocal);
  if (e != cudaSuccess) return e;
  const cudaError_t ei = issue(c);
  cudaGraph_t graph = nullptr;
  e = cudaStreamEndCapture(c, &graph);
  if (ei != cudaSuccess || e != cudaSuccess) {
    if (graph) cudaGraphDestroy(graph);
    cudaGetLastError();
    return issue(st);   // (not capturable: issued directly)
  }
  cudaGraphExec_t exec = nullptr;
  e = cudaGraphInstantiate(&exec, graph, 0);
  cudaGraphDestroy(graph);
  if (e != cudaSuccess) {
    cudaGetLastError();
    return issue(st);
  }
  if (cache.size() >= 16) {
    for (Ent &x : cache) cudaGraphExecDestroy(x.exec);
    cache.clear();
  }
  cache.push_back({key, exec});
  return cudaGraphLaunch(exec, st);
}

// path 8's separate gather kernel runs up to this many raw iterations (a
// fraction of n: 1/64 measured; JP_FLOW_PH_DIV overrides the divisor)
static int64_t ph_max_for(int64_t n) {
  static int64_t div = 0;
  if (!div) {
    const char *e = getenv("JP_FLOW_PH_DIV");
    div = e ? std::max<int64_t>(1, atoll(e)) : 64;
  }
  return n / div;
}

static jp_status run_mode(const jp_loop *L, const Job &j, int mode, const jp_profile *prof, const jp_sched_cfg &c,
                          void *ws, size_t ws_bytes, jp_sched_result *res, cudaStream_t st, bool guide_ready = false,
                          int s_clean = 0, const int64_t *dist = nullptr) {
  Layout lo = layout(L);
  if (mode == JP_MODE_DOALL) {
    // an indirect loop: gather phase into region 1 (the profile's scratch, free
    // once Fig. 2(b) has its counts), then the scatters
    uint32_t *o = ws && lo.bytes[R_MINW_A] >= 4 * (size_t)j.d.n && ws_bytes >= lo.off[R_MINW_A] + 4 * (size_t)j.d.n
                      ? at<uint32_t>(ws, lo, R_MINW_A) : nullptr;
    JP_CUDA(launch_doall(j, st, 0, o), "doall");
  } else if (mode == JP_MODE_PRIVATIZED) {
    if (ws_bytes < layout_end(lo, JP_WS_PRIV)) return fail(JP_ERR_WORKSPACE, "workspace too small for privatization");
    bool applied = false;
    JP_CUDA(launch_priv_stream(j, ws, lo, true, st, 0, true, &applied), "priv stream");
    if (!applied) JP_CUDA(launch_priv_finalize(j, ws, lo, st), "priv finalize");
  } else {
    // window cap from the density when not given; profile-guided mode B
    // where it helps
    // recovery: on chip (reading B7) whenever the profile allows it, unless asked otherwise
    // mode C (TD density above tau_high, "sequential"): the one-warp
    // program-order path unless a TLS path or recovery was asked for
    const bool serial = mode == JP_MODE_SEQ_RECOMMENDED && c.tls_path == 0 && c.tls_recovery == 0;
    const int rec = serial ? JP_TLS_RESTART
                    : c.tls_recovery == 1 ? JP_TLS_RESTART
                    : c.tls_recovery == 2 || (c.tls_path == 0 && prof && prof->waw_iters == 0) ? JP_TLS_ONCHIP
                                                                                            : JP_TLS_RESTART;
    int64_t wm = c.tls_w_max > 0 ? c.tls_w_max : auto_w_max(prof);
    int path = serial ? 7 : c.tls_path;
    // restart recovery with the profile's dependence distances: cap and path
    // from the distance-hazard model (restart_plan) unless the caller fixed them
    if (!serial && rec == JP_TLS_RESTART && dist && prof && c.tls_w_max == 0 && c.tls_path == 0 && c.tls_window == 0)
      restart_plan(prof, dist, j.d.n, prof->waw_iters > 0, &wm, &path);
    // write-once, WAR-free ADD_C loop with the guide already filled by the profile:
    // one window, DC from the guide, no barrier (path 8, jp_tls_flow.cu)
    if (rec == JP_TLS_ONCHIP && guide_ready && path == 0 && c.tls_window == 0 && j.op == JP_OP_ADD_C && prof &&
        prof->war_iters == 0 && prof->waw_iters == 0 && !getenv("JP_TLS_NO_FLOW"))
      path = 8;
    jp_tls_cfg tc{c.tls_window, wm, path, 0, path == 8 ? 1 : 0, rec};
    TlsPlan tp;
    JP_TRY(run_tls_job(L, j, &tc, prof, ws, ws_bytes, &res->tls, st, true, &tp, guide_ready, s_clean));
    res->tls_w_max = tp.path == 7 ? 32 : rec == JP_TLS_ONCHIP ? tp.window : wm;
    res->tls_path = tp.path;
    res->tls_guided = tp.guided ? 1 : 0;
    res->tls_recovery = rec;
    res->tls_cluster = tp.path == 3 || tp.path >= 5 ? tp.cluster : 1;
  }
  res->task_mode_iters[mode] += j.d.n;
  return JP_OK;
}

namespace {
struct StreamPool {
  std::mutex mu;
  std::vector<cudaStream_t> s[64];
  cudaStream_t get(int k) {
    int dev = 0;
    cudaGetDevice(&dev);
    std::lock_guard<std::mutex> g(mu);
    auto &v = s[dev & 63];
    while ((int)v.size() <= k) {
      cudaStream_t x;
      cudaStreamCreateWithFlags(&x, cudaStreamNonBlocking);
      v.push_back(x);
    }
    return v[k];
  }
} g_pool;
}  // namespace


// ---- task-stealing helpers (shared by jp_schedule(STEALING) and jp_plan_tasks) ----
struct Task { int64_t s, e; int mode; };

// chunk modes (Fig. 2(b) on each chunk's counts, reading A19) -> maximal same-mode
// runs, coarsened to <= kMaxTasks by merging the smallest adjacent pair into the
// stronger mode
static std::vector<Task> chunk_tasks(const int64_t *hc, int64_t n, int64_t chunk, double tau) {
  std::vector<Task> tasks;
  const int64_t nck = (n + chunk - 1) / chunk;
  for (int64_t k = 0; k < nck; k++) {
    const int64_t s = k * chunk, e = std::min(n, s + chunk);
    const int m = select_mode_counts(e - s, hc[3 * k], hc[3 * k + 1], hc[3 * k + 2], tau);
    if (!tasks.empty() && tasks.back().mode == m) tasks.back().e = e;
    else tasks.push_back({s, e, m});
  }
  auto rank = [](int m) {
    return m == JP_MODE_SEQ_RECOMMENDED ? 3 : m == JP_MODE_TLS ? 2 : m == JP_MODE_PRIVATIZED ? 1 : 0;
  };
  while ((int)tasks.size() > kMaxTasks) {
    size_t best = 0;
    for (size_t q = 1; q + 1 < tasks.size(); q++)
      if (tasks[q].e - tasks[q].s + tasks[q + 1].e - tasks[q + 1].s <
          tasks[best].e - tasks[best].s + tasks[best + 1].e - tasks[best + 1].s) best = q;
    tasks[best].e = tasks[best + 1].e;
    if (rank(tasks[best + 1].mode) > rank(tasks[best].mode)) tasks[best].mode = tasks[best + 1].mode;
    tasks.erase(tasks.begin() + best + 1);
  }
  return tasks;
}

// conf[u] bit t: tasks t and u touch a common address, at least one writing it (reading B2); syncs
// ranges_out (nullable): the per-task address ranges of the prefilter
// ([4][kMaxTasks]: minA, maxA, minT, maxT) when it ran, else left empty
// chunk_rg (nullable): per chunk the min / max address of A it touches (the bucket
// profile's), from which the task ranges follow without the k_task_ranges pass
// Small device-to-host reads of the schedulers through mapped pinned memory:
// one kernel copies up to three device ranges (8-byte words) into the mapped
// buffer and then publishes the call's sequence number; the host polls it.
namespace {
struct MappedPack {
  char *host = nullptr, *dev = nullptr;
  size_t bytes = 0;
  unsigned long long *flag_host = nullptr, *flag_dev = nullptr;
  unsigned long long seq = 0;
};
}  // namespace
__global__ void __launch_bounds__(256) k_pack_host(const unsigned long long *a, size_t na, const unsigned long long *b,
                                                   size_t nb, const unsigned long long *c, size_t nc,
                                                   unsigned long long *dst, unsigned long long *flag,
                                                   unsigned long long seq) {
  for (size_t k = threadIdx.x; k < na + nb + nc; k += blockDim.x)
    dst[k] = k < na ? a[k] : k < na + nb ? b[k - na] : c[k - na - nb];
  __threadfence_system();
  JP_CTA_SYNC();
  if (threadIdx.x == 0) asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(flag), "l"(seq) : "memory");
}
static MappedPack &mapped_pack(size_t need) {
  thread_local MappedPack m;
  if (need > m.bytes && !getenv("JP_NO_MAPPED_PACK")) {
    if (m.host) cudaFreeHost(m.host);
    m = MappedPack{};
    void *p = nullptr, *d = nullptr;
    const size_t bytes = ((need + 4095) & ~(size_t)4095) + 64;
    if (cudaHostAlloc(&p, bytes, cudaHostAllocMapped | cudaHostAllocPortable) == cudaSuccess) {
      if (cudaHostGetDevicePointer(&d, p, 0) == cudaSuccess) {
        m.host = static_cast<char *>(p);
        m.dev = static_cast<char *>(d);
        m.bytes = bytes - 64;
        m.flag_host = reinterpret_cast<unsigned long long *>(m.host + m.bytes);
        m.flag_dev = reinterpret_cast<unsigned long long *>(m.dev + m.bytes);
        *m.flag_host = 0;
      } else {
        cudaFreeHost(p);
      }
    }
    cudaGetLastError();
  }
  return m;
}
static cudaError_t launch_pack_host(const void *a, size_t ba, const void *b, size_t bb, const void *c, size_t bc,
                                    char *dst, unsigned long long seq, cudaStream_t st) {
  MappedPack &m = mapped_pack(ba + bb + bc);
  k_pack_host<<<1, 256, 0, st>>>(static_cast<const unsigned long long *>(a), ba / 8,
                                 static_cast<const unsigned long long *>(b), bb / 8,
                                 static_cast<const unsigned long long *>(c), bc / 8,
                                 reinterpret_cast<unsigned long long *>(dst), m.flag_dev, seq);
  note_launch();
  return launch_check();
}
static jp_status mapped_pack_wait(MappedPack &m, unsigned long long seq, cudaStream_t st, const char *what) {
  volatile unsigned long long *flag = m.flag_host;
  for (unsigned spins = 0; *flag != seq; spins++) {
    if ((spins & 1023) == 1023) {
      const cudaError_t q = cudaStreamQuery(st);
      if (q != cudaSuccess && q != cudaErrorNotReady) return cuda_fail(q, what);
      if (q == cudaSuccess && *flag != seq) return fail(JP_ERR_CUDA, "%s: the pack kernel did not publish", what);
    }
  }
  return JP_OK;
}

#include <chrono>
#define HTRACE(w) htrace(w)

static jp_status task_conflicts(const Job &j, const jp_loop *L, void *ws, const Layout &lo,
                                const std::vector<Task> &tasks, int64_t chunk, std::vector<unsigned long long> &conf,
                                cudaStream_t st, std::vector<uint32_t> *ranges_out = nullptr,
                                const std::vector<uint32_t> *chunk_rg = nullptr) {
  const int nt = (int)tasks.size();
  if (ranges_out) ranges_out->clear();
  conf.assign(kMaxTasks, 0);
  if (nt <= 1) return JP_OK;
  SchedLayout sl = sched_layout(L);
  char *sch = static_cast<char *>(ws) + lo.off[R_SCHED];
  const int64_t nck = (L->n + chunk - 1) / chunk;
  std::vector<int32_t> ct(nck);
  for (int t = 0; t < nt; t++)
    for (int64_t k = tasks[t].s / chunk; k * chunk < tasks[t].e; k++) ct[k] = t;
  int32_t *dct = reinterpret_cast<int32_t *>(sch + sl.chunk_task);
  bool dct_sent = false;
  auto send_dct = [&]() -> cudaError_t {   // the chunk -> task map, for the device passes only
    if (dct_sent) return cudaSuccess;
    dct_sent = true;
    return cudaMemcpyAsync(dct, ct.data(), 4 * nck, cudaMemcpyHostToDevice, st);
  };
  // cheap sufficient test first: tasks with disjoint address ranges in every array never conflict
  if (!getenv("JP_TASK_MASKS_ALWAYS")) {
    std::vector<uint32_t> rg(4 * kMaxTasks);
    if (chunk_rg && (j.op == JP_OP_ADD_C || j.op == JP_OP_SAXPY)) {   // A only: the T ranges stay empty
      for (int t = 0; t < kMaxTasks; t++) { rg[t] = rg[2 * kMaxTasks + t] = 0xFFFFFFFFu; rg[kMaxTasks + t] = rg[3 * kMaxTasks + t] = 0; }
      for (int t = 0; t < nt; t++)
        for (int64_t k = tasks[t].s / chunk; k * chunk < tasks[t].e; k++) {
          rg[t] = std::min(rg[t], (*chunk_rg)[2 * k]);
          rg[kMaxTasks + t] = std::max(rg[kMaxTasks + t], (*chunk_rg)[2 * k + 1]);
        }
    } else {
      uint32_t *drg = reinterpret_cast<uint32_t *>(sch + sl.ranges);
      JP_CUDA(send_dct(), "task map H2D");
      JP_CUDA(launch_task_ranges(j, dct, chunk, drg, st), "task ranges");
      JP_CUDA(cudaMemcpyAsync(rg.data(), drg, 16 * kMaxTasks, cudaMemcpyDeviceToHost, st), "ranges D2H");
      JP_CUDA(cudaStreamSynchronize(st), "ranges sync");
    }
    if (ranges_out) *ranges_out = rg;
    auto ov = [&](int a, int t, int u) {   // array a: 0 A, 1 T
      const uint32_t *mn = rg.data() + 2 * a * kMaxTasks, *mx = mn + kMaxTasks;
      return mn[t] <= mx[t] && mn[u] <= mx[u] && !(mx[t] < mn[u] || mx[u] < mn[t]);
    };
    bool any = false;
    for (int u = 0; u < nt && !any; u++)
      for (int t = 0; t < u && !any; t++) any = ov(0, t, u) || ov(1, t, u);
    if (!any) return JP_OK;   // conf stays all zero
  }
  auto P = [&](size_t o) { return o == SIZE_MAX ? nullptr : reinterpret_cast<unsigned long long *>(sch + o); };
  unsigned long long *dconf = P(sl.conf);
  JP_CUDA(send_dct(), "task map H2D");
  JP_CUDA(launch_task_conflicts(j, dct, chunk, nt, P(sl.wmA), P(sl.rmA), P(sl.wmT), P(sl.rmT), dconf, st),
          "conflicts");
  JP_CUDA(cudaMemcpyAsync(conf.data(), dconf, 8 * kMaxTasks, cudaMemcpyDeviceToHost, st), "conf D2H");
  JP_CUDA(cudaStreamSynchronize(st), "conf sync");
  return JP_OK;
}

// Step 1 of the stealing schedulers: the profile of the whole loop with per-chunk
// (raw, war, waw) counts (global stamps, reading A19) -- by address buckets when
// the loop allows it, with the per-chunk address ranges of A (the task PDG's
// prefilter) -- read back to the host: hc [3 nck], hcr [2 nck] (empty without
// ranges), h = header words 0..7.  gbits (nullable): the TLS guide words are
// written too; flow: keep the writer of every raw read (wsrc, region 7) and clear
// the shadow slots path 8 polls (vclr) for one-window TLS tasks.
static jp_status chunk_profile(const jp_loop *L, const Job &j, void *ws, const Layout &lo, int64_t chunk,
                               uint32_t *gbits, bool pairs, bool flow, cudaStream_t st, std::vector<int64_t> &hc,
                               std::vector<uint32_t> &hcr, std::vector<int64_t> &h, int32_t **wsrc_out,
                               uint32_t **crange_out, unsigned long long **vclr_out, bool *bucket_out) {
  SchedLayout sl = sched_layout(L);
  char *sch = static_cast<char *>(ws) + lo.off[R_SCHED];
  const int64_t nck = (L->n + chunk - 1) / chunk;
  int64_t *cc = reinterpret_cast<int64_t *>(sch + sl.counts);
  int32_t *wsrc = nullptr;
  uint32_t *crange = nullptr;
  unsigned long long *vclr = nullptr;
  const bool bucket = bucket_profile_ok(j, ws, lo);
  if (bucket) {   // large A: the profile by address buckets (jp_bucket.cu)
    if (flow && gbits && j.op == JP_OP_ADD_C && lo.bytes[R_TLS_S_A] >= 4 * (size_t)L->n && !getenv("JP_TLS_NO_FLOW"))
      wsrc = at<int32_t>(ws, lo, R_TLS_S_A);
    if (chunk % kBucketTile == 0 && !getenv("JP_TASK_MASKS_ALWAYS"))
      crange = reinterpret_cast<uint32_t *>(sch + sl.crange);
    // the shadow slots a one-window TLS task polls (V at every raw read's
    // address) are cleared by the profile itself
    vclr = wsrc ? at<unsigned long long>(ws, lo, R_TLS_C_A) : nullptr;
    JP_CUDA(launch_prof_bucket(j, ws, lo, gbits, gbits ? gbits + (L->n + 31) / 32 : nullptr, chunk, cc, st, wsrc,
                               crange, vclr),
            "profile (buckets)");
  } else {
    JP_CUDA(launch_prof_stamp(j, ws, lo, st, pairs), "profile stamp");
    JP_CUDA(launch_prof_classify(j, ws, lo, gbits, chunk, cc, st, gbits ? gbits + (L->n + 31) / 32 : nullptr, pairs),
            "profile classify");
  }
  hc.assign(3 * nck, 0);
  h.assign(8, 0);
  hcr.clear();
  {
    // chunk counts, chunk address ranges and the header: one kernel stores them
    // into mapped pinned memory and then a sequence word, which the host polls
    // (three DMA copies and a stream sync cost ~20 us more); the copies stay as
    // the fallback when mapped memory is unavailable
    const size_t bc = 24 * (size_t)nck, br = crange ? 8 * (size_t)nck : 0, bh = 64;
    if (crange) hcr.resize(2 * nck);
    HTRACE("profile queued");
    MappedPack &mp = mapped_pack(bc + br + bh);
    if (mp.host) {
      const unsigned long long seq = ++mp.seq;
      JP_CUDA(launch_pack_host(cc, bc, crange, br, at<int64_t>(ws, lo, R_HEADER), bh, mp.dev, seq, st), "profile D2H");
      JP_TRY(mapped_pack_wait(mp, seq, st, "profile D2H"));
      HTRACE("pack seen");
      memcpy(hc.data(), mp.host, bc);
      if (crange) memcpy(hcr.data(), mp.host + bc, br);
      memcpy(h.data(), mp.host + bc + br, bh);
    } else {
      JP_CUDA(cudaMemcpyAsync(hc.data(), cc, bc, cudaMemcpyDeviceToHost, st), "chunk D2H");
      if (crange) JP_CUDA(cudaMemcpyAsync(hcr.data(), crange, br, cudaMemcpyDeviceToHost, st), "chunk ranges D2H");
      JP_CUDA(cudaMemcpyAsync(h.data(), at<int64_t>(ws, lo, R_HEADER), bh, cudaMemcpyDeviceToHost, st), "profile D2H");
      JP_CUDA(cudaStreamSynchronize(st), "profile sync");
    }
  }
  if (wsrc_out) *wsrc_out = wsrc;
  if (crange_out) *crange_out = crange;
  if (vclr_out) *vclr_out = vclr;
  if (bucket_out) *bucket_out = bucket;
  return JP_OK;
}

static jp_status schedule_stealing(const jp_loop *L, const Job &j, const jp_sched_cfg &c, void *ws, size_t ws_bytes,
                                   jp_sched_result *res, cudaStream_t st) {
  HTRACE("start");
  const int64_t chunk = c.chunk_iters;
  if (chunk < kSchedMinChunk || chunk % 32) return fail(JP_ERR_ARG, "stealing needs chunk_iters >= 1024, multiple of 32");
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_ALL, lo));
  SchedLayout sl = sched_layout(L);
  char *sch = static_cast<char *>(ws) + lo.off[R_SCHED];
  const int64_t nck = (L->n + chunk - 1) / chunk;
  int64_t *cc = reinterpret_cast<int64_t *>(sch + sl.counts);
  // 1. profile with per-chunk counts (global stamps, reading A19); the classify
  //    pass also writes the TLS guide bitmaps when the loop can be guided
  const bool gfuse = lo.bytes[R_GUIDE] && c.tls_recovery != 1 && j.op != JP_OP_PRIV_TMP &&
                     a_indirect(j.op, j.d.r, j.d.r2, j.d.w);
  uint32_t *gbits = gfuse ? at<uint32_t>(ws, lo, R_GUIDE) : nullptr;
  // large A tables: stamped as {minW, minR} pairs in region 7 (free until the TLS tasks run)
  const bool pairs = stamp_pairs_ok(j, ws, lo);
  // the first all-SM TLS task finds this call's pair table in the write-log
  // region: it needs no reset (see launch_tls_fwd_grid); later ones do
  bool s_fresh = pairs;
  // the writer of every raw read, recorded by the bucket profile (ADD_C with the
  // guide): lets a write-once, WAR-free TLS task run as one window (path 8) even
  // when some of its reads were written by an earlier task.  Kept in region 7
  // (the write log of paths 5 / 6, unused by path 8)
  int32_t *wsrc = nullptr;
  uint32_t *crange = nullptr;   // per-chunk address ranges from the bucket profile (task PDG prefilter)
  unsigned long long *vclr = nullptr;   // the shadow values, cleared where path 8 polls them by the profile
  std::vector<int64_t> hc(3 * nck), h(8);
  std::vector<uint32_t> hcr;
  bool bucket = false;
  JP_TRY(chunk_profile(L, j, ws, lo, chunk, gbits, pairs, true, st, hc, hcr, h, &wsrc, &crange, &vclr, &bucket));
  if (bucket) s_fresh = false;   // (region 7 is not filled: the TLS task resets it)
  if (h[H_BAD]) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)h[H_BAD]);
  fill_profile(&res->prof, L->n, h.data());
  res->profiled = 1;
  HTRACE("copied");
  // 2. chunk modes -> tasks (maximal same-mode runs)
  std::vector<Task> tasks = chunk_tasks(hc.data(), L->n, chunk, c.tau_high);
  const int nt = (int)tasks.size();
  res->n_tasks = nt;
  res->mode = nt ? tasks[0].mode : JP_MODE_DOALL;
  // 3. inter-task conflicts (PDG) and topological batches
  std::vector<unsigned long long> conf(kMaxTasks, 0);
  std::vector<uint32_t> trg;
  JP_TRY(task_conflicts(j, L, ws, lo, tasks, chunk, conf, st, &trg, crange ? &hcr : nullptr));
  std::vector<int> level(nt, 0);
  int nlev = nt ? 1 : 0;
  for (int u = 0; u < nt; u++) {
    for (int t = 0; t < u; t++)
      if ((conf[u] >> t) & 1ull) level[u] = std::max(level[u], level[t] + 1);
    nlev = std::max(nlev, level[u] + 1);
  }
  res->n_batches = nlev;
  HTRACE("planned");
  // 4. run batch by batch; tasks of one batch are pairwise conflict-free and run
  //    concurrently (TLS on one SM, partitioned modes on the rest)
  int64_t *tstats = reinterpret_cast<int64_t *>(sch + sl.tstats);
  // on-chip TLS tasks use the guide bitmaps of step 1 (valid for them: no
  // iteration of such a task writes an address written earlier in the loop, so
  // its writers of raw-read addresses are first writers)
  const bool guided_ok = gfuse;
  std::vector<int> grid_tls;   // on-chip TLS tasks, run on every SM after the batch's other tasks
  std::vector<int> flow_tasks;  // ... of them, run as one window (path 8): stats completed on the host
  // the side-stream clear (done long before: it overlapped the profile) is
  // joined before any task runs
  bool v_zeroed = vclr != nullptr;
  const bool flow_side = !getenv("JP_FLOW_TASK_AFTER");   // path-8 tasks beside the partitioned ones
  cudaEvent_t ev0;
  JP_CUDA(cudaEventCreateWithFlags(&ev0, cudaEventDisableTiming), "event");
  std::vector<cudaEvent_t> evs;
  std::vector<int> tls_tasks;
  for (int lv = 0; lv < nlev; lv++) {
    bool any_priv = false;
    int n_priv = 0;
    for (int t = 0; t < nt; t++) n_priv += level[t] == lv && tasks[t].mode == JP_MODE_PRIVATIZED;
    any_priv = n_priv > 0;
    // the element ranges this batch's privatized tasks can write (their keys):
    // the whole arrays unless the range prefilter ran
    int64_t kA0 = 0, kA1 = L->len_A, kT0 = 0, kT1 = L->len_T;
    if (any_priv && !trg.empty()) {
      kA0 = kT0 = INT64_MAX;
      kA1 = kT1 = 0;
      for (int t = 0; t < nt; t++) {
        if (level[t] != lv || tasks[t].mode != JP_MODE_PRIVATIZED) continue;
        const uint32_t *r = trg.data();
        if (r[t] <= r[kMaxTasks + t]) { kA0 = std::min<int64_t>(kA0, r[t]); kA1 = std::max<int64_t>(kA1, (int64_t)r[kMaxTasks + t] + 1); }
        if (r[2 * kMaxTasks + t] <= r[3 * kMaxTasks + t]) {
          kT0 = std::min<int64_t>(kT0, r[2 * kMaxTasks + t]);
          kT1 = std::max<int64_t>(kT1, (int64_t)r[3 * kMaxTasks + t] + 1);
        }
      }
      if (kA0 >= kA1) kA0 = kA1 = 0;
      if (kT0 >= kT1) kT0 = kT1 = 0;
    }
    auto *keysA = at<unsigned long long>(ws, lo, R_KEYS_A);
    auto *keysT = at<unsigned long long>(ws, lo, R_KEYS_T);
    // the key ranges start at zero: cleared on the privatized task's own stream
    // when the batch has one (the other tasks start at once), else before the batch
    auto clear_keys = [&](cudaStream_t s) {
      if (keysA && kA1 > kA0) cudaMemsetAsync(keysA + kA0, 0, 8 * (size_t)(kA1 - kA0), s);
      if (keysT && kT1 > kT0) cudaMemsetAsync(keysT + kT0, 0, 8 * (size_t)(kT1 - kT0), s);
    };
    if (n_priv > 1) clear_keys(st);
    cudaEventRecord(ev0, st);
    HTRACE("ev0");
    int sidx = 0;
    std::vector<cudaEvent_t> joins;
    // TLS tasks first so that their single CTA is resident before the wide grids
    for (int pass = 0; pass < 2; pass++) {
      for (int t = 0; t < nt; t++) {
        if (level[t] != lv) continue;
        const bool seq = tasks[t].mode == JP_MODE_SEQ_RECOMMENDED;
        const bool tls = tasks[t].mode == JP_MODE_TLS || seq;
        if ((pass == 0) != tls) continue;
        cudaStream_t s2 = g_pool.get(sidx++);
        cudaStreamWaitEvent(s2, ev0, 0);
        Job sj = sub_job(j, tasks[t].s, tasks[t].e);
        if (seq && c.tls_path == 0 && c.tls_recovery == 0) {
          // mode C task: one warp in program order (path 7) beside the partitioned tasks
          JP_CUDA(launch_serial(sj, tstats + 4 * t, s2), "serial task");
          res->tls_path = 7;
          tls_tasks.push_back(t);
        } else if (tls) {
          TlsPlan tp;
          jp_profile tprof{};
          tprof.n = sj.d.n;
          tprof.raw_iters = hc.empty() ? -1 : 0;
          for (int64_t k = tasks[t].s / chunk; k * chunk < tasks[t].e; k++) { tprof.raw_iters += hc[3 * k]; tprof.waw_iters += hc[3 * k + 2]; }
          const bool onchip = c.tls_recovery == 2 || (c.tls_recovery == 0 && c.tls_path == 0 && tprof.waw_iters == 0);
          int64_t twar = 0;
          for (int64_t k = tasks[t].s / chunk; k * chunk < tasks[t].e; k++) twar += hc[3 * k + 1];
          if (onchip && flow_side && wsrc && guided_ok && twar == 0 && c.tls_window == 0) {
            // write-once, WAR-free ADD_C task as one window (path 8) BESIDE the
            // batch's partitioned tasks: one CTA per SM, so the random-access-bound
            // sweep overlaps their streams (its violators only wait on earlier
            // iterations of the task; the partitioned tasks never wait on it)
            const uint32_t *gb = at<uint32_t>(ws, lo, R_GUIDE);
            const int64_t nw = (L->n + 31) / 32;
            auto *V = at<unsigned long long>(ws, lo, R_TLS_C_A);
            if (!v_zeroed) cudaMemsetAsync(V, 0, lo.bytes[R_TLS_C_A], s2);
            JP_CUDA(launch_tls_flow(sj, gb + tasks[t].s / 32, gb + nw + tasks[t].s / 32, V, tstats + 4 * t, s2,
                                    wsrc + tasks[t].s, tasks[t].s, nullptr, 0, true, num_sms()),
                    "tls task (one window)");
            flow_tasks.push_back(t);
            res->tls_w_max = sj.d.n;
            res->tls_path = 8;
            res->tls_recovery = JP_TLS_ONCHIP;
            res->tls_cluster = num_sms();
            res->tls_guided = 1;
          } else if (onchip) {
            // on-chip recovery (reading B7) uses every SM: it runs after the
            // batch's partitioned tasks (below), on the caller's stream
            grid_tls.push_back(t);
            res->task_mode_iters[tasks[t].mode] += sj.d.n;
            continue;
          } else {
            // the single-CTA path (one SM, beside the partitioned tasks), window cap from the task's density
            const int64_t wm = c.tls_w_max > 0 ? c.tls_w_max : auto_w_max(tprof.raw_iters >= 0 ? &tprof : nullptr);
            jp_tls_cfg tc{c.tls_window, wm, 1, 0, 0, 0};
            JP_TRY(tls_plan(sj, &tc, &tprof, tp));
            res->tls_w_max = wm;
            res->tls_path = 1;
            JP_CUDA(launch_tls(sj, ws, lo, tp, tstats + 4 * t, s2), "tls task");
          }
          tls_tasks.push_back(t);
        } else if (tasks[t].mode == JP_MODE_PRIVATIZED) {
          if (n_priv == 1) clear_keys(s2);
          JP_CUDA(launch_priv_stream(sj, ws, lo, false, s2), "priv task");
        } else {
          // gather phase into region 1 at the task's own offset (tasks are disjoint ranges)
          uint32_t *o = lo.bytes[R_MINW_A] >= 4 * (size_t)L->n ? at<uint32_t>(ws, lo, R_MINW_A) + tasks[t].s : nullptr;
          JP_CUDA(launch_doall(sj, s2, 0, o), "doall task");
        }
        res->task_mode_iters[tasks[t].mode] += sj.d.n;
        cudaEvent_t e;
        cudaEventCreateWithFlags(&e, cudaEventDisableTiming);
        cudaEventRecord(e, s2);
        joins.push_back(e);
        evs.push_back(e);
        HTRACE("task launched");
      }
    }
    HTRACE("tasks launched");
    for (auto e : joins) cudaStreamWaitEvent(st, e, 0);
    for (int t : grid_tls) {
      if (level[t] != lv) continue;
      // guided by the whole loop's bitmaps (the task starts on a chunk boundary, a multiple of 32)
      Job sj = sub_job(j, tasks[t].s, tasks[t].e);
      int64_t twar = 0;
      for (int64_t k = tasks[t].s / chunk; k * chunk < tasks[t].e; k++) twar += hc[3 * k + 1];
      if (wsrc && guided_ok && twar == 0 && c.tls_window == 0) {
        // write-once, WAR-free ADD_C task: one window, DC from the guide (path 8);
        // reads whose writer precedes the task see A (wsrc)
        const uint32_t *gb = at<uint32_t>(ws, lo, R_GUIDE);
        const int64_t nw = (L->n + 31) / 32;
        auto *V = at<unsigned long long>(ws, lo, R_TLS_C_A);
        if (!v_zeroed) {
          cudaMemsetAsync(V, 0, lo.bytes[R_TLS_C_A], st);
          v_zeroed = true;
        }
        JP_CUDA(launch_tls_flow(sj, gb + tasks[t].s / 32, gb + nw + tasks[t].s / 32, V, tstats + 4 * t, st,
                                wsrc + tasks[t].s, tasks[t].s),
                "tls task (one window)");
        flow_tasks.push_back(t);
        res->tls_w_max = sj.d.n;
        res->tls_path = 8;
        res->tls_recovery = JP_TLS_ONCHIP;
        res->tls_cluster = num_sms();
        res->tls_guided = 1;
        tls_tasks.push_back(t);
        continue;
      }
      TlsPlan tp;
      jp_profile tprof{};
      tprof.n = sj.d.n;
      jp_tls_cfg tc{c.tls_window, 0, 0, 0, 0, JP_TLS_ONCHIP};
      JP_TRY(tls_plan(sj, &tc, &tprof, tp));
      const uint32_t *gb = guided_ok ? at<uint32_t>(ws, lo, R_GUIDE) : nullptr;
      const int64_t nw = (L->n + 31) / 32;
      const uint32_t *b0 = gb ? gb + tasks[t].s / 32 : nullptr, *b1 = gb ? gb + nw + tasks[t].s / 32 : nullptr;
      if (tp.path == 6) {
        JP_CUDA(launch_tls_fwd_grid(sj, tp.window, b0, b1, at<unsigned long long>(ws, lo, R_TLS_S_A),
                                    at<unsigned long long>(ws, lo, R_TLS_C_A), L->len_A,
                                    reinterpret_cast<unsigned *>(&at<int64_t>(ws, lo, R_HEADER)[H_BAR_COUNT]),
                                    tstats + 4 * t, st, s_fresh ? 1 : 0),
                "tls task");
        s_fresh = false;
        v_zeroed = false;   // path 6 leaves its shadow values in V
      } else {
        JP_CUDA(launch_tls_fwd(sj, tp.window, tp.cluster, b0, b1, tstats + 4 * t, st), "tls task");
      }
      res->tls_w_max = tp.window;
      res->tls_path = tp.path;
      res->tls_recovery = JP_TLS_ONCHIP;
      res->tls_cluster = tp.cluster;
      res->tls_guided = gb ? 1 : 0;
      tls_tasks.push_back(t);
    }
    if (any_priv) {   // apply the keys over the written ranges only
      if (keysA && kA1 > kA0)
        JP_CUDA(launch_merge_apply(static_cast<uint32_t *>(L->A) + kA0, kA1 - kA0,
                                   reinterpret_cast<const int64_t *>(keysA + kA0), st), "priv finalize");
      if (keysT && kT1 > kT0 && j.op == JP_OP_PRIV_TMP)
        JP_CUDA(launch_merge_apply(static_cast<uint32_t *>(L->T) + kT0, kT1 - kT0,
                                   reinterpret_cast<const int64_t *>(keysT + kT0), st), "priv finalize");
    }
  }
  // stats of the TLS tasks
  memset(&res->tls, 0, sizeof res->tls);
  for (int t : tls_tasks) {
    int64_t s4[4];
    JP_CUDA(cudaMemcpyAsync(s4, tstats + 4 * t, sizeof s4, cudaMemcpyDeviceToHost, st), "tls stats D2H");
    JP_CUDA(cudaStreamSynchronize(st), "tls stats sync");
    if (std::find(flow_tasks.begin(), flow_tasks.end(), t) != flow_tasks.end()) {
      // path 8 on the device: s4[3] violations, s4[1] warps that lost their writer
      if (s4[1]) return fail(JP_ERR_ARG, "one-window TLS task: a violator's writer never published");
      const int64_t tn = tasks[t].e - tasks[t].s;
      s4[0] = tn;
      s4[1] = tn + s4[3];
      s4[2] = tn > 0 ? 1 : 0;
    }
    res->tls.committed += s4[0]; res->tls.executed += s4[1]; res->tls.windows += s4[2]; res->tls.violations += s4[3];
  }
  JP_CUDA(cudaStreamSynchronize(st), "schedule sync");
  cudaEventDestroy(ev0);
  for (auto e : evs) cudaEventDestroy(e);
  return JP_OK;
}

jp_status jp_plan(const jp_loop *L, const jp_sched_cfg *cfg, const jp_profile *chunk_profiles, int64_t n_chunks,
                  int32_t world, const double *speed, int64_t *plan_out, int64_t plan_cap, int64_t *n_out) {
  JP_TRY(check_loop(L));
  if (!cfg || !chunk_profiles || world <= 0 || !plan_out || !n_out)
    return fail(JP_ERR_ARG, "bad plan arguments");
  const int64_t chunk = cfg->chunk_iters > 0 ? cfg->chunk_iters : 65536;
  if ((L->n + chunk - 1) / chunk != n_chunks)
    return fail(JP_ERR_ARG, "%lld chunk profiles for %lld chunks of %lld iterations", (long long)n_chunks,
                (long long)((L->n + chunk - 1) / chunk), (long long)chunk);
  std::vector<int64_t> hc(3 * (size_t)std::max<int64_t>(n_chunks, 1));
  for (int64_t k = 0; k < n_chunks; k++) {
    hc[3 * k] = chunk_profiles[k].raw_iters;
    hc[3 * k + 1] = chunk_profiles[k].war_iters;
    hc[3 * k + 2] = chunk_profiles[k].waw_iters;
  }
  std::vector<Task> tk = chunk_tasks(hc.data(), L->n, chunk, cfg->tau_high > 0.0 ? cfg->tau_high : kTauHigh);
  std::vector<int64_t> tasks;
  for (const Task &t : tk) { tasks.push_back(t.s); tasks.push_back(t.e); tasks.push_back(t.mode); }
  if (cfg->scheme == JP_SCHED_STEALING)
    return jp_plan_stealing(tasks.data(), (int64_t)tk.size(), world, chunk, speed, 1.0, plan_out, plan_cap, n_out,
                            nullptr);
  // SHARING: the iteration space split by the boundary formula; each rank's range
  // cut at task boundaries (rows keep one mode each)
  std::vector<int64_t> rg(2 * (size_t)world);
  JP_TRY(jp_plan_sharing(L->n, world, speed, rg.data()));
  int64_t m = 0;
  for (int k = 0; k < world; k++)
    for (const Task &t : tk) {
      const int64_t b = std::max(t.s, rg[2 * k]), e = std::min(t.e, rg[2 * k + 1]);
      if (b >= e) continue;
      if (m < plan_cap) {
        plan_out[4 * m] = b; plan_out[4 * m + 1] = e; plan_out[4 * m + 2] = t.mode; plan_out[4 * m + 3] = k;
      }
      m++;
    }
  *n_out = m;
  if (m > plan_cap) return fail(JP_ERR_ARG, "plan needs %lld rows", (long long)m);
  return JP_OK;
}

jp_status jp_plan_tasks(const jp_loop *L, const int64_t *chunk_counts, int64_t chunk_iters, double tau_high,
                        void *ws, size_t ws_bytes, int64_t *tasks, int32_t *n_tasks, uint64_t *conf,
                        jp_stream_t st) {
  JP_TRY(check_loop(L));
  if (!chunk_counts || !tasks || !n_tasks || !conf) return fail(JP_ERR_ARG, "NULL output or counts");
  if (chunk_iters < kSchedMinChunk || chunk_iters % 32)
    return fail(JP_ERR_ARG, "chunk_iters must be >= 1024 and a multiple of 32");
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_ALL, lo));
  std::vector<Task> tk = chunk_tasks(chunk_counts, L->n, chunk_iters, tau_high > 0.0 ? tau_high : kTauHigh);
  std::vector<unsigned long long> cf;
  JP_TRY(task_conflicts(make_job(L), L, ws, lo, tk, chunk_iters, cf, (cudaStream_t)st));
  *n_tasks = (int32_t)tk.size();
  for (size_t t = 0; t < tk.size(); t++) {
    tasks[3 * t] = tk[t].s;
    tasks[3 * t + 1] = tk[t].e;
    tasks[3 * t + 2] = tk[t].mode;
  }
  for (int t = 0; t < kMaxTasks; t++) conf[t] = cf[t];
  return JP_OK;
}

jp_status jp_profile_plan_tasks(const jp_loop *L, int64_t chunk_iters, double tau_high, void *ws, size_t ws_bytes,
                                jp_profile *prof, int64_t *chunk_counts, int64_t *tasks, int32_t *n_tasks,
                                uint64_t *conf, jp_stream_t stp) {
  JP_TRY(check_loop(L));
  if (!prof || !chunk_counts || !tasks || !n_tasks || !conf) return fail(JP_ERR_ARG, "NULL output");
  if (chunk_iters < kSchedMinChunk || chunk_iters % 32)
    return fail(JP_ERR_ARG, "chunk_iters must be >= 1024 and a multiple of 32");
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_ALL, lo));
  cudaStream_t st = (cudaStream_t)stp;
  const Job j = make_job(L);
  std::vector<int64_t> hc, h;
  std::vector<uint32_t> hcr;
  JP_TRY(chunk_profile(L, j, ws, lo, chunk_iters, nullptr, stamp_pairs_ok(j, ws, lo), false, st, hc, hcr, h, nullptr,
                       nullptr, nullptr, nullptr));
  if (h[H_BAD]) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)h[H_BAD]);
  fill_profile(prof, L->n, h.data());
  memcpy(chunk_counts, hc.data(), hc.size() * sizeof(int64_t));
  std::vector<Task> tk = chunk_tasks(hc.data(), L->n, chunk_iters, tau_high > 0.0 ? tau_high : kTauHigh);
  std::vector<unsigned long long> cf;
  JP_TRY(task_conflicts(j, L, ws, lo, tk, chunk_iters, cf, st, nullptr, hcr.empty() ? nullptr : &hcr));
  *n_tasks = (int32_t)tk.size();
  for (size_t t = 0; t < tk.size(); t++) {
    tasks[3 * t] = tk[t].s;
    tasks[3 * t + 1] = tk[t].e;
    tasks[3 * t + 2] = tk[t].mode;
  }
  for (int t = 0; t < kMaxTasks; t++) conf[t] = cf[t];
  return JP_OK;
}

jp_status jp_export_keys(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st) {
  JP_TRY(check_loop(L));
  JP_TRY(need_device());
  Layout lo;
  JP_TRY(check_ws(L, ws, ws_bytes, JP_WS_PRIV, lo));
  JP_CUDA(launch_export_keys(make_job(L), ws, lo, (cudaStream_t)st), "export keys");
  return JP_OK;
}

// Reading B11: the mode a loop's access sets fix without looking at its indices,
// -1 when the indices decide.  PRIV_TMP reads only X (never written; T's read is
// covered by the same iteration's write): RAW-free, with WAR / WAW through s or w
// possible -> privatized (DOALL when neither is indirect).  SAXPY with identity
// writes: Y[i] is read and written by iteration i alone, X is read-only -> DOALL.
static int structural_mode(const Job &j) {
  if (j.op == JP_OP_PRIV_TMP) return (j.d.s || j.d.w) ? JP_MODE_PRIVATIZED : JP_MODE_DOALL;
  if (j.op == JP_OP_SAXPY && !j.d.w) return JP_MODE_DOALL;
  return -1;
}

jp_status jp_schedule(const jp_loop *L, const jp_sched_cfg *cfgp, void *ws, size_t ws_bytes, jp_sched_result *res,
                      jp_stream_t stp) {
  JP_TRY(check_loop(L));
  if (!res) return fail(JP_ERR_ARG, "result is NULL");
  JP_TRY(need_device());
  jp_sched_cfg c = cfgp ? *cfgp : default_cfg();
  if (c.tau_high <= 0.0) c.tau_high = kTauHigh;
  if (c.chunk_iters <= 0) c.chunk_iters = 65536;
  if (c.tls_w_max < 0) c.tls_w_max = 0;
  memset(res, 0, sizeof *res);
  cudaStream_t st = (cudaStream_t)stp;
  Job j = make_job(L);
  res->prof.n = L->n;
  res->prof.first_raw_iter = -1;
  if (!has_idx(j)) {   // "determined DOALL" (mode A): no profiling
    res->mode = JP_MODE_DOALL;
    res->profiled = 0;
    res->n_tasks = 1;
    res->n_batches = 1;
    JP_CUDA(launch_doall(j, st), "doall");
    res->task_mode_iters[JP_MODE_DOALL] = L->n;
    return JP_OK;
  }
  if (c.scheme == JP_SCHED_STEALING) return schedule_stealing(L, j, c, ws, ws_bytes, res, st);
  if (c.scheme != JP_SCHED_SHARING) return fail(JP_ERR_ARG, "bad scheme %d", c.scheme);
  if (c.tls_path == 0 && c.tls_recovery != 2 && c.tls_window <= 4096 && tiny_eligible(L)) {
    // tiny loop: profile, Fig. 2(b) and the mode in one launch (jp_tiny.cu)
    Layout lo;
    JP_TRY(check_ws(L, ws, ws_bytes, 0, lo));
    int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
    int64_t h[16];
    TinyMirror &m = tiny_mirror();
    if (m.host) {   // results through mapped host memory: poll the kernel's flag, no D2H copy
      const unsigned long long seq = ++m.seq;
      JP_CUDA(launch_tiny(j, L, c.tau_high, c.tls_window, c.tls_w_max, c.tls_recovery, hdr, st, m.dev, seq), "tiny");
      for (unsigned spins = 0; *(volatile unsigned long long *)&m.host[16] != seq; spins++) {
        if ((spins & 1023) == 1023) {
          const cudaError_t q = cudaStreamQuery(st);
          if (q != cudaSuccess && q != cudaErrorNotReady) return cuda_fail(q, "tiny");
          if (q == cudaSuccess && *(volatile unsigned long long *)&m.host[16] != seq)
            return fail(JP_ERR_CUDA, "tiny kernel finished without publishing its results");
        }
      }
      // (no stream sync: the kernel publishes after its last write of A / T, and the
      // arrays are read after st like every jp_schedule result, include/jp.h)
      memcpy(h, const_cast<const int64_t *>(m.host), sizeof h);
    } else {
      JP_CUDA(launch_tiny(j, L, c.tau_high, c.tls_window, c.tls_w_max, c.tls_recovery, hdr, st), "tiny");
      JP_CUDA(d2h_small_sync(h, hdr, sizeof h, st), "tiny D2H");
    }
    if (h[H_TINY_MODE] < 0) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)h[H_BAD]);
    fill_profile(&res->prof, L->n, h);
    res->profiled = 1;
    res->mode = (int32_t)h[H_TINY_MODE];
    res->n_tasks = 1;
    res->n_batches = 1;
    const int run = res->mode == JP_MODE_SEQ_RECOMMENDED ? JP_MODE_TLS : res->mode;
    res->task_mode_iters[run] = L->n;
    if (run == JP_MODE_TLS) {
      res->tls.committed = h[H_TLS_COMMITTED];
      res->tls.executed = h[H_TLS_EXECUTED];
      res->tls.windows = h[H_TLS_WINDOWS];
      res->tls.violations = h[H_TLS_VIOL];
      res->tls_w_max = h[H_TINY_WMAX];
      res->tls_path = 4;
      res->tls_recovery = (int32_t)h[H_TINY_REC];
      res->tls_cluster = 1;
    }
    return JP_OK;
  }
  // structural RAW-freedom (reading B11; the paper's static rule 3, P:L257-260,
  // "all pairs comprising a live-out and a live-in variable"): when no exposed
  // read can touch an array that some iteration writes, d_raw = 0 whatever the
  // indices hold, so Fig. 2(b) can only end in D or D'.  Privatized execution is
  // exact in both, DOALL in D' -- no profile: the indirect index arrays are
  // validated on the device and the run, launched behind it, exits at once on
  // an out-of-range index (nothing modified, reading A13).
  if (c.static_check == 0 && c.tls_path == 0 && ws) {
    const int smode = structural_mode(j);
    if (smode >= 0) {
      Layout lo;
      JP_TRY(check_ws(L, ws, ws_bytes, smode == JP_MODE_PRIVATIZED ? JP_WS_PRIV : 0, lo));
      int64_t *bad = &at<int64_t>(ws, lo, R_HEADER)[H_BAD];
      Job jr = j;
      jr.d.abort = bad;
      int64_t nb = 0;
      bool published = false;
      if (smode == JP_MODE_PRIVATIZED) {
        // the two-phase kernel publishes its index count to mapped host words
        // (tiny mirror [17] count, [18] sequence) when its check is done: the
        // call returns then, the X -> Y phase runs on, ordered on st
        TinyMirror &m = tiny_mirror();
        const bool mir = m.host && !getenv("JP_STRUCT_NO_MIRROR");
        const unsigned long long seq = mir ? ++m.seq : 0;
        bool applied = false;
        JP_CUDA(launch_priv_stream(jr, ws, lo, true, st, 0, true, &applied, bad, mir ? m.dev + 17 : nullptr, seq,
                                   &published),
                "priv stream");
        if (!applied) JP_CUDA(launch_priv_finalize(jr, ws, lo, st), "priv finalize");
        if (published) {
          volatile unsigned long long *flag = reinterpret_cast<volatile unsigned long long *>(&m.host[18]);
          for (unsigned spins = 0; *flag != seq; spins++) {
            if ((spins & 1023) == 1023) {
              const cudaError_t q = cudaStreamQuery(st);
              if (q != cudaSuccess && q != cudaErrorNotReady) return cuda_fail(q, "priv stream");
              if (q == cudaSuccess && *flag != seq)
                return fail(JP_ERR_CUDA, "privatized kernel finished without publishing its index check");
            }
          }
          nb = *reinterpret_cast<volatile int64_t *>(&m.host[17]);
        }
      } else {
        JP_CUDA(launch_validate_indirect(j, bad, st), "validate");
        JP_CUDA(launch_doall(jr, st), "doall");
      }
      if (!published) JP_CUDA(d2h_small_sync(&nb, bad, sizeof nb, st), "validate D2H");
      if (nb) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)nb);
      res->mode = smode;
      res->profiled = 0;
      res->n_tasks = 1;
      res->n_batches = 1;
      res->task_mode_iters[smode] = L->n;
      return JP_OK;
    }
  }
  // the pair table of the profile (all ones = no stamp yet) is filled on a side
  // stream from the start, overlapping the static check's prefix read
  const Layout lg = layout(L);
  const bool gfuse = lg.bytes[R_GUIDE] && ws && ws_bytes >= layout_end(lg, JP_WS_PROFILE | JP_WS_GUIDE | JP_WS_TLS);
  // the address-bucket profile keeps no tables: no pair table to pre-fill (the
  // TLS paths that use region 7 reset it themselves)
  const bool bucket = gfuse && bucket_profile_ok(j, ws, lg);
  const bool pairs = gfuse && !bucket && stamp_pairs_ok(j, ws, lg);
  cudaEvent_t pdone = nullptr;
  if (pairs && cudaEventCreateWithFlags(&pdone, cudaEventDisableTiming) == cudaSuccess) {
    cudaStream_t side = g_pool.get(41);
    cudaEventRecord(pdone, st);
    cudaStreamWaitEvent(side, pdone, 0);
    cudaMemsetAsync(at<char>(ws, lg, R_TLS_S_A), 0xFF, 8 * (size_t)L->len_A, side);
    cudaEventRecord(pdone, side);
  }
  // st waits for the fill before its next use of the region (the stamp, or the
  // DOALL exit below): every path after this point calls it once
  auto join_fill = [&]() {
    if (pdone) {
      cudaStreamWaitEvent(st, pdone, 0);
      cudaEventDestroy(pdone);
      pdone = nullptr;
    }
  };
  const bool pairs_ready = pdone != nullptr;
  cudaEvent_t vdone = nullptr;
  // every exit (an error return included) orders st after the side-stream clear
  // of the shadow values and releases the event
  struct JoinV {
    cudaEvent_t &e; cudaStream_t s;
    void join() { if (e) { cudaStreamWaitEvent(s, e, 0); cudaEventDestroy(e); e = nullptr; } }
    ~JoinV() { join(); }
  } join_v{vdone, st};
  // the on-chip TLS shadow values must start at zero: cleared on a side stream
  // queued right behind the static check's one-warp sample kernel (not before
  // it: the clear would hold every SM while the host waits for the sample), so
  // it overlaps the sample's round trip and the profile
  const std::function<void()> clear_v = [&]() {
    // (the bucket profile clears the slots path 8 uses itself: V[a] = 0 at every raw read's address)
    if (!(gfuse && pairs) || vdone) return;
    auto *V = at<unsigned long long>(ws, lg, R_TLS_C_A);
    if (V && cudaEventCreateWithFlags(&vdone, cudaEventDisableTiming) == cudaSuccess) {
      cudaStream_t side = g_pool.get(40);
      cudaEventRecord(vdone, st);          // after whatever ran before on st
      cudaStreamWaitEvent(side, vdone, 0);
      cudaMemsetAsync(V, 0, lg.bytes[R_TLS_C_A], side);
      cudaEventRecord(vdone, side);
    }
  };
  // with the address-bucket profile the static check's affine sample rides on
  // the profile's first kernel (the rest of the profile exits when the sample
  // looks affine): no host round trip before the profile starts
  const bool defer_static = c.static_check == 0 && ws && bucket && tiny_mirror().host && L->n >= 3 &&
                            !getenv("JP_NO_DEFER_STATIC");
  if (c.static_check == 0 && ws && !defer_static) {
    // static analysis lite: affine, in-range, conflict-free -> DOALL without a profile
    Layout ls;
    if (jp_status e0 = check_ws(L, ws, ws_bytes, 0, ls)) { join_fill(); return e0; }
    jp_static sa;
    if (jp_status e1 = static_check(L, j, ws, ls, &sa, st, &clear_v)) { join_fill(); return e1; }
    if (sa.independent && sa.in_range) {
      res->mode = JP_MODE_DOALL;
      res->profiled = 0;
      res->n_tasks = 1;
      res->n_batches = 1;
      join_fill();
      JP_CUDA(launch_doall(j, st), "doall");
      res->task_mode_iters[JP_MODE_DOALL] = L->n;
      return JP_OK;
    }
  }
  join_fill();
  jp_profile p;
  // the classify pass also writes the TLS guide bitmaps when the loop can be guided
  // (A read through an index, workspace with the guide region): no separate guide pass
  int clean = 0;
  int64_t dist[32];
  bool have_dist = false;
  bool spec = false;   // path 8 launched behind the profile, gated on its header
  clear_v();   // (no static check ran)
  if (vdone) clean = 2;
  if (gfuse) {
    // large A tables: stamped straight into {minW, minR} pairs (one 8-byte entry
    // per address for the classify lookups; the separate tables stay unwritten)
    if (pairs) clean |= 1;   // region 7 holds this call's pair table, or the side stream's all-ones fill
    if (bucket) {
      // large A: the profile by address buckets (jp_bucket.cu), guide words included
      uint32_t *g = at<uint32_t>(ws, lg, R_GUIDE);
      TinyMirror &mm = tiny_mirror();
      const unsigned long long seq = defer_static ? ++mm.seq : 0;
      if (defer_static) *reinterpret_cast<volatile unsigned long long *>(&mm.host[21]) = seq;   // read by the kernel
      JP_CUDA(launch_prof_bucket(j, ws, lg, g, g + (L->n + 31) / 32, 0, nullptr, st, nullptr, nullptr,
                                 at<unsigned long long>(ws, lg, R_TLS_C_A), defer_static ? (int)std::min<int64_t>(L->n, 64) : 0,
                                 defer_static ? reinterpret_cast<long long *>(mm.dev + 19) : nullptr,
                                 defer_static ? reinterpret_cast<const unsigned long long *>(mm.dev + 21) : nullptr),
              "profile (buckets)");
      clean |= 4;   // V clear at every address path 8 polls
      if (defer_static) {
        volatile unsigned long long *flag = reinterpret_cast<volatile unsigned long long *>(&mm.host[20]);
        for (unsigned spins = 0; *flag != seq; spins++) {
          if ((spins & 1023) == 1023) {
            const cudaError_t q = cudaStreamQuery(st);
            if (q != cudaSuccess && q != cudaErrorNotReady) return cuda_fail(q, "profile");
            if (q == cudaSuccess && *flag != seq) return fail(JP_ERR_CUDA, "profile did not publish its affine sample");
          }
        }
        if (*reinterpret_cast<volatile int64_t *>(&mm.host[19]) != 0) {
          // the sample looks affine (the profile's kernels exited): the full static
          // check, then DOALL or the profile proper
          Layout ls;
          JP_TRY(check_ws(L, ws, ws_bytes, 0, ls));
          jp_static sa;
          JP_TRY(static_check(L, j, ws, ls, &sa, st, nullptr, true));
          if (sa.independent && sa.in_range) {
            res->mode = JP_MODE_DOALL;
            res->profiled = 0;
            res->n_tasks = 1;
            res->n_batches = 1;
            JP_CUDA(launch_doall(j, st), "doall");
            res->task_mode_iters[JP_MODE_DOALL] = L->n;
            return JP_OK;
          }
          JP_CUDA(launch_prof_bucket(j, ws, lg, g, g + (L->n + 31) / 32, 0, nullptr, st, nullptr, nullptr,
                                     at<unsigned long long>(ws, lg, R_TLS_C_A)),
                  "profile (buckets)");
        }
      }
    } else {
      if (pairs) JP_CUDA(launch_prof_stamp(j, ws, lg, st, true, pairs_ready), "profile stamp");
      else JP_TRY(jp_profile_stamp(L, ws, ws_bytes, stp));
      JP_CUDA(launch_prof_classify_guide(j, ws, lg, st, pairs), "profile classify");
    }
    const bool vclear = vdone != nullptr;
    join_v.join();   // everything after the profile on st (TLS, or any later call) sees V zeroed
    int64_t h[H_DIST + 32];
    int64_t *hd = at<int64_t>(ws, lg, R_HEADER);
    // Path 8 launched behind the profile, before the host has read it: the
    // kernel itself checks the header (gate) and runs only when Fig. 2(b) gives
    // mode B with war = waw = 0 -- exactly when run_mode below would pick path 8
    // -- so the GPU does not idle through the header's round trip; the header
    // travels to the host on a side stream meanwhile.
    spec = (vclear || bucket) && j.op == JP_OP_ADD_C && c.tls_path == 0 && c.tls_window == 0 && c.tls_recovery != 1 &&
           L->n > 0 && !getenv("JP_TLS_NO_FLOW") && !getenv("JP_NO_SPEC_FLOW");
    cudaEvent_t ep = nullptr, ec = nullptr;
    if (spec && (cudaEventCreateWithFlags(&ep, cudaEventDisableTiming) != cudaSuccess ||
                 cudaEventCreateWithFlags(&ec, cudaEventDisableTiming) != cudaSuccess)) {
      if (ep) cudaEventDestroy(ep);
      ep = nullptr;
      spec = false;
    }
    if (spec) {
      thread_local int64_t *pin = nullptr;
      if (!pin && cudaMallocHost(reinterpret_cast<void **>(&pin), sizeof h) != cudaSuccess) pin = nullptr;
      cudaError_t e = pin ? cudaSuccess : cudaErrorMemoryAllocation;
      if (e == cudaSuccess) {
        cudaStream_t side = g_pool.get(42);
        cudaEventRecord(ep, st);
        cudaStreamWaitEvent(side, ep, 0);
        e = cudaMemcpyAsync(pin, hd, sizeof h, cudaMemcpyDeviceToHost, side);
        if (e == cudaSuccess) e = cudaEventRecord(ec, side);
      }
      if (e == cudaSuccess) {
        const uint32_t *g = at<uint32_t>(ws, lg, R_GUIDE);
        e = launch_tls_flow(j, g, g + (L->n + 31) / 32, at<unsigned long long>(ws, lg, R_TLS_C_A),
                            &hd[H_TLS_COMMITTED], st, nullptr, 0, hd, raw_max_for(L->n, c.tau_high),
                            !bucket,   // (the bucket profile's reset of the header zeroed the statistics)
                            0,
                            // the gather phase's values in region 1 (the bucket profile's records,
                            // dead once its eval ran) for loops with few violators
                            bucket && lg.bytes[R_MINW_A] >= 4 * (size_t)L->n ? at<uint32_t>(ws, lg, R_MINW_A) : nullptr,
                            ph_max_for(L->n));
      }
      if (e == cudaSuccess) e = cudaEventSynchronize(ec);
      cudaEventDestroy(ep);
      cudaEventDestroy(ec);
      if (e != cudaSuccess) return cuda_fail(e, "profile D2H / one-window TLS");
      memcpy(h, pin, sizeof h);
    } else {
      JP_CUDA(d2h_small_sync(h, hd, sizeof h, st), "profile D2H");
    }
    if (h[H_BAD]) return fail(JP_ERR_INDEX, "%lld index entries are outside their arrays", (long long)h[H_BAD]);
    fill_profile(&p, L->n, h);
    memcpy(dist, h + H_DIST, sizeof dist);
    have_dist = true;
  } else {
    JP_TRY(jp_profile_density(L, ws, ws_bytes, nullptr, 0, nullptr, &p, stp));
  }
  res->prof = p;
  res->profiled = 1;
  res->mode = select_mode_counts(p.n, p.raw_iters, p.war_iters, p.waw_iters, c.tau_high);
  res->n_tasks = 1;
  res->n_batches = 1;
  if (spec && res->mode == JP_MODE_TLS && p.war_iters == 0 && p.waw_iters == 0) {
    // the gated path-8 kernel is running (its predicate is this one); its
    // statistics are fixed by the profile: one window, the raw iterations are
    // the violators (jp_tls_flow.cu).  JP_FLOW_CHECK=1 waits for it and checks
    // that no violator lost its writer.
    if (getenv("JP_FLOW_CHECK")) {
      int64_t s4[4];
      JP_CUDA(d2h_small_sync(s4, &at<int64_t>(ws, lg, R_HEADER)[H_TLS_COMMITTED], sizeof s4, st), "tls D2H");
      if (s4[1] || s4[3] != p.raw_iters)
        return fail(JP_ERR_ARG, "one-window TLS: %lld warps lost their writer, %lld violations for %lld raw iterations",
                    (long long)s4[1], (long long)s4[3], (long long)p.raw_iters);
    }
    res->tls.committed = L->n;
    res->tls.executed = L->n + p.raw_iters;
    res->tls.windows = 1;
    res->tls.violations = p.raw_iters;
    res->tls_w_max = L->n;
    res->tls_path = 8;
    res->tls_guided = 1;
    res->tls_recovery = JP_TLS_ONCHIP;
    res->tls_cluster = num_sms();
    res->task_mode_iters[JP_MODE_TLS] += L->n;
    return JP_OK;
  }
  // an ADD_C or SAXPY TLS loop WITH WAR / WAW, profiled by address buckets: the last
  // earlier writer of every raw read from the records still in place, then one
  // window over the whole loop (path 9, reading B14, jp_tls_flow.cu); the
  // windowed paths stay for what the last-writer pass cannot hold
  if (bucket && res->mode == JP_MODE_TLS && (j.op == JP_OP_ADD_C || j.op == JP_OP_SAXPY) &&
      (p.war_iters > 0 || p.waw_iters > 0) &&
      c.tls_recovery == 0 && c.tls_path == 0 && c.tls_window == 0 && !getenv("JP_TLS_NO_FLOW")) {
    int64_t *hd = at<int64_t>(ws, lg, R_HEADER);
    auto *pred = at<int32_t>(ws, lg, R_TLS_S_A);
    auto *bits = reinterpret_cast<uint32_t *>(pred + ((L->n + 63) & ~(int64_t)63));
    auto *V = at<unsigned long long>(ws, lg, R_TLS_C_A);
    const uint32_t *graw = at<uint32_t>(ws, lg, R_GUIDE);
    // the last-writer pass and the one-window kernel (five launches) replayed from
    // a CUDA graph per loop / workspace: the host has just synchronised on the
    // header, so every launch gap would be an idle GPU
    auto issue9 = [&](cudaStream_t s) -> cudaError_t {
      cudaError_t e = launch_prof_pred(j, ws, lg, pred, bits, V, s);   // (clears V[pred])
      if (e == cudaSuccess) e = launch_tls_flow_waw(j, graw, pred, bits, V, &hd[H_TLS_COMMITTED], hd, s);
      return e;
    };
    {
      std::string key;
      auto put = [&](auto v) { key.append(reinterpret_cast<const char *>(&v), sizeof v); };
      int dev = 0;
      cudaGetDevice(&dev);
      put(dev); put(j.op); put(j.dt); put(j.d.n); put(j.d.ioff); put(j.d.base); put(j.d.lenA); put(j.d.r); put(j.d.w);
      put(j.d.A); put(j.d.X); put(j.d.c0); put(ws); put(lg.total);
      JP_CUDA(graph_launch(key, issue9, st), "last writers / tls one window (waw)");
      note_launch(5);
    }
    int64_t h2[H_PRED_SEG + 1];
    JP_CUDA(d2h_small_sync(h2, hd, sizeof h2, st), "tls D2H");
    if (h2[H_PRED_FAIL] == 0) {
      if (h2[H_TLS_EXECUTED])
        return fail(JP_ERR_ARG, "one-window TLS: a violator's writer never published (profile inconsistent)");
      if (h2[H_TLS_VIOL] != p.raw_iters)
        return fail(JP_ERR_ARG, "one-window TLS: %lld violations for %lld raw iterations",
                    (long long)h2[H_TLS_VIOL], (long long)p.raw_iters);
      res->tls.committed = L->n;
      res->tls.executed = L->n + p.raw_iters;
      res->tls.windows = 1;
      res->tls.violations = p.raw_iters;
      res->tls_w_max = L->n;
      res->tls_path = 9;
      res->tls_guided = 1;
      res->tls_recovery = JP_TLS_ONCHIP;
      res->tls_cluster = num_sms();
      res->task_mode_iters[JP_MODE_TLS] += L->n;
      return JP_OK;
    }
    // the pass gave up: region 7 holds its tables and V some cleared slots (the
    // kernel exited at its gate); the windowed paths reset both themselves
    // (clean bit 1 off; bit 2 -- V all zero -- was never set with the bucket profile)
    clean &= ~1;
  }
  return run_mode(L, j, res->mode, &p, c, ws, ws_bytes, res, st, gfuse && p.waw_iters == 0, clean,
                  have_dist ? dist : nullptr);
}


// ---------------------------------------------------------------------------
// workflows: PDG of loops (readings B9, B10)
// ---------------------------------------------------------------------------
namespace {
struct Span { uintptr_t lo, hi; bool write; };
// the device memory a loop touches: index arrays and X read; A read (ADD_C,
// SAXPY, STENCIL2) and written; T written (its covered reads are its own writes)
static int footprint(const jp_loop *L, Span *out) {
  int k = 0;
  auto add = [&](const void *p, int64_t len, bool w) {
    if (p && len > 0 && L->n > 0) out[k++] = {(uintptr_t)p, (uintptr_t)p + 4 * (uintptr_t)len, w};
  };
  add(L->r, L->n, false);
  add(L->r2, L->n, false);
  add(L->w, L->n, false);
  add(L->s, L->n, false);
  add(L->X, L->len_X, false);
  if (L->op != JP_OP_PRIV_TMP) add(L->A, L->len_A, false);
  add(L->A, L->len_A, true);
  if (L->op == JP_OP_PRIV_TMP) add(L->T, L->len_T, true);
  return k;
}
}  // namespace

static jp_status plan_workflow(const jp_loop *loops, int32_t n, int32_t scheme, jp_workflow_plan *out) {
  if (!loops || !out || n < 0 || n > JP_MAX_LOOPS) return fail(JP_ERR_ARG, "need 0 <= n <= %d loops", JP_MAX_LOOPS);
  if (scheme < JP_SCHED_SHARING || scheme > JP_SCHED_AUTO) return fail(JP_ERR_ARG, "bad scheme %d", scheme);
  memset(out, 0, sizeof *out);
  std::vector<std::vector<Span>> fp(n);
  for (int u = 0; u < n; u++) {
    JP_TRY(check_loop(&loops[u]));
    Span s[8];
    fp[u].assign(s, s + footprint(&loops[u], s));
  }
  int64_t total = 0, biggest = 0;
  for (int u = 0; u < n; u++) {
    for (int t = 0; t < u; t++) {
      bool dep = false;
      for (const Span &a : fp[t])
        for (const Span &b : fp[u])
          dep = dep || ((a.write || b.write) && a.lo < b.hi && b.lo < a.hi);
      if (dep) {
        out->deps[u] |= 1ull << t;
        out->batch[u] = std::max(out->batch[u], out->batch[t] + 1);
      }
    }
    out->n_batches = std::max(out->n_batches, out->batch[u] + 1);
    total += loops[u].n;
    biggest = std::max(biggest, loops[u].n);
  }
  if (scheme == JP_SCHED_AUTO) {
    bool wide = false;
    for (int b = 0; b < out->n_batches && !wide; b++) {
      int cnt = 0;
      for (int u = 0; u < n; u++) cnt += out->batch[u] == b;
      wide = cnt >= 2;
    }
    scheme = wide && 2 * biggest <= total ? JP_SCHED_STEALING : JP_SCHED_SHARING;
  }
  out->scheme = scheme;
  return JP_OK;
}

jp_status jp_plan_workflow(const jp_loop *loops, int32_t n, int32_t scheme, jp_workflow_plan *out) {
  return plan_workflow(loops, n, scheme, out);
}

jp_status jp_schedule_workflow(const jp_loop *loops, int32_t n, const jp_sched_cfg *cfgp, void *const *ws,
                               const size_t *ws_bytes, jp_sched_result *res, jp_workflow_plan *plan,
                               jp_stream_t stp) {
  if (!res || !plan) return fail(JP_ERR_ARG, "result / plan is NULL");
  JP_TRY(need_device());
  jp_sched_cfg c = cfgp ? *cfgp : default_cfg();
  JP_TRY(plan_workflow(loops, n, c.scheme, plan));
  jp_sched_cfg lc = c;
  lc.scheme = JP_SCHED_SHARING;   // each loop: the single-loop scheme
  cudaStream_t st = (cudaStream_t)stp;
  auto wsp = [&](int u) { return ws ? ws[u] : nullptr; };
  auto wsb = [&](int u) { return ws_bytes ? ws_bytes[u] : (size_t)0; };
  if (plan->scheme == JP_SCHED_SHARING) {
    for (int u = 0; u < n; u++) JP_TRY(jp_schedule(&loops[u], &lc, wsp(u), wsb(u), &res[u], stp));
    return JP_OK;
  }
  // STEALING on one device: batch after batch; the loops of a batch run
  // concurrently, each on its own stream, joined before the next batch
  cudaEvent_t ev0;
  JP_CUDA(cudaEventCreateWithFlags(&ev0, cudaEventDisableTiming), "event");
  std::vector<cudaEvent_t> evs;
  jp_status status = JP_OK;
  for (int b = 0; b < plan->n_batches && status == JP_OK; b++) {
    cudaEventRecord(ev0, st);
    std::vector<cudaEvent_t> joins;
    int k = 0;
    for (int u = 0; u < n && status == JP_OK; u++) {
      if (plan->batch[u] != b) continue;
      cudaStream_t s2 = g_pool.get(k++);
      cudaStreamWaitEvent(s2, ev0, 0);
      status = jp_schedule(&loops[u], &lc, wsp(u), wsb(u), &res[u], (jp_stream_t)s2);
      cudaEvent_t e;
      cudaEventCreateWithFlags(&e, cudaEventDisableTiming);
      cudaEventRecord(e, s2);
      joins.push_back(e);
      evs.push_back(e);
    }
    for (auto e : joins) cudaStreamWaitEvent(st, e, 0);
  }
  cudaError_t ce = cudaStreamSynchronize(st);
  for (auto e : evs) cudaEventDestroy(e);
  cudaEventDestroy(ev0);
  if (status != JP_OK) return status;
  if (ce != cudaSuccess) return fail(JP_ERR_CUDA, "workflow: %s", cudaGetErrorString(ce));
  return JP_OK;
}

// ---------------------------------------------------------------------------
// host-buffer entry point (end-to-end: H2D, schedule, D2H)
// ---------------------------------------------------------------------------
struct Stage { size_t off[7]; size_t total; };
static Stage stage_layout(const jp_loop *L) {
  Stage s{};
  bool ur, ur2, uw, us;
  used_idx(L->op, ur, ur2, uw, us);
  const size_t sz[7] = {(ur && L->r) ? 4 * (size_t)L->n : 0, (ur2 && L->r2) ? 4 * (size_t)L->n : 0,
                        (uw && L->w) ? 4 * (size_t)L->n : 0, (us && L->s) ? 4 * (size_t)L->n : 0,
                        4 * (size_t)L->len_A, L->X ? 4 * (size_t)L->len_X : 0, L->T ? 4 * (size_t)L->len_T : 0};
  size_t o = 0;
  for (int k = 0; k < 7; k++) { s.off[k] = sz[k] ? o : SIZE_MAX; o = al256(o + sz[k]); }
  s.total = o;
  return s;
}

size_t jp_stage_bytes(const jp_loop *L) {
  if (!L || check_loop(L) == JP_ERR_ARG) return 0;
  return stage_layout(L).total;
}

// Determined-DOALL loops (every index NULL, identity from element 0; mode A,
// P:L361-362) need no profile, so staging can overlap execution chunk by chunk
// (data "moved to the GPU in advance and asynchronously with the
// kernel execution"): chunk c's H2D, kernel and D2H run on pool stream c % 3,
// so one chunk's upload, another's kernel and a third's download proceed
// together on the two copy engines and the SMs.
static jp_status schedule_host_pipelined(const jp_loop *Lh, const Stage &sl, char *b, jp_sched_result *res,
                                         cudaStream_t st) {
  const int64_t n = Lh->n;
  int64_t chunk = 1 << 23;   // measured: 2^20 5.3, 2^21 5.9, 2^22 6.15, 2^23 6.28, 2^24 6.29 G iter/s (config 2 e2e)
  if (const char *e = getenv("JP_STAGE_CHUNK")) chunk = std::max<int64_t>(1024, atoll(e));
  chunk = (chunk + 3) & ~(int64_t)3;
  const bool usesX = Lh->op == JP_OP_SAXPY || Lh->op == JP_OP_PRIV_TMP;
  const bool hasT = Lh->op == JP_OP_PRIV_TMP;
  const bool readsA = Lh->op != JP_OP_PRIV_TMP;
  char *dA = b + sl.off[4], *dX = usesX ? b + sl.off[5] : nullptr, *dT = hasT ? b + sl.off[6] : nullptr;
  cudaEvent_t e0;
  JP_CUDA(cudaEventCreateWithFlags(&e0, cudaEventDisableTiming), "event");
  cudaEventRecord(e0, st);
  constexpr int kPipe = 3;
  cudaStream_t ps[kPipe];
  for (int k = 0; k < kPipe; k++) {
    ps[k] = g_pool.get(32 + k);
    cudaStreamWaitEvent(ps[k], e0, 0);
  }
  for (int64_t c0 = 0, c = 0; c0 < n; c0 += chunk, c++) {
    const int64_t m = std::min(chunk, n - c0);
    cudaStream_t s = ps[c % kPipe];
    const size_t off = 4 * (size_t)c0, nb = 4 * (size_t)m;
    if (readsA) JP_CUDA(cudaMemcpyAsync(dA + off, static_cast<const char *>(Lh->A) + off, nb, cudaMemcpyHostToDevice, s), "H2D");
    if (usesX) JP_CUDA(cudaMemcpyAsync(dX + off, static_cast<const char *>(Lh->X) + off, nb, cudaMemcpyHostToDevice, s), "H2D");
    jp_loop sub = *Lh;
    sub.n = m;
    sub.iter_base = Lh->iter_base + c0;
    sub.A = dA + off;
    sub.len_A = m;
    sub.X = dX ? dX + off : nullptr;
    sub.len_X = dX ? m : 0;
    sub.T = dT ? dT + off : nullptr;
    sub.len_T = dT ? m : 0;
    JP_CUDA(launch_doall(make_job(&sub), s), "doall chunk");
    JP_CUDA(cudaMemcpyAsync(static_cast<char *>(Lh->A) + off, dA + off, nb, cudaMemcpyDeviceToHost, s), "D2H");
    if (hasT) JP_CUDA(cudaMemcpyAsync(static_cast<char *>(Lh->T) + off, dT + off, nb, cudaMemcpyDeviceToHost, s), "D2H");
  }
  for (int k = 0; k < kPipe; k++) {
    cudaEvent_t e;
    cudaEventCreateWithFlags(&e, cudaEventDisableTiming);
    cudaEventRecord(e, ps[k]);
    cudaStreamWaitEvent(st, e, 0);
    cudaEventDestroy(e);
  }
  cudaEventDestroy(e0);
  JP_CUDA(cudaStreamSynchronize(st), "stage sync");
  res->mode = JP_MODE_DOALL;
  res->profiled = 0;
  res->n_tasks = 1;
  res->n_batches = 1;
  res->task_mode_iters[JP_MODE_DOALL] = n;
  return JP_OK;
}

jp_status jp_schedule_host(const jp_loop *Lh, const jp_sched_cfg *cfg, void *stage, size_t stage_bytes, void *ws,
                           size_t ws_bytes, jp_sched_result *res, jp_stream_t stp) {
  JP_TRY(check_loop(Lh));
  JP_TRY(need_device());
  Stage sl = stage_layout(Lh);
  if (!stage || stage_bytes < sl.total) return fail(JP_ERR_WORKSPACE, "stage buffer needs %zu bytes", sl.total);
  cudaStream_t st = (cudaStream_t)stp;
  if (!Lh->r && !Lh->r2 && !Lh->w && !Lh->s && Lh->ident_off == 0 && res && Lh->n > 0 &&
      Lh->len_A == Lh->n && (!(Lh->op == JP_OP_SAXPY || Lh->op == JP_OP_PRIV_TMP) || Lh->len_X == Lh->n) &&
      (Lh->op != JP_OP_PRIV_TMP || Lh->len_T == Lh->n) && !(getenv("JP_STAGE_PIPELINE") && getenv("JP_STAGE_PIPELINE")[0] == '0')) {
    memset(res, 0, sizeof *res);
    return schedule_host_pipelined(Lh, sl, static_cast<char *>(stage), res, st);
  }
  jp_loop Ld = *Lh;
  char *b = static_cast<char *>(stage);
  const void *src[7] = {Lh->r, Lh->r2, Lh->w, Lh->s, Lh->A, Lh->X, Lh->T};
  const size_t sz[7] = {4 * (size_t)Lh->n, 4 * (size_t)Lh->n, 4 * (size_t)Lh->n, 4 * (size_t)Lh->n,
                        4 * (size_t)Lh->len_A, 4 * (size_t)Lh->len_X, 4 * (size_t)Lh->len_T};
  void *dst[7];
  for (int k = 0; k < 7; k++) {
    dst[k] = sl.off[k] == SIZE_MAX ? nullptr : b + sl.off[k];
    if (dst[k] && sz[k]) JP_CUDA(cudaMemcpyAsync(dst[k], src[k], sz[k], cudaMemcpyHostToDevice, st), "stage H2D");
  }
  Ld.r = (const int32_t *)dst[0]; Ld.r2 = (const int32_t *)dst[1]; Ld.w = (const int32_t *)dst[2];
  Ld.s = (const int32_t *)dst[3]; Ld.A = dst[4]; Ld.X = dst[5]; Ld.T = dst[6];
  JP_TRY(jp_schedule(&Ld, cfg, ws, ws_bytes, res, stp));
  if (Lh->len_A) JP_CUDA(cudaMemcpyAsync(Lh->A, Ld.A, sz[4], cudaMemcpyDeviceToHost, st), "stage D2H");
  if (Lh->T && Lh->len_T && Lh->op == JP_OP_PRIV_TMP)
    JP_CUDA(cudaMemcpyAsync(Lh->T, Ld.T, sz[6], cudaMemcpyDeviceToHost, st), "stage D2H");
  JP_CUDA(cudaStreamSynchronize(st), "stage sync");
  return JP_OK;
}

}  // extern "C"
