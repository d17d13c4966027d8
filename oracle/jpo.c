/*
 * oracle/jpo.c -- TEST INFRASTRUCTURE ONLY (see jpo.h).  Plain sequential C.
 *
 * Every function below restates a definition from the paper or from the
 * readings listed in DESIGN.md Sec.3 (the paper defers the density model to
 * its ref [4], and the GPU-TLS internals to ref [3],
 * P:L79-81; neither is in /root/reference).  No blocking, fusion
 * or reordering beyond what the definition states.
 *
 * Build: gcc -O2 -ffp-contract=off -fno-fast-math -fPIC -shared
 */
#include "jpo.h"
#include <stdlib.h>
#include <string.h>

/* ---------------------------------------------------------------------------
 * Access sets of one iteration (SURVEY Sec.8 opcode table).
 *   R_exp(i): exposed reads  -- read before any write of the same iteration
 *   R_cov(i): covered reads  -- read after the same iteration wrote it
 *   W(i)    : writes
 * ------------------------------------------------------------------------- */
typedef struct { int arr; int64_t a; } acc_t;
typedef struct { acc_t rexp[2]; int nrexp; acc_t rcov[1]; int nrcov; acc_t wr[2]; int nwr; } accs_t;

static int64_t ix(const int32_t *p, int64_t i) { return p ? (int64_t)p[i] : i; }

static int op_valid(const jpo_loop *L) {
  if (!L || L->n < 0) return 0;
  if (L->op < JPO_OP_ADD_C || L->op > JPO_OP_STENCIL2) return 0;
  if (L->dtype != JPO_I32 && L->dtype != JPO_F32) return 0;
  if (L->n > 0 && !L->A) return 0;
  if ((L->op == JPO_OP_SAXPY || L->op == JPO_OP_PRIV_TMP) && L->n > 0 && !L->X) return 0;
  if (L->op == JPO_OP_PRIV_TMP && L->n > 0 && !L->T) return 0;
  return 1;
}

static void accesses(const jpo_loop *L, int64_t i, accs_t *s) {
  s->nrexp = s->nrcov = s->nwr = 0;
  switch (L->op) {
  case JPO_OP_ADD_C:      /* A[w] = A[r] + c0 */
    s->rexp[s->nrexp++] = (acc_t){JPO_ARR_A, ix(L->r, i)};
    s->wr[s->nwr++] = (acc_t){JPO_ARR_A, ix(L->w, i)};
    break;
  case JPO_OP_SAXPY:      /* Y[w] = c0*X[r] + Y[w] */
    s->rexp[s->nrexp++] = (acc_t){JPO_ARR_X, ix(L->r, i)};
    s->rexp[s->nrexp++] = (acc_t){JPO_ARR_A, ix(L->w, i)};
    s->wr[s->nwr++] = (acc_t){JPO_ARR_A, ix(L->w, i)};
    break;
  case JPO_OP_PRIV_TMP:   /* T[s] = c0*X[r]; Y[w] = T[s] + c1 */
    s->rexp[s->nrexp++] = (acc_t){JPO_ARR_X, ix(L->r, i)};
    s->rcov[s->nrcov++] = (acc_t){JPO_ARR_T, ix(L->s, i)};
    s->wr[s->nwr++] = (acc_t){JPO_ARR_T, ix(L->s, i)};
    s->wr[s->nwr++] = (acc_t){JPO_ARR_A, ix(L->w, i)};
    break;
  case JPO_OP_STENCIL2:   /* A[w] = (A[r] + A[r2]) * c0 */
    s->rexp[s->nrexp++] = (acc_t){JPO_ARR_A, ix(L->r, i)};
    s->rexp[s->nrexp++] = (acc_t){JPO_ARR_A, ix(L->r2, i)};
    s->wr[s->nwr++] = (acc_t){JPO_ARR_A, ix(L->w, i)};
    break;
  }
}

static int64_t arr_len(const jpo_loop *L, int arr) {
  return arr == JPO_ARR_A ? L->len_A : arr == JPO_ARR_X ? L->len_X : L->len_T;
}

/* Reading A13: any index outside its array => JPO_ERR_INDEX, nothing modified. */
static int check_indices(const jpo_loop *L) {
  for (int64_t i = 0; i < L->n; i++) {
    accs_t s; accesses(L, i, &s);
    for (int k = 0; k < s.nrexp; k++) if (s.rexp[k].a < 0 || s.rexp[k].a >= arr_len(L, s.rexp[k].arr)) return JPO_ERR_INDEX;
    for (int k = 0; k < s.nrcov; k++) if (s.rcov[k].a < 0 || s.rcov[k].a >= arr_len(L, s.rcov[k].arr)) return JPO_ERR_INDEX;
    for (int k = 0; k < s.nwr; k++)   if (s.wr[k].a < 0 || s.wr[k].a >= arr_len(L, s.wr[k].arr)) return JPO_ERR_INDEX;
  }
  return JPO_OK;
}

static float f32(uint32_t b) { float f; memcpy(&f, &b, 4); return f; }

/* ---------------------------------------------------------------------------
 * The loop body, executed for one iteration i reading `src` arrays and
 * writing `dst` arrays.  In sequential execution src == dst.  In privatized
 * execution (reading A10) exposed reads come from the pre-loop snapshot while
 * the covered read of T is the iteration's own private copy.
 * ------------------------------------------------------------------------- */
static void body(const jpo_loop *L, int64_t i,
                 const void *srcA, const void *srcX, void *dstA, void *dstT) {
  int64_t r = ix(L->r, i), w = ix(L->w, i);
  if (L->dtype == JPO_I32) {
    const uint32_t *sa = (const uint32_t *)srcA, *sx = (const uint32_t *)srcX;
    uint32_t *da = (uint32_t *)dstA, *dt = (uint32_t *)dstT;
    uint32_t c0 = L->c0, c1 = L->c1;
    switch (L->op) {
    case JPO_OP_ADD_C:    da[w] = sa[r] + c0; break;
    case JPO_OP_SAXPY:    da[w] = c0 * sx[r] + sa[w]; break;
    case JPO_OP_PRIV_TMP: { uint32_t t = c0 * sx[r]; dt[ix(L->s, i)] = t; da[w] = t + c1; } break;
    case JPO_OP_STENCIL2: da[w] = (sa[r] + sa[ix(L->r2, i)]) * c0; break;
    }
  } else {
    const float *sa = (const float *)srcA, *sx = (const float *)srcX;
    float *da = (float *)dstA, *dt = (float *)dstT;
    float c0 = f32(L->c0), c1 = f32(L->c1);
    switch (L->op) {
    case JPO_OP_ADD_C:    da[w] = sa[r] + c0; break;
    case JPO_OP_SAXPY:    { float p = c0 * sx[r]; float q = p + sa[w]; da[w] = q; } break;
    case JPO_OP_PRIV_TMP: { float t = c0 * sx[r]; dt[ix(L->s, i)] = t; float q = t + c1; da[w] = q; } break;
    case JPO_OP_STENCIL2: { float p = sa[r] + sa[ix(L->r2, i)]; float q = p * c0; da[w] = q; } break;
    }
  }
}

/* for i = 0..n-1 execute the body in program order. */
int jpo_run_seq(const jpo_loop *L) {
  if (!op_valid(L)) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  for (int64_t i = 0; i < L->n; i++) body(L, i, L->A, L->X, L->A, L->T);
  return JPO_OK;
}

int jpo_run_order(const jpo_loop *L, const int64_t *perm) {
  if (!op_valid(L) || !perm) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  for (int64_t k = 0; k < L->n; k++) body(L, perm[k], L->A, L->X, L->A, L->T);
  return JPO_OK;
}

/* ---------------------------------------------------------------------------
 * Dependency density, reading A1 (the paper's quantitative model is in its
 * ref [4]; P:L626-627 prints a fraction, "about 0.012"):
 *   raw_i: some exposed read a of i was written by some j < i
 *   war_i: some write a of i was read (exposed or covered) by some j < i
 *   waw_i: some write a of i was written by some j < i
 * Arrays are distinct (reading A14); granularity is the element.
 * ------------------------------------------------------------------------- */
int jpo_profile_run(const jpo_loop *L, jpo_profile *out, uint8_t *flags) {
  if (!op_valid(L) || !out) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  int64_t len[3] = {L->len_A, L->len_X, L->len_T};
  int64_t *first_writer[3]; uint8_t *read_before[3];
  for (int k = 0; k < 3; k++) {
    int64_t m = len[k] > 0 ? len[k] : 1;
    first_writer[k] = (int64_t *)malloc(sizeof(int64_t) * m);
    read_before[k] = (uint8_t *)calloc(m, 1);
    for (int64_t a = 0; a < m; a++) first_writer[k][a] = -1;
  }
  memset(out, 0, sizeof(*out));
  out->n = L->n; out->first_raw_iter = -1;
  out->raw_pairs = out->war_pairs = out->waw_pairs = -1;
  for (int64_t i = 0; i < L->n; i++) {
    accs_t s; accesses(L, i, &s);
    int raw = 0, war = 0, waw = 0;
    for (int k = 0; k < s.nrexp; k++) if (first_writer[s.rexp[k].arr][s.rexp[k].a] >= 0) raw = 1;
    for (int k = 0; k < s.nwr; k++) {
      if (read_before[s.wr[k].arr][s.wr[k].a]) war = 1;
      if (first_writer[s.wr[k].arr][s.wr[k].a] >= 0) waw = 1;
    }
    /* record i's accesses only after its own checks */
    for (int k = 0; k < s.nrexp; k++) read_before[s.rexp[k].arr][s.rexp[k].a] = 1;
    for (int k = 0; k < s.nrcov; k++) read_before[s.rcov[k].arr][s.rcov[k].a] = 1;
    for (int k = 0; k < s.nwr; k++) if (first_writer[s.wr[k].arr][s.wr[k].a] < 0) first_writer[s.wr[k].arr][s.wr[k].a] = i;
    out->raw_iters += raw; out->war_iters += war; out->waw_iters += waw;
    if (raw && out->first_raw_iter < 0) out->first_raw_iter = i;
    if (flags) flags[i] = (uint8_t)(raw | (war << 1) | (waw << 2));
  }
  for (int k = 0; k < 3; k++) { free(first_writer[k]); free(read_before[k]); }
  return JPO_OK;
}

static int meets(const acc_t *x, int nx, const acc_t *y, int ny) {
  for (int p = 0; p < nx; p++) for (int q = 0; q < ny; q++)
    if (x[p].arr == y[q].arr && x[p].a == y[q].a) return 1;
  return 0;
}

/* every ordered pair (j < i). */
int jpo_pairs(const jpo_loop *L, jpo_profile *out, uint8_t *flags) {
  if (!op_valid(L) || !out) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  memset(out, 0, sizeof(*out));
  out->n = L->n; out->first_raw_iter = -1;
  for (int64_t i = 0; i < L->n; i++) {
    accs_t si; accesses(L, i, &si);
    acc_t rall_i[3]; int nrall_i = 0; (void)rall_i; (void)nrall_i;
    int raw = 0, war = 0, waw = 0;
    for (int64_t j = 0; j < i; j++) {
      accs_t sj; accesses(L, j, &sj);
      acc_t rall_j[3]; int nrall_j = 0;
      for (int k = 0; k < sj.nrexp; k++) rall_j[nrall_j++] = sj.rexp[k];
      for (int k = 0; k < sj.nrcov; k++) rall_j[nrall_j++] = sj.rcov[k];
      if (meets(sj.wr, sj.nwr, si.rexp, si.nrexp)) { raw = 1; out->raw_pairs++; }
      if (meets(rall_j, nrall_j, si.wr, si.nwr))   { war = 1; out->war_pairs++; }
      if (meets(sj.wr, sj.nwr, si.wr, si.nwr))     { waw = 1; out->waw_pairs++; }
    }
    out->raw_iters += raw; out->war_iters += war; out->waw_iters += waw;
    if (raw && out->first_raw_iter < 0) out->first_raw_iter = i;
    if (flags) flags[i] = (uint8_t)(raw | (war << 1) | (waw << 2));
  }
  return JPO_OK;
}

/* RAW sources (profile-guided mode B): src[j] = 1 iff
 * some write of j is an exposed read of a LATER iteration, i.e. j is the
 * earlier end of a RAW pair (W(j) ∩ R_exp(i) != {} for some i > j, reading
 * A1's pair relation).  Single backward pass: before recording i's exposed
 * reads, its writes are checked against the addresses read by iterations > i.
 * Only such writes can make an in-window RAW violation (reading A7).       */
int jpo_raw_sources(const jpo_loop *L, uint8_t *src) {
  if (!op_valid(L) || !src) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  int64_t len[3] = {L->len_A, L->len_X, L->len_T};
  uint8_t *read_after[3];
  for (int k = 0; k < 3; k++) read_after[k] = (uint8_t *)calloc(len[k] > 0 ? len[k] : 1, 1);
  for (int64_t i = L->n - 1; i >= 0; i--) {
    accs_t s; accesses(L, i, &s);
    int f = 0;
    for (int k = 0; k < s.nwr; k++) if (read_after[s.wr[k].arr][s.wr[k].a]) f = 1;
    src[i] = (uint8_t)f;
    for (int k = 0; k < s.nrexp; k++) read_after[s.rexp[k].arr][s.rexp[k].a] = 1;
  }
  for (int k = 0; k < 3; k++) free(read_after[k]);
  return JPO_OK;
}

/* ---------------------------------------------------------------------------
 * GPU-TLS as a definition (P:L314-333 SE/DC/commit/recovery; P:L367-375 mode
 * B restarts "from the violating warp"; readings A6, A7, A8):
 *   ws = 0; loop: we = min(ws+W, n);
 *   fv = min{ i in [ws,we) : exists j in [ws,i) with W(j) ∩ R_exp(i) != {} } or we
 *   commit [ws, fv) in program order; windows++; violations += (fv < we);
 *   executed += we-ws; ws = fv.
 * ------------------------------------------------------------------------- */
static int64_t pow2ceil(int64_t x) { int64_t p = 1; while (p < x) p <<= 1; return p; }
static int64_t clampi(int64_t x, int64_t lo, int64_t hi) { return x < lo ? lo : x > hi ? hi : x; }

/* Reading A8.  Initial: ceil(4n/raw) rounded up to a power of two when a
 * profile with raw > 0 is known, w_max when the profile says raw == 0, 4096
 * with no profile; all clamped to [32, w_max].  After a window that committed
 * c iterations: pow2ceil(2*max(c,16)) clamped to [32, w_max].               */
int64_t jpo_tls_next_window(int64_t n, int64_t prof_raw_iters, int64_t prev_commit, int64_t w_max) {
  if (prev_commit < 0) {
    int64_t w0;
    if (prof_raw_iters < 0) w0 = 4096;
    else if (prof_raw_iters == 0) w0 = w_max;
    else w0 = pow2ceil((4 * n + prof_raw_iters - 1) / prof_raw_iters);
    return clampi(w0, 32, w_max);
  }
  int64_t c = prev_commit > 16 ? prev_commit : 16;
  return clampi(pow2ceil(2 * c), 32, w_max);
}

int jpo_sim_tls(const jpo_loop *L, int64_t window, int64_t w_max, int64_t prof_raw_iters,
                jpo_tls_stats *st) {
  if (!op_valid(L) || !st || window < 0 || (window == 0 && w_max < 32)) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  memset(st, 0, sizeof(*st));
  /* writer_window[arr][a] = 1 + index of the last window in which some
   * iteration already scanned wrote a (the in-window write set W([ws,i))). */
  int64_t len[3] = {L->len_A, L->len_X, L->len_T};
  int64_t *wmark[3];
  for (int k = 0; k < 3; k++) wmark[k] = (int64_t *)calloc(len[k] > 0 ? len[k] : 1, sizeof(int64_t));
  int64_t ws = 0, W = window > 0 ? window : jpo_tls_next_window(L->n, prof_raw_iters, -1, w_max);
  while (ws < L->n) {
    int64_t we = ws + W < L->n ? ws + W : L->n;
    int64_t tag = st->windows + 1, fv = we;
    for (int64_t i = ws; i < we; i++) {
      accs_t s; accesses(L, i, &s);
      int viol = 0;
      for (int k = 0; k < s.nrexp; k++) if (wmark[s.rexp[k].arr][s.rexp[k].a] == tag) viol = 1;
      if (viol) { fv = i; break; }
      for (int k = 0; k < s.nwr; k++) wmark[s.wr[k].arr][s.wr[k].a] = tag;
    }
    for (int64_t i = ws; i < fv; i++) body(L, i, L->A, L->X, L->A, L->T);
    st->windows++;
    if (fv < we) st->violations++;
    st->executed += we - ws;
    st->committed += fv - ws;
    if (window == 0) W = jpo_tls_next_window(L->n, prof_raw_iters, fv - ws, w_max);
    ws = fv;
  }
  for (int k = 0; k < 3; k++) free(wmark[k]);
  return JPO_OK;
}

/* ---------------------------------------------------------------------------
 * TLS with on-chip recovery (reading B7).  P:L320-333 lists the four phases of
 * a sub-loop: SE, DC, commit of the threads "not found to have violations",
 * and mis-speculation recovery.  Written as its definition: DC over the window
 * exactly as in jpo_sim_tls but without stopping at the first violator (every
 * violating iteration is counted), then the window's iterations take effect
 * in program order -- the state a correct recovery must reach.
 * ------------------------------------------------------------------------- */
int jpo_sim_tls_fwd(const jpo_loop *L, int64_t window, jpo_tls_stats *st) {
  if (!op_valid(L) || !st || window <= 0) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  memset(st, 0, sizeof(*st));
  int64_t len[3] = {L->len_A, L->len_X, L->len_T};
  int64_t *wmark[3];
  for (int k = 0; k < 3; k++) wmark[k] = (int64_t *)calloc(len[k] > 0 ? len[k] : 1, sizeof(int64_t));
  for (int64_t ws = 0; ws < L->n; ws += window) {
    int64_t we = ws + window < L->n ? ws + window : L->n;
    int64_t tag = st->windows + 1, v = 0;
    for (int64_t i = ws; i < we; i++) {
      accs_t s; accesses(L, i, &s);
      int viol = 0;
      for (int k = 0; k < s.nrexp; k++) if (wmark[s.rexp[k].arr][s.rexp[k].a] == tag) viol = 1;
      v += viol;
      for (int k = 0; k < s.nwr; k++) wmark[s.wr[k].arr][s.wr[k].a] = tag;
    }
    for (int64_t i = ws; i < we; i++) body(L, i, L->A, L->X, L->A, L->T);
    st->windows++;
    st->violations += v;
    st->executed += (we - ws) + v;
    st->committed += we - ws;
  }
  for (int k = 0; k < 3; k++) free(wmark[k]);
  return JPO_OK;
}

/* ---------------------------------------------------------------------------
 * Privatized execution PE(V) (Table I private(list)
 * P:L276; readings A9, A10): exposed reads see the pre-loop snapshot, covered
 * reads see the iteration's own private copy, and after all iterations the
 * highest-i writer of each address wins; unwritten addresses keep their value.
 * ------------------------------------------------------------------------- */
int jpo_sim_priv(const jpo_loop *L) {
  if (!op_valid(L)) return JPO_ERR_ARG;
  int e = check_indices(L); if (e) return e;
  size_t bytesA = (size_t)(L->len_A > 0 ? L->len_A : 1) * 4, bytesX = (size_t)(L->len_X > 0 ? L->len_X : 1) * 4;
  void *snapA = malloc(bytesA), *snapX = malloc(bytesX);
  if (L->len_A > 0) memcpy(snapA, L->A, (size_t)L->len_A * 4);
  if (L->len_X > 0 && L->X) memcpy(snapX, L->X, (size_t)L->len_X * 4);
  /* ascending i: a later writer's store overwrites an earlier one's. */
  for (int64_t i = 0; i < L->n; i++) body(L, i, snapA, snapX, L->A, L->T);
  free(snapA); free(snapX);
  return JPO_OK;
}
