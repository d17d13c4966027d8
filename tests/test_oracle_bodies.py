"""Pins of the oracle's remaining body x dtype cases, its order-taking entry,
its pair counts and its IEEE special values (-m "not gpu").

Round 1 pinned ADD_C-i32, STENCIL2-i32, SAXPY-f32 and PRIV_TMP-f32
independently; this file pins the other four bodies of ``jpo_run_seq``
(ADD_C-f32, SAXPY-i32, PRIV_TMP-i32, STENCIL2-f32), ``jpo_run_order`` on loops
whose result depends on the order, ``jpo_pairs``' pair counts, and the fp32
bodies on IEEE specials (reading A12: RN-even, no contraction, no FTZ/DAZ;
DESIGN.md Sec.3 "A12b" for NaN).

Every expected value here is computed WITHOUT the oracle's arithmetic:
  * int32 bodies with Python integers reduced mod 2^32 (reading A11, Java int),
    in closed forms (sums, last writers) the loop shape makes exact;
  * fp32 bodies with exact rationals rounded by ``rn32`` below, a restatement
    of IEEE 754 binary32 round-to-nearest-even (subnormals and overflow
    included) -- P:L486-488 does not fix a precision, reading A12 does;
  * specials by the IEEE rules for inf / NaN / signed zero written out.
A plausible slip on either side (a dropped Y[w] term, (a+b)*c computed as
a*c+b*c, one rounding instead of two, flush-to-zero, an order-ignoring
``jpo_run_order``) fails at least one case below; each such case also checks
that it discriminates.
"""
import fractions
import math

import numpy as np
import pytest

import oracle as O

Fr = fractions.Fraction
M32 = 1 << 32


# ----------------------------------------------------------------------------
# IEEE binary32 round-to-nearest-even from an exact rational
# ----------------------------------------------------------------------------
EMIN, PREC = -126, 24            # binary32: normal exponent range starts at 2^-126
MAXF = (2 - Fr(1, 2 ** 23)) * Fr(2) ** 127
OVF = (2 - Fr(1, 2 ** 24)) * Fr(2) ** 127      # halfway to 2^128: rounds to inf from here


def rn32(q: Fr, neg_zero: bool = False) -> np.float32:
    """Nearest binary32 to q, ties to even; subnormals kept (no FTZ), overflow to
    +-inf.  A result that rounds to zero keeps q's sign (IEEE 754 Sec. 6.3)."""
    if q == 0:
        return np.float32(-0.0) if neg_zero else np.float32(0.0)
    sign = -1 if q < 0 else 1
    a = abs(q)
    if a >= OVF:
        return np.float32(sign * np.inf)
    e = a.numerator.bit_length() - a.denominator.bit_length()
    while Fr(2) ** e > a:
        e -= 1
    while Fr(2) ** (e + 1) <= a:
        e += 1
    ulp = Fr(2) ** (max(e, EMIN) - (PREC - 1))        # fixed 2^-149 in the subnormal range
    m = a / ulp
    fl = m.numerator // m.denominator
    rem = m - fl
    if rem > Fr(1, 2) or (rem == Fr(1, 2) and fl % 2 == 1):
        fl += 1
    v = fl * ulp
    if v == 0:
        return np.float32(-0.0) if sign < 0 else np.float32(0.0)
    return np.float32(sign * float(v))


def F(x) -> Fr:
    return Fr(float(x))


def is_neg(x) -> bool:
    return math.copysign(1.0, float(x)) < 0


def ieee_mul(a: np.float32, b: np.float32) -> np.float32:
    a, b = float(a), float(b)
    if math.isnan(a) or math.isnan(b):
        return np.float32(np.nan)
    neg = is_neg(a) != is_neg(b)
    if math.isinf(a) or math.isinf(b):
        if a == 0 or b == 0:
            return np.float32(np.nan)            # 0 * inf
        return np.float32(-np.inf if neg else np.inf)
    if a == 0 or b == 0:
        return np.float32(-0.0 if neg else 0.0)
    return rn32(Fr(a) * Fr(b))


def ieee_add(a: np.float32, b: np.float32) -> np.float32:
    a, b = float(a), float(b)
    if math.isnan(a) or math.isnan(b):
        return np.float32(np.nan)
    if math.isinf(a) and math.isinf(b):
        return np.float32(a) if (a > 0) == (b > 0) else np.float32(np.nan)
    if math.isinf(a) or math.isinf(b):
        return np.float32(a if math.isinf(a) else b)
    s = Fr(a) + Fr(b)
    if s == 0:   # exact zero sum: +0 under RN unless both operands are -0
        return np.float32(-0.0) if (a == 0 and b == 0 and is_neg(a) and is_neg(b)) else np.float32(0.0)
    return rn32(s)


def f32(x) -> np.float32:
    return np.float32(x)


def nan_eq(got: np.ndarray, exp) -> bool:
    """Reading A12b: NaN results compare as NaN (payloads are not part of the
    contract); everything else compares bit for bit (so +0 != -0)."""
    g = np.asarray(got, dtype=np.float32)
    e = np.asarray(exp, dtype=np.float32)
    gn, en = np.isnan(g), np.isnan(e)
    if not np.array_equal(gn, en):
        return False
    return g[~gn].view(np.uint32).tolist() == e[~en].view(np.uint32).tolist()


def grid_f32(rng, n, lo_exp=-30, hi_exp=30):
    """fp32 values over many binades (not just the [-1, 1) 2^-22 grid)."""
    m = rng.integers(1 << 23, 1 << 24, size=n).astype(np.float64)
    e = rng.integers(lo_exp, hi_exp, size=n)
    s = np.where(rng.random(n) < 0.5, -1.0, 1.0)
    return (s * m * np.exp2(e - 23.0)).astype(np.float32)


# ----------------------------------------------------------------------------
# ADD_C fp32: A[w] = A[r] + c0
# ----------------------------------------------------------------------------
def test_rn32_self_checks():
    """The rounding restatement against facts about binary32 (no oracle involved)."""
    assert rn32(Fr(1) + Fr(1, 2 ** 24)) == np.float32(1.0)               # tie -> even
    assert rn32(Fr(1) + Fr(3, 2 ** 25)) == np.float32(1.0 + 2.0 ** -23)  # above the tie
    assert rn32(Fr(1, 2 ** 149)).view(np.uint32) == 1                    # smallest subnormal
    assert rn32(Fr(1, 2 ** 150)) == 0 and not is_neg(rn32(Fr(1, 2 ** 150)))  # tie to even (0)
    assert rn32(Fr(3, 2 ** 151)).view(np.uint32) == 1
    assert rn32(-Fr(1, 2 ** 151)).view(np.uint32) == 0x80000000          # underflow keeps the sign
    assert rn32(MAXF) == np.float32(3.4028234663852886e38)
    assert np.isinf(rn32(OVF)) and not np.isinf(rn32(OVF - Fr(1, 2 ** 200)))


@pytest.mark.parametrize("n", [1, 7, 500])
def test_addc_f32_permutation_and_chain(n):
    rng = np.random.default_rng(40 + n)
    A0 = grid_f32(rng, n)
    c = f32(1.1)
    pi = rng.permutation(n).astype(np.int32)
    # permutation self-update: every address once, A'[a] = fl(A[a] + c)
    L = O.Loop(O.OP_ADD_C, O.F32, n, A0, r=pi, w=pi, c0=c)
    exp = [rn32(F(a) + F(c)) for a in A0]
    assert nan_eq(O.run_seq(L)[1], exp)
    # prefix chain w = i, r = max(i-1, 0): one rounding per link, in order
    L = O.Loop(O.OP_ADD_C, O.F32, n, A0, r=np.maximum(np.arange(n) - 1, 0), w=np.arange(n), c0=c)
    v, exp = F(A0[0]), []
    for _ in range(n):
        v = F(rn32(v + F(c)))
        exp.append(float(v))
    assert nan_eq(O.run_seq(L)[1], exp)
    if n >= 7:   # a sum rounded once differs from the chain: the pin discriminates
        once = [rn32(F(A0[0]) + (i + 1) * F(c)) for i in range(n)]
        assert not nan_eq(np.array(exp, np.float32), once)


# ----------------------------------------------------------------------------
# SAXPY int32: Y[w] = c0*X[r] + Y[w]  (mod 2^32)
# ----------------------------------------------------------------------------
@pytest.mark.parametrize("n", [1, 9, 1000])
def test_saxpy_i32_closed_forms(n):
    rng = np.random.default_rng(60 + n)
    X = rng.integers(-2 ** 31, 2 ** 31, size=n + 3, dtype=np.int64).astype(np.int32)
    Y = rng.integers(-2 ** 31, 2 ** 31, size=n + 5, dtype=np.int64).astype(np.int32)
    c = 2 ** 31 - 3
    u = lambda a: [int(x) & 0xFFFFFFFF for x in a]  # noqa: E731
    xs, ys = u(X), u(Y)
    r = rng.integers(0, n + 3, size=n).astype(np.int32)
    # distinct writes: Y'[w[i]] = c*X[r[i]] + Y[w[i]]
    w = rng.permutation(n + 5)[:n].astype(np.int32)
    L = O.Loop(O.OP_SAXPY, O.I32, n, Y, r=r, w=w, X=X, c0=c)
    exp = list(ys)
    for i in range(n):
        exp[w[i]] = (c * xs[r[i]] + ys[w[i]]) % M32
    assert O.run_seq(L)[1].view(np.uint32).tolist() == exp
    # every iteration into one address k: Y'[k] = Y[k] + c * sum X[r[i]]  (the Y[w] term accumulates)
    k = 2
    L = O.Loop(O.OP_SAXPY, O.I32, n, Y, r=r, w=np.full(n, k, np.int32), X=X, c0=c)
    exp = list(ys)
    exp[k] = (ys[k] + c * sum(xs[j] for j in r)) % M32
    got = O.run_seq(L)[1].view(np.uint32).tolist()
    assert got == exp
    if n > 1:   # dropping the Y[w] read would leave only the last term
        assert exp[k] != (c * xs[r[-1]] + ys[k]) % M32


# ----------------------------------------------------------------------------
# PRIV_TMP int32: T[s] = c0*X[r]; Y[w] = T[s] + c1
# ----------------------------------------------------------------------------
@pytest.mark.parametrize("n,S", [(1, 4), (50, 8), (3000, 64)])
def test_priv_tmp_i32_closed_form(n, S):
    rng = np.random.default_rng(70 + n)
    X = rng.integers(-2 ** 31, 2 ** 31, size=n, dtype=np.int64).astype(np.int32)
    T0 = rng.integers(-2 ** 31, 2 ** 31, size=S, dtype=np.int64).astype(np.int32)
    s = rng.integers(0, S - 2, size=n).astype(np.int32)        # the last two slots are never written
    c0, c1 = 0x7FFF_FFF1, -(2 ** 31) + 9
    xs = [int(x) & 0xFFFFFFFF for x in X]
    L = O.Loop(O.OP_PRIV_TMP, O.I32, n, np.zeros(n, np.int32), s=s, X=X, T=T0, c0=c0, c1=c1)
    st, Y, T = O.run_seq(L)
    assert st == O.OK
    assert Y.view(np.uint32).tolist() == [(c0 * x + c1) % M32 for x in xs]
    last = {}
    for i, k in enumerate(s.tolist()):
        last[k] = i
    expT = [(c0 * xs[last[k]]) % M32 if k in last else int(T0[k]) & 0xFFFFFFFF for k in range(S)]
    assert T.view(np.uint32).tolist() == expT
    # 2-to-1 writes of Y (w[i] = i // 2): the later (odd) iteration's value wins
    m = (n + 1) // 2
    L = O.Loop(O.OP_PRIV_TMP, O.I32, n, np.zeros(m, np.int32), w=(np.arange(n) // 2).astype(np.int32), s=s, X=X,
               T=T0, c0=c0, c1=c1)
    Y = O.run_seq(L)[1].view(np.uint32).tolist()
    assert Y == [(c0 * xs[min(2 * k + 1, n - 1)] + c1) % M32 for k in range(m)]


# ----------------------------------------------------------------------------
# STENCIL2 fp32: A[w] = (A[r] + A[r2]) * c0
# ----------------------------------------------------------------------------
def test_stencil2_f32_two_roundings_and_gauss_seidel():
    rng = np.random.default_rng(81)
    m = 3000
    A0 = grid_f32(rng, 2 * m, -20, 20)
    c = f32(1.1)
    r = (m + rng.integers(0, m, size=m)).astype(np.int32)       # reads from the read-only half
    r2 = (m + rng.integers(0, m, size=m)).astype(np.int32)
    w = rng.permutation(m).astype(np.int32)
    L = O.Loop(O.OP_STENCIL2, O.F32, m, A0, r=r, r2=r2, w=w, c0=c)
    exp = A0.copy()
    for i in range(m):
        exp[w[i]] = ieee_mul(ieee_add(A0[r[i]], A0[r2[i]]), c)
    got = O.run_seq(L)[1]
    assert nan_eq(got, exp)
    distributed = A0.copy()     # (a*c + b*c): the pin discriminates the factorisation
    for i in range(m):
        distributed[w[i]] = ieee_add(ieee_mul(A0[r[i]], c), ieee_mul(A0[r2[i]], c))
    assert not nan_eq(distributed, exp)
    # Gauss-Seidel sweep: reads the value written by i-1 and the old i+1
    n = 400
    B0 = grid_f32(rng, n, -3, 3)
    ar = np.arange(n)
    c = f32(0.3)
    L = O.Loop(O.OP_STENCIL2, O.F32, n, B0, r=np.maximum(ar - 1, 0), r2=np.minimum(ar + 1, n - 1), w=ar, c0=c)
    B = B0.copy()
    for i in range(n):
        B[i] = ieee_mul(ieee_add(B[max(i - 1, 0)], B[min(i + 1, n - 1)]), c)
    assert nan_eq(O.run_seq(L)[1], B)


# ----------------------------------------------------------------------------
# jpo_run_order on loops whose result depends on the order
# ----------------------------------------------------------------------------
@pytest.mark.parametrize("seed", range(5))
def test_run_order_follows_perm(seed):
    rng = np.random.default_rng(90 + seed)
    n = 64
    A0 = rng.integers(0, 1 << 20, size=n + 1).astype(np.int32)
    perm = rng.permutation(n)
    # every iteration writes address 0 from a distinct source: the LAST executed wins
    L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=np.arange(1, n + 1), w=np.zeros(n, np.int32), c0=5)
    got = O.run_order(L, perm)[1]
    assert int(got[0]) == int(A0[perm[-1] + 1]) + 5
    assert got[1:].tolist() == A0[1:].tolist()
    # prefix chain run backwards: no link sees its predecessor's new value
    ar = np.arange(n)
    C = O.Loop(O.OP_ADD_C, O.I32, n, A0[:n], r=np.maximum(ar - 1, 0), w=ar, c0=7)
    back = O.run_order(C, ar[::-1].copy())[1]
    assert back.tolist() == [int(A0[max(i - 1, 0)]) + 7 if i > 0 else int(A0[0]) + 7 for i in range(n)]
    fwd = O.run_order(C, ar)[1]
    assert fwd.tolist() == [int(A0[0]) + 7 * (i + 1) for i in range(n)]      # and forwards it chains
    assert O.run_seq(C)[1].tolist() == fwd.tolist()


def test_run_order_rejects_missing_perm():
    L = O.Loop(O.OP_ADD_C, O.I32, 4, np.zeros(4, np.int32), c0=1)
    lib = O.oracle._load()
    assert lib.jpo_run_order(O.oracle.C.byref(L._c()), None) == O.oracle.ERR_ARG


# ----------------------------------------------------------------------------
# jpo_pairs: pair counts
# ----------------------------------------------------------------------------
def _sets(op, i, r, r2, w, s):
    ix = lambda a: i if a is None else int(a[i])  # noqa: E731
    if op == O.OP_ADD_C:
        return {("A", ix(r))}, {("A", ix(w))}
    if op == O.OP_SAXPY:
        return {("X", ix(r)), ("A", ix(w))}, {("A", ix(w))}
    if op == O.OP_PRIV_TMP:
        return {("X", ix(r)), ("T", ix(s))}, {("T", ix(s)), ("A", ix(w))}   # all reads (covered included)
    return {("A", ix(r)), ("A", ix(r2))}, {("A", ix(w))}


def _exposed(op, i, r, r2, w, s):
    ix = lambda a: i if a is None else int(a[i])  # noqa: E731
    if op == O.OP_PRIV_TMP:
        return {("X", ix(r))}
    return _sets(op, i, r, r2, w, s)[0]


def brute_pair_counts(op, n, r=None, r2=None, w=None, s=None):
    """Reading A1's pair relations counted over all j < i (one count per pair)."""
    raw = war = waw = 0
    for i in range(n):
        ri, wi = _sets(op, i, r, r2, w, s)
        ei = _exposed(op, i, r, r2, w, s)
        for j in range(i):
            rj, wj = _sets(op, j, r, r2, w, s)
            raw += bool(wj & ei)
            war += bool(rj & wi)
            waw += bool(wj & wi)
    return raw, war, waw


def test_pair_counts_closed_forms():
    n = 40
    ar = np.arange(n, dtype=np.int32)
    A0 = np.zeros(n, np.int32)
    # every iteration writes one address: all n(n-1)/2 pairs are WAW
    p = O.pairs(O.Loop(O.OP_ADD_C, O.I32, n, A0, r=ar, w=np.zeros(n, np.int32), c0=1))
    assert p["waw_pairs"] == n * (n - 1) // 2
    # ... and read it too (r = w = 0): every pair is RAW, WAR and WAW
    p = O.pairs(O.Loop(O.OP_ADD_C, O.I32, n, A0, r=np.zeros(n, np.int32), w=np.zeros(n, np.int32), c0=1))
    assert (p["raw_pairs"], p["war_pairs"], p["waw_pairs"]) == (n * (n - 1) // 2,) * 3
    # prefix chain: exactly the n-1 links are RAW pairs
    p = O.pairs(O.Loop(O.OP_ADD_C, O.I32, n, A0, r=np.maximum(ar - 1, 0), w=ar, c0=1))
    assert (p["raw_pairs"], p["war_pairs"], p["waw_pairs"]) == (n - 1, 0, 0)
    # Gauss-Seidel: i reads i-1 (RAW) and i+1 (read before written: WAR pair (i, i+1)), plus the edges
    p = O.pairs(O.Loop(O.OP_STENCIL2, O.I32, n, A0, r=np.maximum(ar - 1, 0), r2=np.minimum(ar + 1, n - 1), w=ar,
                       c0=1))
    assert (p["raw_pairs"], p["war_pairs"], p["waw_pairs"]) == (n - 1, n - 1, 0)
    # PRIV_TMP over S slots: WAR = WAW = pairs sharing a slot (the covered read counts)
    S = 4
    s = (ar % S).astype(np.int32)
    p = O.pairs(O.Loop(O.OP_PRIV_TMP, O.I32, n, A0, s=s, X=A0, T=np.zeros(S, np.int32), c0=1))
    same = S * ((n // S) * (n // S - 1) // 2)
    assert (p["raw_pairs"], p["war_pairs"], p["waw_pairs"]) == (0, same, same)


@pytest.mark.parametrize("seed", range(24))
def test_pair_counts_random_vs_bruteforce(seed):
    rng = np.random.default_rng(300 + seed)
    op = seed % 4
    n = int(rng.integers(1, 30))
    la, lt = int(rng.integers(1, 8)), int(rng.integers(1, 5))
    lx = n + 2
    r = rng.integers(0, lx if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else la, size=n).astype(np.int32)
    w = rng.integers(0, la, size=n).astype(np.int32)
    r2 = rng.integers(0, la, size=n).astype(np.int32) if op == O.OP_STENCIL2 else None
    s = rng.integers(0, lt, size=n).astype(np.int32) if op == O.OP_PRIV_TMP else None
    L = O.Loop(op, O.I32, n, np.zeros(la, np.int32), r=r, r2=r2, w=w, s=s, X=np.zeros(lx, np.int32),
               T=np.zeros(lt, np.int32), c0=1)
    p = O.pairs(L)
    assert (p["raw_pairs"], p["war_pairs"], p["waw_pairs"]) == brute_pair_counts(op, n, r, r2, w, s)


# ----------------------------------------------------------------------------
# IEEE specials through every fp32 body (reading A12, A12b)
# ----------------------------------------------------------------------------
SPECIALS = np.array([0.0, -0.0, np.inf, -np.inf, np.nan, 1e-45, -1e-45, 1.1754942e-38, 1.17549435e-38,
                     -5.877472e-39, 3.4028235e38, -3.4028235e38, 1.7e38, 2.9e-39, 1.0, -1.0], dtype=np.float32)


def special_vec(rng, n):
    """Specials mixed with ordinary values (and a signalling-free quiet NaN with a payload)."""
    v = np.concatenate([SPECIALS, grid_f32(rng, max(n - len(SPECIALS), 0), -140, 127)])[:n].copy()
    v = v.view(np.uint32)
    v[4] = 0x7FC12345            # a quiet NaN with a payload
    return v.view(np.float32)


def test_specials_saxpy_and_addc():
    rng = np.random.default_rng(5)
    n = 400
    X, Y = special_vec(rng, n), special_vec(rng, n)[::-1].copy()
    for c in (f32(1.1), f32(-0.5), f32(0.0), f32(np.inf), f32(1e-40)):
        got = O.run_seq(O.Loop(O.OP_SAXPY, O.F32, n, Y, X=X, c0=c))[1]
        exp = [ieee_add(ieee_mul(c, x), y) for x, y in zip(X, Y)]
        assert nan_eq(got, exp)
        got = O.run_seq(O.Loop(O.OP_ADD_C, O.F32, n, X, c0=c))[1]
        assert nan_eq(got, [ieee_add(x, c) for x in X])
    # denormals survive (no FTZ/DAZ): 1.1 * smallest subnormal = smallest subnormal
    got = O.run_seq(O.Loop(O.OP_SAXPY, O.F32, 1, np.zeros(1, np.float32), X=np.array([1e-45], np.float32),
                           c0=f32(1.1)))[1]
    assert got.view(np.uint32)[0] == 1


def test_specials_priv_tmp_and_stencil2():
    rng = np.random.default_rng(6)
    n, S = 300, 7
    X = special_vec(rng, n)
    s = rng.integers(0, S, size=n).astype(np.int32)
    c0, c1 = f32(1.1), f32(-0.0)
    st, Y, T = O.run_seq(O.Loop(O.OP_PRIV_TMP, O.F32, n, np.zeros(n, np.float32), s=s, X=X,
                                T=np.full(S, 2.0, np.float32), c0=c0, c1=c1))
    t = [ieee_mul(c0, x) for x in X]
    assert nan_eq(Y, [ieee_add(v, c1) for v in t])
    last = {int(k): i for i, k in enumerate(s)}
    assert nan_eq(T, [t[last[k]] if k in last else np.float32(2.0) for k in range(S)])
    A0 = special_vec(rng, 2 * n)
    r = (n + rng.integers(0, n, size=n)).astype(np.int32)
    r2 = (n + rng.integers(0, n, size=n)).astype(np.int32)
    got = O.run_seq(O.Loop(O.OP_STENCIL2, O.F32, n, A0, r=r, r2=r2, w=np.arange(n, dtype=np.int32), c0=c0))[1]
    exp = A0.copy()
    for i in range(n):
        exp[i] = ieee_mul(ieee_add(A0[r[i]], A0[r2[i]]), c0)
    assert nan_eq(got, exp)
