"""Counter-based generators and the five BASELINE.json workload recipes.

Generator (restated in DESIGN.md Sec.5):
    sm(x)  = splitmix64 finalizer
    rnd(seed, stream, i) = sm((seed << 40) ^ (stream << 32) ^ i)      (uint64)
Implemented with torch int64 tensors (two's-complement wrap == uint64 wrap for
+, *, ^; right shifts are made logical by masking), so the same code runs on
the CPU (tests, oracle inputs) and on cuda:0 (bench-size inputs) and produces
identical bits.  No arithmetic of the loop method lives here.
"""
from __future__ import annotations

from dataclasses import dataclass, field

import numpy as np
import torch

_M64 = (1 << 64) - 1


def _s64(c: int) -> int:
    c &= _M64
    return c - (1 << 64) if c >= (1 << 63) else c


_K0 = _s64(0x9E3779B97F4A7C15)
_K1 = _s64(0xBF58476D1CE4E5B9)
_K2 = _s64(0x94D049BB133111EB)


def _lsr(x: torch.Tensor, k: int) -> torch.Tensor:
    """Logical right shift of int64 viewed as uint64."""
    return (x >> k) & ((1 << (64 - k)) - 1)


def splitmix64(x: torch.Tensor) -> torch.Tensor:
    x = x + _K0
    x = (x ^ _lsr(x, 30)) * _K1
    x = (x ^ _lsr(x, 27)) * _K2
    return x ^ _lsr(x, 31)


def rnd(seed: int, stream: int, i: torch.Tensor) -> torch.Tensor:
    """uint64 draws (as int64 bit patterns) for counters i."""
    return splitmix64(i ^ _s64((seed << 40) ^ (stream << 32)))


def _ar(n: int, device, start: int = 0) -> torch.Tensor:
    return torch.arange(start, start + n, dtype=torch.int64, device=device)


def permutation(seed: int, n: int, device="cpu", stream: int = 7) -> torch.Tensor:
    """pi = stable argsort of the 63-bit keys rnd(seed, stream, k) >> 1 (int64)."""
    keys = _lsr(rnd(seed, stream, _ar(n, device)), 1)
    return torch.argsort(keys, stable=True)


def i32_data(seed: int, stream: int, n: int, device="cpu", start: int = 0) -> torch.Tensor:
    """A0[k] = rnd(seed, stream, k) & 0xFFFFF   (int32), k in [start, start+n)."""
    return (rnd(seed, stream, _ar(n, device, start)) & 0xFFFFF).to(torch.int32)


def f32_data(seed: int, stream: int, n: int, device="cpu", start: int = 0) -> torch.Tensor:
    """X[k] = (rnd >> 41) * 2^-22 - 1: uniform on [-1, 1) on a 2^-22 grid, exact in fp32.
    Generated in slices so that 2^28-element arrays fit comfortably."""
    out = torch.empty(n, dtype=torch.float32, device=device)
    step = 1 << 24
    for o in range(0, n, step):
        m = _lsr(rnd(seed, stream, _ar(min(step, n - o), device, start + o)), 41).to(torch.float64)
        out[o:o + step] = (m * (2.0 ** -22) - 1.0).to(torch.float32)
    return out


def dependent_set(seed: int, n: int, k: int, device="cpu") -> torch.Tensor:
    """Exactly k distinct local iterations from [1, n): the k smallest keys
    rnd(seed, 4, i) >> 1 (stable by i)."""
    if k <= 0:
        return torch.empty(0, dtype=torch.int64, device=device)
    keys = _lsr(rnd(seed, 4, _ar(n - 1, device, 1)), 1)
    order = torch.argsort(keys, stable=True)[:k]
    return order + 1


def dep_region(seed: int, n: int, addr_base: int, density: float, delta: int, device="cpu"):
    """ADD_C dependent-set construction over n local iterations
    writing a permutation of addresses [addr_base, addr_base+n):
        w = addr_base + pi;  r[i] = w[i] (independent);
        for the K = round(d*n) chosen i: r[i] = w[i - delta_i],
        delta_i = 1 + ((rnd(seed,5,i) >> 1) mod min(i, delta)).
    Designed profile: raw = K, war = 0, waw = 0 exactly."""
    w = permutation(seed, n, device) + addr_base
    r = w.clone()
    k = int(round(density * n))
    dep = dependent_set(seed, n, k, device)
    if k:
        m = torch.clamp(dep, max=delta)
        d = 1 + _lsr(rnd(seed, 5, dep), 1) % m
        r[dep] = w[dep - d]
    return r.to(torch.int32), w.to(torch.int32), k


# fp32 constants of the recipes: 1.1f (0x3F8CCCCD: products really round) and 0.3f
C0_F32 = float(np.float32(1.1))
C1_F32 = float(np.float32(0.3))
C0_I32 = 7


@dataclass
class Workload:
    """One synthetic loop: opcode, dtype, trip count, arrays and constants."""
    name: str
    op: int            # 0 ADD_C, 1 SAXPY, 2 PRIV_TMP, 3 STENCIL2
    dtype: int         # 0 int32, 1 fp32
    n: int
    A: torch.Tensor
    r: torch.Tensor | None = None
    r2: torch.Tensor | None = None
    w: torch.Tensor | None = None
    s: torch.Tensor | None = None
    X: torch.Tensor | None = None
    T: torch.Tensor | None = None
    c0: float | int = 0
    c1: float | int = 0
    meta: dict = field(default_factory=dict)

    def arrays(self) -> dict:
        return {k: getattr(self, k) for k in ("A", "r", "r2", "w", "s", "X", "T") if getattr(self, k) is not None}

    def to(self, device) -> "Workload":
        kw = dict(self.__dict__)
        for k, v in self.arrays().items():
            kw[k] = v.to(device)
        kw["meta"] = dict(self.meta)
        return Workload(**kw)


def config1(density: float = 0.05, n: int = 4096, delta: int = 64, device="cpu") -> Workload:
    """Config 1: tiny indirect ADD_C int32, N=4096, density 0% or 5% (K=205)."""
    seed = 1001
    r, w, k = dep_region(seed, n, 0, density, delta, device)
    return Workload("config1", 0, 0, n, i32_data(seed, 1, n, device), r=r, w=w, c0=C0_I32,
                    meta={"raw": k, "war": 0, "waw": 0, "delta": delta, "density": density})


def config2(n: int = 1 << 28, device="cpu", start: int = 0, count: int | None = None) -> Workload:
    """Config 2: DOALL streaming SAXPY fp32, affine (r = w = NULL).  start/count
    select a shard [start, start+count) of the n-iteration loop (task sharing)."""
    seed = 1002
    count = n - start if count is None else count
    return Workload("config2", 1, 1, count, f32_data(seed, 6, count, device, start),
                    X=f32_data(seed, 2, count, device, start), c0=C0_F32,
                    meta={"raw": 0, "war": 0, "waw": 0, "start": start, "total": n})


def config3(density: float = 0.01, n: int = 1 << 24, delta: int = 1024, device="cpu") -> Workload:
    """Config 3: TLS sweep, ADD_C int32, N=2^24, true-RAW density d (exact)."""
    seed = 1003
    r, w, k = dep_region(seed, n, 0, density, delta, device)
    return Workload("config3", 0, 0, n, i32_data(seed, 1, n, device), r=r, w=w, c0=C0_I32,
                    meta={"raw": k, "war": 0, "waw": 0, "delta": delta, "density": density})


def config3_waw(density: float = 0.01, n: int = 1 << 24, delta: int = 1024, device="cpu") -> Workload:
    """Config 3's shape with write-after-write (the loop on which on-chip
    recovery, reading B7, is illegal and restart TLS must run): w is 2-to-1
    onto [0, n/2) (w[i] = pi[i] >> 1); an independent iteration reads the
    read-only half [n/2, n) (n/2 + (pi2[i] >> 1)); the K = round(d*n) dependent
    iterations (same choice as config 3) read w[i - delta_i].  Designed
    profile: raw = K, waw = n/2 exactly."""
    assert n % 2 == 0
    seed = 1013
    w = _lsr(permutation(seed, n, device), 1)
    r = n // 2 + _lsr(permutation(seed + 1, n, device), 1)
    k = int(round(density * n))
    dep = dependent_set(seed, n, k, device)
    if k:
        m = torch.clamp(dep, max=delta)
        d = 1 + _lsr(rnd(seed, 5, dep), 1) % m
        r[dep] = w[dep - d]
    return Workload("config3_waw", 0, 0, n, i32_data(seed, 1, n, device), r=r.to(torch.int32),
                    w=w.to(torch.int32), c0=C0_I32, meta={"raw": k, "waw": n // 2, "delta": delta,
                                                          "density": density})


def config4(n: int = 1 << 26, slots: int = 1024, device="cpu") -> Workload:
    """Config 4: PRIV_TMP fp32, s[i] = rnd(seed,3,i) mod S (S = 1024 scratch slots)."""
    seed = 1004
    assert slots & (slots - 1) == 0
    s = (rnd(seed, 3, _ar(n, device)) & (slots - 1)).to(torch.int32)
    return Workload("config4", 2, 1, n, f32_data(seed, 6, n, device), s=s, X=f32_data(seed, 2, n, device),
                    T=f32_data(seed, 8, slots, device), c0=C0_F32, c1=C1_F32,
                    meta={"raw": 0, "slots": slots})


def config5(n: int = 1 << 24, density: float = 0.05, delta: int = 1024, device="cpu") -> Workload:
    """Config 5: mixed ADD_C int32 over three regions with disjoint addresses:
      head   [0, n/2)    : r = w = pi over [0, n/2)               -> DOALL
      middle [n/2, 3n/4) : dependent-set loop, d = 5%, delta 1024 -> TLS
      tail   [3n/4, n)   : w 2-to-1 onto [3n/4, 7n/8) (WAW); r[t] = w[t+1] when
                           t+1 is that address's first writer (WAR), else the
                           read-only address 7n/8 + (t' mod n/8)     -> PRIVATIZED
    """
    assert n % 8 == 0 and n >= 64
    seed = 1005
    h, q, m = n // 2, n // 4, n // 8
    r = torch.empty(n, dtype=torch.int64, device=device)
    w = torch.empty(n, dtype=torch.int64, device=device)
    ph = permutation(seed, h, device)
    w[:h] = ph
    r[:h] = ph
    rm, wm, k = dep_region(seed + 100, q, h, density, delta, device)
    r[h:h + q] = rm.to(torch.int64)
    w[h:h + q] = wm.to(torch.int64)
    tb = h + q
    tp = _ar(q, device)                       # t' = t - 3n/4
    pt = permutation(seed + 200, m, device)
    w[tb:] = tb + pt[tp % m]
    nxt = tp + 1
    first_half_next = nxt < m
    r_first = tb + pt[torch.clamp(nxt, max=m - 1)]
    r[tb:] = torch.where(first_half_next, r_first, 7 * m + (tp % m))
    return Workload("config5", 0, 0, n, i32_data(seed, 1, n, device), r=r.to(torch.int32), w=w.to(torch.int32),
                    c0=C0_I32, meta={"regions": [(0, h), (h, h + q), (h + q, n)], "raw": k,
                                     "war": q - 2, "waw": m, "delta": delta, "density": density})


# ---------------------------------------------------------------------------
# workflows of several loops: the shapes of the
# paper's task-stealing applications.  Loops share storage through
# tensor views, so the device ranges they read and write are those of the
# original program.  Each function returns (loops, arrays): a list of
# Workloads in program order and the distinct base tensors they view.
# ---------------------------------------------------------------------------
def workflow_bicg(n: int = 1 << 24, parts: int = 4, device="cpu"):
    """BICG: two independent DOALL loops of similar work (s = c0*p + s and
    t = c0*q + t, fp32), each divided evenly into `parts` subloops."""
    seed = 1006
    p, q = f32_data(seed, 1, n, device), f32_data(seed, 2, n, device)
    s, t = f32_data(seed, 3, n, device), f32_data(seed, 4, n, device)
    m = n // parts
    loops = []
    for X, Y in ((p, s), (q, t)):
        for k in range(parts):
            b, e = k * m, (n if k == parts - 1 else (k + 1) * m)
            loops.append(Workload("bicg", 1, 1, e - b, Y[b:e], X=X[b:e], c0=C0_F32))
    return loops, [p, q, s, t]


def workflow_2mm(n: int = 1 << 24, device="cpu"):
    """2MM: two DOALL loops, the second consuming the first's output
    (y = c0*x + y, then z = c0*y + z, fp32)."""
    seed = 1007
    x, y, z = f32_data(seed, 1, n, device), f32_data(seed, 2, n, device), f32_data(seed, 3, n, device)
    return [Workload("2mm-1", 1, 1, n, y, X=x, c0=C0_F32), Workload("2mm-2", 1, 1, n, z, X=y, c0=C0_F32)], [x, y, z]


def workflow_crypt(n: int = 1 << 24, parts: int = 8, device="cpu"):
    """Crypt: an encryption loop (c[i] = c0*p[pi(i)] + c[i], int32) and a
    decryption loop reading the whole cipher (d[i] = c0*c[pi2(i)] + d[i]),
    each divided evenly into `parts` subloops: 2*parts loops in two batches."""
    seed = 1008
    p, c, d = i32_data(seed, 1, n, device), i32_data(seed, 2, n, device), i32_data(seed, 3, n, device)
    pi, pi2 = permutation(seed, n, device).to(torch.int32), permutation(seed + 1, n, device).to(torch.int32)
    m = n // parts
    loops = []
    for X, Y, perm in ((p, c, pi), (c, d, pi2)):
        for k in range(parts):
            b, e = k * m, (n if k == parts - 1 else (k + 1) * m)
            loops.append(Workload("crypt", 1, 0, e - b, Y[b:e], r=perm[b:e], X=X, c0=C0_I32))
    return loops, [p, c, d, pi, pi2]


# IEEE binary32 specials (reading A12 / A12b tests): +-0, +-inf, quiet NaNs with
# payloads, subnormals, the normal/subnormal boundary and values near overflow
F32_SPECIAL_BITS = [0x00000000, 0x80000000, 0x7F800000, 0xFF800000, 0x7FC00000, 0x7FC12345, 0xFFC00001,
                    0x00000001, 0x80000001, 0x007FFFFF, 0x00800000, 0x80400000, 0x7F7FFFFF, 0xFF7FFFFF,
                    0x7F000000, 0x00200000, 0x3F800000, 0xBF800000]


def f32_specials(seed: int, stream: int, n: int, frac: float = 0.25, device="cpu") -> torch.Tensor:
    """fp32 data of which about `frac` are drawn from F32_SPECIAL_BITS (chosen by
    the counter generator) and the rest from f32_data's grid."""
    out = f32_data(seed, stream, n, device)
    u = rnd(seed, stream + 32, _ar(n, device))
    pick = (_lsr(u, 11) % 1024) < int(frac * 1024)
    which = (u & 0x3FF) % len(F32_SPECIAL_BITS)
    table = torch.tensor(F32_SPECIAL_BITS, dtype=torch.int64, device=device)
    bits = out.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    bits = torch.where(pick, table[which], bits)
    return (bits - ((bits >> 31) << 32)).to(torch.int32).view(torch.float32)
