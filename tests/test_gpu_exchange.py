"""Owner-partitioned sparse exchange: jp_sparse_pack /
reduce_max / gather / scatter on the GPU against their plain definitions
(include/jp.h), and the two-rank owner-form schedule against the oracle.

The definitions are restated here in numpy: pack = the addresses in [lo, hi)
where a table is not empty, ascending, with the tables' values; the per-owner
counts use owner(a) = a // ceil(len / world).  Integer work: bit-exact."""
import numpy as np
import pytest
import torch

import paper_conf_icpp_hanzlw13_b200 as jp
from paper_conf_icpp_hanzlw13_b200 import _abi

pytestmark = pytest.mark.gpu
DEV = "cuda"


def _tables(seed, n, elem, ntab, fill):
    g = np.random.default_rng(seed)
    dt, empty = (np.int32, -1) if elem == 4 else (np.int64, 0)
    hi = 0x7FFFFFF0 if elem == 4 else (1 << 62)
    out = []
    for _ in range(ntab):
        v = g.integers(0, hi, size=n, dtype=np.int64).astype(dt)
        v[g.random(n) >= fill] = empty
        out.append(v)
    return out, empty


def _pack_def(tabs, empty, world, lo, hi):
    n = len(tabs[0])
    a = np.arange(lo, hi, dtype=np.int64)
    full = np.zeros(hi - lo, dtype=bool)
    for t in tabs:
        full |= t[lo:hi] != empty
    a = a[full]
    rows = np.stack([a.astype(tabs[0].dtype)] + [t[a] for t in tabs], axis=1)
    sl = max(-(-n // world), 1)
    return rows, [int(np.count_nonzero(a // sl == k)) for k in range(world)]


@pytest.mark.parametrize("elem", [4, 8])
@pytest.mark.parametrize("ntab", [1, 2])
@pytest.mark.parametrize("n,world,fill", [(1, 1, 1.0), (4095, 2, 0.3), (4096, 8, 0.01), (4097, 3, 1.0),
                                          (100003, 8, 0.2), (100003, 5, 0.0), ((1 << 20) + 3, 8, 0.05),
                                          (7, 8, 0.5), ((1 << 22) + 1, 3, 0.7)])
def test_pack_matches_definition(elem, ntab, n, world, fill):
    tabs, empty = _tables(n * 7 + elem + ntab, n, elem, ntab, fill)
    d = [torch.from_numpy(t).to(DEV) for t in tabs]
    rows, counts = jp.jp_sparse_pack(d[0], d[1] if ntab == 2 else None, empty, world)
    exp, ecounts = _pack_def(tabs, empty, world, 0, n)
    assert counts == ecounts
    assert rows.shape == exp.shape and np.array_equal(rows.cpu().numpy(), exp)


@pytest.mark.parametrize("elem", [4, 8])
@pytest.mark.parametrize("lo,hi", [(0, 0), (5, 9), (4095, 8193), (12345, 100003), (0, 100003)])
def test_pack_subrange(elem, lo, hi):
    n = 100003
    tabs, empty = _tables(lo + hi + elem, n, elem, 1, 0.4)
    rows, counts = jp.jp_sparse_pack(torch.from_numpy(tabs[0]).to(DEV), None, empty, 1, lo, hi)
    exp, ecounts = _pack_def(tabs, empty, 1, lo, hi)
    assert counts == ecounts and np.array_equal(rows.cpu().numpy().reshape(exp.shape), exp)


def test_pack_capacity_error():
    t = torch.zeros(1000, dtype=torch.int32, device=DEV)
    lib = _abi.lib()
    scratch = torch.empty(jp.jp_sparse_scratch_bytes(1000, 2) // 8 + 1, dtype=torch.int64, device=DEV)
    rows = torch.empty((10, 2), dtype=torch.int32, device=DEV)
    import ctypes as C
    cnt = (C.c_int64 * 2)()
    st = lib.jp_sparse_pack(t.data_ptr(), None, 4, 1000, 0, 1000, -1, 2, rows.data_ptr(), 10, cnt,
                            scratch.data_ptr(), scratch.numel() * 8, torch.cuda.current_stream().cuda_stream)
    assert st == _abi.JP_ERR_ARG and list(cnt) == [500, 500]


@pytest.mark.parametrize("elem", [4, 8])
@pytest.mark.parametrize("ntab", [1, 2])
def test_rows_reduce_gather_scatter(elem, ntab):
    n, m = 50021, 200000
    g = np.random.default_rng(elem * 10 + ntab)
    tabs, empty = _tables(elem + ntab, n, elem, ntab, 0.5)
    dt = tabs[0].dtype
    addr = g.integers(-3, n + 3, size=m)           # a few out-of-range rows (ignored)
    vals = [g.integers(0, 0x7FFFFFF0 if elem == 4 else 1 << 62, size=m).astype(dt) for _ in range(ntab)]
    rows = np.stack([addr.astype(dt)] + vals, axis=1)
    ok = (addr >= 0) & (addr < n)
    d = [torch.from_numpy(t.copy()).to(DEV) for t in tabs]
    t1 = d[1] if ntab == 2 else None
    R = torch.from_numpy(rows).to(DEV)
    jp.jp_sparse_reduce_max(d[0], t1, R)
    exp = [t.copy() for t in tabs]
    for q in range(ntab):
        np.maximum.at(exp[q], addr[ok], vals[q][ok])
        assert np.array_equal(d[q].cpu().numpy(), exp[q])
    jp.jp_sparse_gather(d[0], t1, R)
    got = R.cpu().numpy()
    for q in range(ntab):
        assert np.array_equal(got[ok, 1 + q], exp[q][addr[ok]])
        assert np.array_equal(got[~ok, 1 + q], vals[q][~ok])
    # scatter distinct addresses
    ua = g.permutation(n)[:n // 3]
    srows = np.stack([ua.astype(dt)] + [np.full(len(ua), 17 + q, dtype=dt) for q in range(ntab)], axis=1)
    srows = np.concatenate([srows, np.full((5, 1 + ntab), -1, dtype=dt)])   # padding rows
    jp.jp_sparse_scatter(d[0], t1, torch.from_numpy(srows).to(DEV))
    for q in range(ntab):
        exp[q][ua] = 17 + q
        assert np.array_equal(d[q].cpu().numpy(), exp[q])


def test_owner_roundtrip_equals_dense_allreduce():
    """The owner form's data movement, simulated for 4 ranks inside one process
    with the real kernels: every rank ends with the dense MAX at each touched
    address (C1o), and with the dense MAX everywhere it is non-empty (C4o)."""
    world, n = 4, 300007
    g = np.random.default_rng(5)
    W, R = [], []
    for k in range(world):
        tabs, _ = _tables(100 + k, n, 4, 2, 0.05 + 0.05 * k)
        W.append(torch.from_numpy(tabs[0]).to(DEV))
        R.append(torch.from_numpy(tabs[1]).to(DEV))
    dense_w = torch.stack(W).amax(0)
    dense_r = torch.stack(R).amax(0)
    packs = [jp.jp_sparse_pack(W[k], R[k], -1, world) for k in range(world)]
    # all_to_all: split each rank's rows by owner counts
    send = [list(torch.split(p[0], p[1])) for p in packs]
    recv = [torch.cat([send[src][dst] for src in range(world)]) for dst in range(world)]
    for k in range(world):
        jp.jp_sparse_reduce_max(W[k], R[k], recv[k])
        jp.jp_sparse_gather(W[k], R[k], recv[k])
    back_parts = [list(torch.split(recv[dst], [packs[src][1][dst] for src in range(world)])) for dst in range(world)]
    for k in range(world):
        before = (packs[k][0][:, 0]).long()
        jp.jp_sparse_scatter(W[k], R[k], torch.cat([back_parts[dst][k] for dst in range(world)]))
        assert torch.equal(W[k][before], dense_w[before]) and torch.equal(R[k][before], dense_r[before])
    del g
