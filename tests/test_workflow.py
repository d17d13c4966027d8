"""Workflows of several loops (PAPER P:L197-200 PDG,
P:L438-460 Alg. 1 over loops, P:L461-469 scheme selection; DESIGN readings
B9, B10).

CPU: jp_plan_workflow (host C) against oracle/sched.workflow_plan on the
paper's three task-stealing shapes (hand-checked batches and AUTO scheme) and
on random overlapping views.  GPU: jp_schedule_workflow under every scheme
ends in the state of the loops executed one after another in program order
(oracle/jpo.c jpo_run_seq chained over shared arrays).
"""
import numpy as np
import pytest
import torch

import oracle as O
import synth
from oracle import sched as OS
import paper_conf_icpp_hanzlw13_b200 as jp


def footprint(wl):
    """Byte ranges a loop touches, restated from the opcode table: index arrays
    and X read; A read (ADD_C, SAXPY, STENCIL2) and written; T written."""
    out = []

    def add(t, n, w):
        if t is not None and n > 0 and wl.n > 0:
            out.append((t.data_ptr(), t.data_ptr() + 4 * n, w))
    for t in (wl.r, wl.r2, wl.w, wl.s):
        add(t, wl.n, False)
    if wl.X is not None:
        add(wl.X, wl.X.numel(), False)
    add(wl.A, wl.A.numel(), True)
    if wl.op == O.OP_PRIV_TMP and wl.T is not None:
        add(wl.T, wl.T.numel(), True)
    return out


def plan_both(loops, scheme):
    got = jp.jp_plan_workflow([jp.Loop.from_workload(wl) for wl in loops], scheme)
    exp = OS.workflow_plan([footprint(wl) for wl in loops], [wl.n for wl in loops], scheme)
    assert got == exp, (got, exp)
    return got


@pytest.mark.parametrize("scheme", [jp.JP_SCHED_SHARING, jp.JP_SCHED_STEALING, jp.JP_SCHED_AUTO])
def test_plan_paper_shapes(scheme):
    # BICG: 2 independent loops x 4 subloops -> one batch of 8; AUTO -> stealing
    p = plan_both(synth.workflow_bicg(n=4096)[0], scheme)
    assert p["n_batches"] == 1 and p["batch"] == [0] * 8
    assert p["scheme"] == (jp.JP_SCHED_STEALING if scheme == jp.JP_SCHED_AUTO else scheme)
    # 2MM: the second loop reads the first's output -> two batches; AUTO -> sharing
    p = plan_both(synth.workflow_2mm(n=4096)[0], scheme)
    assert p["n_batches"] == 2 and p["batch"] == [0, 1] and p["deps"] == [0, 1]
    assert p["scheme"] == (jp.JP_SCHED_SHARING if scheme == jp.JP_SCHED_AUTO else scheme)
    # Crypt: 8 encryption subloops, then 8 decryption subloops reading all of the cipher
    p = plan_both(synth.workflow_crypt(n=4096)[0], scheme)
    assert p["n_batches"] == 2 and p["batch"] == [0] * 8 + [1] * 8
    assert all(p["deps"][8 + k] == 0xFF for k in range(8))
    assert p["scheme"] == (jp.JP_SCHED_STEALING if scheme == jp.JP_SCHED_AUTO else scheme)


def test_plan_random_views():
    g = np.random.default_rng(12)
    base = [torch.zeros(4096, dtype=torch.int32) for _ in range(3)]
    for trial in range(200):
        loops = []
        for u in range(int(g.integers(1, 12))):
            op = int(g.integers(0, 4))

            def view(m):
                b = base[int(g.integers(0, 3))]
                o = int(g.integers(0, 4096 - m))
                return b[o:o + m]
            n = int(g.integers(1, 200))
            A = view(int(g.integers(n, 600)))                     # w is NULL: identity into A
            r = view(n) if g.random() < 0.5 else None
            X = view(int(g.integers(n, 600))) if op in (1, 2) else None
            T = view(int(g.integers(n, 600))) if op == 2 else None   # s is NULL: identity into T
            wl = synth.Workload("v", op, 0, n, A, r=r, w=None, X=X, T=T)
            loops.append(wl)
        plan_both(loops, int(g.integers(0, 3)))


def test_plan_args():
    with pytest.raises(jp.JPError):
        jp.jp_plan_workflow([jp.Loop.from_workload(synth.workflow_2mm(n=64)[0][0])] * 65)
    with pytest.raises(jp.JPError):
        jp.jp_plan_workflow([jp.Loop.from_workload(synth.workflow_2mm(n=64)[0][0])], 7)


# ---------------------------------------------------------------------------
# GPU: execution
# ---------------------------------------------------------------------------
def run_program_order(loops, arrays):
    """The oracle: every loop's jpo_run_seq in program order over host copies
    of the shared base arrays (a loop's tensors are views into them)."""
    host = {b.data_ptr(): b.cpu().numpy().copy() for b in arrays}

    def find(t):
        for b in arrays:
            if b.data_ptr() <= t.data_ptr() < b.data_ptr() + 4 * b.numel():
                o = (t.data_ptr() - b.data_ptr()) // 4
                return host[b.data_ptr()], o
        raise AssertionError("tensor outside the workflow's arrays")

    def np_of(t):
        if t is None:
            return None
        a, o = find(t)
        return a[o:o + t.numel()]
    for wl in loops:
        ref = O.Loop(wl.op, wl.dtype, wl.n, np_of(wl.A), r=np_of(wl.r), r2=np_of(wl.r2), w=np_of(wl.w),
                     s=np_of(wl.s), X=np_of(wl.X), T=np_of(wl.T), c0=wl.c0, c1=wl.c1)
        st, A, T = O.run_seq(ref)
        assert st == O.OK
        np_of(wl.A)[:] = A
        if T is not None:
            np_of(wl.T)[:] = T
    return host


@pytest.mark.gpu
@pytest.mark.parametrize("shape", ["bicg", "2mm", "crypt"])
@pytest.mark.parametrize("scheme", [jp.JP_SCHED_SHARING, jp.JP_SCHED_STEALING, jp.JP_SCHED_AUTO])
def test_workflow_runs_in_program_order(shape, scheme):
    fn = {"bicg": synth.workflow_bicg, "2mm": synth.workflow_2mm, "crypt": synth.workflow_crypt}[shape]
    loops, arrays = fn(n=(1 << 16) + 40, device="cuda")
    exp = run_program_order(loops, arrays)
    L = [jp.Loop.from_workload(wl) for wl in loops]
    wss = [jp.workspace(lp) for lp in L]
    res, plan = jp.jp_schedule_workflow(L, wss, scheme=scheme)
    torch.cuda.synchronize()
    for b in arrays:
        assert b.cpu().numpy().tobytes() == exp[b.data_ptr()].tobytes(), shape
    assert plan["n_batches"] == {"bicg": 1, "2mm": 2, "crypt": 2}[shape]
    assert all(r["mode"] == jp.JP_MODE_DOALL for r in res)


@pytest.mark.gpu
def test_workflow_mixed_modes():
    """A workflow whose loops take different Fig. 2(b) modes (TLS, privatized,
    DOALL), with a dependence between the first and the last."""
    a = synth.config3(0.05, n=1 << 15, device="cuda")
    b = synth.config4(n=1 << 15, device="cuda")
    y = torch.zeros(1 << 15, dtype=torch.int32, device="cuda")
    c = synth.Workload("reader", O.OP_SAXPY, O.I32, 1 << 15, y, X=a.A, c0=3)   # reads loop a's output
    loops, arrays = [a, b, c], [a.A, a.r, a.w, b.A, b.X, b.s, b.T, y]
    exp = run_program_order(loops, arrays)
    L = [jp.Loop.from_workload(wl) for wl in loops]
    res, plan = jp.jp_schedule_workflow(L, [jp.workspace(lp) for lp in L], scheme=jp.JP_SCHED_STEALING)
    torch.cuda.synchronize()
    assert plan["batch"] == [0, 0, 1]
    assert [r["mode"] for r in res] == [jp.JP_MODE_TLS, jp.JP_MODE_PRIVATIZED, jp.JP_MODE_DOALL]
    for t in arrays:
        assert t.cpu().numpy().tobytes() == exp[t.data_ptr()].tobytes()
