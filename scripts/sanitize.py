"""Small-N driver over every kernel family of libjp.so, for compute-sanitizer
(SURVEY Sec.4 layer 8):

  compute-sanitizer --tool memcheck  python scripts/sanitize.py
  compute-sanitizer --tool synccheck python scripts/sanitize.py
  compute-sanitizer --tool racecheck python scripts/sanitize.py

Every result is also compared with the oracle, so a run under a tool that
perturbs timing still checks the arithmetic.  Prints one line per case."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
import numpy as np  # noqa: E402
import torch  # noqa: E402

import oracle as O  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402
from helpers import random_loop, region_workload, seq_mixed, to_oracle  # noqa: E402

DEV = "cuda"
fails = 0


def check(name, g, wl, T=True):
    global fails
    _, A, Te = O.run_seq(to_oracle(wl))
    ok = g.A.cpu().numpy().tobytes() == A.tobytes()
    if T and wl.T is not None:
        ok &= g.T.cpu().numpy().tobytes() == Te.tobytes()
    fails += not ok
    print(f"{name}: {'ok' if ok else 'MISMATCH'}", flush=True)


def run(name, wl, fn):
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    fn(L, g)
    torch.cuda.synchronize()
    check(name, g, wl)


# tiny one-CTA schedule, every opcode
for op in (O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2):
    wl = random_loop(op + 1, op, O.F32 if op != O.OP_ADD_C else O.I32, 2000, len_a=4000)
    run(f"tiny op{op}", wl, lambda L, g: jp.jp_schedule(L, jp.workspace(L)))
# profile + mode + run beyond the tiny path (profile, classify, DOALL / privatized / TLS)
for op in (O.OP_ADD_C, O.OP_SAXPY, O.OP_PRIV_TMP, O.OP_STENCIL2):
    wl = random_loop(op + 11, op, O.F32 if op != O.OP_ADD_C else O.I32, 20000, len_a=30000)
    run(f"schedule op{op}", wl, lambda L, g: jp.jp_schedule(L, jp.workspace(L)))
run("config1 d=5%", synth.config1(0.05), lambda L, g: jp.jp_schedule(L, jp.workspace(L)))
wl3 = synth.config3(0.05, n=1 << 16)
for path in (1, 2, 3):
    run(f"tls restart path {path}", wl3,
        lambda L, g, p=path: jp.jp_run_tls(L, window=2048 if p != 1 else 0, w_max=2048, path=p,
                                           prof=jp.jp_profile_density(L, jp.workspace(L)), ws=jp.workspace(L)))
for path in (5, 6):
    def onchip(L, g, p=path):
        ws = jp.workspace(L)
        pr = jp.jp_profile_density(L, ws)
        jp.jp_run_tls(L, window=4096, prof=pr, ws=ws, path=p, recovery=jp.JP_TLS_ONCHIP)
    run(f"tls on-chip path {path}", wl3, onchip)
run("tls serial path 7", random_loop(77, O.OP_STENCIL2, O.F32, 5000, len_a=300),
    lambda L, g: jp.jp_run_tls(L, path=7, ws=jp.workspace(L)))
run("config4 privatized", synth.config4(n=1 << 16),
    lambda L, g: jp.jp_run_privatized(L, jp.jp_profile_density(L, jp.workspace(L)), jp.workspace(L)))
run("config2 doall", synth.config2(n=(1 << 16) + 3), lambda L, g: jp.jp_schedule(L))
run("stealing config5", synth.config5(n=1 << 15),
    lambda L, g: jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=4096))
run("stealing mode C", seq_mixed(3 * 4096),
    lambda L, g: jp.jp_schedule(L, jp.workspace(L), scheme=jp.JP_SCHED_STEALING, chunk_iters=1024))
# spill (two views on one device, one stream each)
wl2 = synth.config2(n=1 << 16)
_, A2, _ = O.run_seq(to_oracle(wl2))
h = (1 << 15)
shards = [synth.config2(n=1 << 16, start=k * h, count=h).to(DEV) for k in range(2)]
views = [jp.Loop.from_workload(s, iter_base=k * h) for k, s in enumerate(shards)]
ctr = torch.zeros(2, dtype=torch.int64, device=DEV)
for k in range(2):
    jp.jp_run_doall_spill(views, k, 1000, ctr, None, 0 if k == 0 else 1)
torch.cuda.synchronize()
ok = all(s.A.cpu().numpy().tobytes() == A2[k * h:(k + 1) * h].tobytes() for k, s in enumerate(shards))
fails += not ok
print(f"spill: {'ok' if ok else 'MISMATCH'}", flush=True)
# device-side stealing of privatized chunks
wt = region_workload(synth.config5(n=1 << 14), 3 << 12, 1 << 14)
g = wt.to(DEV)
L = jp.Loop.from_workload(g)
ws = jp.workspace(L)
off, nb = jp.jp_ws_region(L, "keys_A")
ws[off:off + nb].zero_()
ch = torch.tensor([(s, min(wt.n, s + 512)) for s in range(0, wt.n, 512)], dtype=torch.int64, device=DEV)
jp.jp_run_priv_claim(L, ch, [0, ch.shape[0]], 0, torch.zeros(1, dtype=torch.int64, device=DEV), ws)
jp.jp_priv_finalize(L, ws)
torch.cuda.synchronize()
check("priv claim", g, wt)
# owner exchange kernels
t = torch.from_numpy(np.random.default_rng(3).integers(-1, 50, size=100003).astype(np.int32)).to(DEV)
rows, counts = jp.jp_sparse_pack(t, None, -1, 4)
jp.jp_sparse_reduce_max(t, None, rows)
jp.jp_sparse_gather(t, None, rows)
jp.jp_sparse_scatter(t, None, rows)
torch.cuda.synchronize()
print(f"sparse exchange: ok ({sum(counts)} rows)", flush=True)
print(f"DONE fails={fails}", flush=True)
sys.exit(1 if fails else 0)
