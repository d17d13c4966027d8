"""Single-GPU driver for ncu captures: runs each hot kernel a few times on the
BASELINE-size workloads (never used for timing numbers)."""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("what", choices=["doall", "priv", "tls", "profile", "all", "spill", "exchange"])
ap.add_argument("--reps", type=int, default=3)
a = ap.parse_args()
dev = torch.device("cuda:0")
if a.what in ("doall", "all"):
    wl = synth.config2(device=dev)
    L = jp.Loop.from_workload(wl)
    for _ in range(a.reps):
        jp.jp_schedule(L)
    torch.cuda.synchronize()
    del wl, L
if a.what in ("priv", "profile", "all"):
    wl = synth.config4(device=dev)
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    for _ in range(a.reps):
        p = jp.jp_profile_density(L, ws)
        jp.jp_run_privatized(L, p, ws)
    torch.cuda.synchronize()
    del wl, L, ws
if a.what in ("tls", "profile", "all"):
    wl = synth.config3(0.01, device=dev)
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    for _ in range(a.reps):
        p = jp.jp_profile_density(L, ws)
    jp.jp_tls_guide(L, ws)
    jp.jp_run_tls(L, window=4096, w_max=4096, path=3, prof=p, ws=ws, guided=True)   # k_tls_cluster
    jp.jp_run_tls(L, window=0, w_max=4096, prof=p, ws=ws)                            # k_tls_cta (adaptive)
    torch.cuda.synchronize()
if a.what == "spill":   # k_doall_spill on config 2, one rank
    wl = synth.config2(device=dev)
    L = jp.Loop.from_workload(wl)
    ctr = torch.zeros(1, dtype=torch.int64, device=dev)
    for _ in range(a.reps):
        ctr.zero_()
        jp.jp_run_doall_spill([L], 0, 1 << 16, ctr)
    torch.cuda.synchronize()
    del wl, L
if a.what == "exchange":   # owner-exchange kernels on config 3 (d = 1%), rank 0 of 8
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    wl = synth.config3(0.01, device=dev)
    full = jp.Loop.from_workload(wl)
    b, e = jd.sharing_ranges(wl.n, 8)[0]
    L = full.range(b, e)
    ws = jp.workspace(L)
    jp.jp_profile_stamp(L, ws)
    W = jd._region(ws, L, "minW_A", torch.int32, jp)
    R = jd._region(ws, L, "minR_A", torch.int32, jp)
    for _ in range(a.reps):
        rows, counts = jp.jp_sparse_pack(W, R, -1, 8)
        jp.jp_sparse_reduce_max(W, R, rows)
        jp.jp_sparse_gather(W, R, rows)
        jp.jp_sparse_scatter(W, R, rows)
    torch.cuda.synchronize()
print("done", jp.jp_launch_count())
