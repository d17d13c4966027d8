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
ap.add_argument("what", choices=["doall", "priv", "tls", "profile", "all"])
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
print("done", jp.jp_launch_count())
