"""Indirect DOALL (config 3 shape at d = 0: A[w[i]] = A[r[i]] + c, r = w a
permutation, N = 2^24): the quad kernel vs the one-iteration-per-thread kernel
(JP_DOALL_GENERIC=1), CUDA events, median of 10."""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

wl = synth.config3(0.0, device="cuda")
L = jp.Loop.from_workload(wl)
prof = {"n": wl.n, "raw_iters": 0, "war_iters": 0, "waw_iters": 0, "first_raw_iter": -1,
        "d_raw": 0.0, "d_war": 0.0, "d_waw": 0.0}
ts = []
for _ in range(12):
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    jp.jp_run_doall(L, prof)
    b.record()
    torch.cuda.synchronize()
    ts.append(a.elapsed_time(b))
ms = statistics.median(ts[2:])
print({"kernel": "generic" if os.environ.get("JP_DOALL_GENERIC") else "quad", "ms": round(ms, 4),
       "G_iter_per_s": round(wl.n / (ms * 1e-3) / 1e9, 2)})
