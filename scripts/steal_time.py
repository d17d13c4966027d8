#!/usr/bin/env python
"""Config 5 through dist.schedule_stealing at one rank, the multi-rank path forced
(force_ranks): profile='replicated' vs 'partitioned', wall clock median of 10,
plus the phases of one call."""
import os
import statistics
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import paper_conf_icpp_hanzlw13_b200.dist as jd  # noqa: E402
import synth  # noqa: E402

wl = synth.config5(device="cuda")
A0 = wl.A.clone()
full = jp.Loop.from_workload(wl)
ws = jp.workspace(full)
for prof in ("replicated", "partitioned"):
    ts = []
    for k in range(12):
        wl.A.copy_(A0)
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        jd.schedule_stealing(full, ws, chunk_iters=65536, force_ranks=True, profile=prof)
        torch.cuda.synchronize()
        if k >= 2:
            ts.append(time.perf_counter() - t0)
    wl.A.copy_(A0)
    ph = jd.schedule_stealing(full, ws, chunk_iters=65536, force_ranks=True, profile=prof, timings=True)["phases"]
    print(prof, "ms", round(statistics.median(ts) * 1e3, 3), {k: round(v, 3) if isinstance(v, float) else v
                                                             for k, v in ph.items()}, flush=True)
