#!/usr/bin/env python
"""Indirect DOALL through jp_schedule (config 3's shape at d = 0, N = 2^24) and
config 5 (STEALING), median of 20 whole calls; run with JP_DOALL_PHASED=0 / 1."""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import bench  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

st = torch.cuda.current_stream()
ph = os.environ.get("JP_DOALL_PHASED", "1")
for name, wl, kw in (("config3_d0", synth.config3(0.0, device="cuda"), {}),
                     ("config5", synth.config5(device="cuda"), {"scheme": jp.JP_SCHED_STEALING, "chunk_iters": 1 << 16})):
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    res, ms = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st, **kw), wl.A, A0, st, 20)
    print(json.dumps({"loop": name, "phased": ph, "mode": res["mode_name"], "ms": round(ms, 4),
                      "G_per_s": round(wl.n / ms / 1e6, 2)}), flush=True)
    del wl, A0, L, ws
