#!/usr/bin/env python
"""Config-3 whole jp_schedule call (median of 20, CUDA events) at several densities;
JP_PROFILE_BUCKETS=0 selects the stamp/classify profile instead of address buckets."""
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
for d in (0.001, 0.01, 0.05, 0.10):
    wl = synth.config3(d, device="cuda")
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    res, ms = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st), wl.A, A0, st, 20)
    _, msp = bench.median_timed(lambda: jp.jp_profile_density(L, ws, stream=st), None, None, st, 20)
    print(json.dumps({"d": d, "buckets": os.environ.get("JP_PROFILE_BUCKETS", "1"), "schedule_ms": round(ms, 4),
                      "G_per_s": round(wl.n / ms / 1e6, 2), "profile_density_ms": round(msp, 4),
                      "windows": res["tls"]["windows"]}), flush=True)
    del wl, A0, L, ws
