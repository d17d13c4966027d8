#!/usr/bin/env python
"""Config-3 whole jp_schedule (d = 1%) under option variants (median of 20, CUDA events):
what the host-side steps of the call cost around the kernels."""
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
wl = synth.config3(0.01, device="cuda")
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
for name, kw in (("default", {}), ("static_check=1", {"static_check": 1})):
    res, ms = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st, **kw), wl.A, A0, st, 20)
    print(json.dumps({"variant": name, "ms": round(ms, 4), "path": res["tls_path"]}), flush=True)
# an empty-ish launch pair for the event floor
_, ms0 = bench.median_timed(lambda: None, None, None, st, 20)
print(json.dumps({"variant": "events only", "ms": round(ms0, 4)}))
