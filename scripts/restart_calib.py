#!/usr/bin/env python
"""Restart-TLS (reading A6) cost calibration on one B200: time per window of
each path (1 single CTA, 3 16-CTA cluster, 2 cooperative grid) at fixed
windows on dependence-free loops (windows = ceil(n / W) exactly), with and
without the WAW commit; then the adaptive policy under several caps on the
config-3 sensitivity loops (delta = 2^20).  One JSON object per line.

  python scripts/restart_calib.py [--n LOG2N]
"""
import argparse
import json
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402


def timed(fn, A, A0, st, reps=3):
    ts, out = [], None
    for k in range(reps + 1):
        A.copy_(A0)
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        out = fn()
        b.record(st)
        torch.cuda.synchronize()
        if k:
            ts.append(a.elapsed_time(b))
    return out, statistics.median(ts)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=22)
    ap.add_argument("--skip-fixed", action="store_true")
    ap.add_argument("--schedule-only", action="store_true")
    args = ap.parse_args()
    st = torch.cuda.current_stream()
    dev = torch.device("cuda:0")
    n = 1 << args.n
    if not args.skip_fixed:
        for name, wl in (("nowaw", synth.config3(0.0, n=n, device=dev)), ("waw", synth.config3_waw(0.0, n=n, device=dev))):
            A0 = wl.A.clone()
            L = jp.Loop.from_workload(wl)
            ws = jp.workspace(L)
            prof = jp.jp_profile_density(L, ws)
            grid = [(1, W) for W in (64, 128, 256, 512, 1024, 2048, 4096)] + \
                   [(3, W) for W in (1024, 2048, 4096, 8192, 16384, 32768, 65536)] + \
                   [(2, W) for W in (4096, 16384, 65536, 262144, 1 << 20)]
            for path, W in grid:
                try:
                    s, ms = timed(lambda: jp.jp_run_tls(L, window=W, path=path, prof=prof, ws=ws, stream=st), wl.A, A0, st)
                except jp.JPError as e:
                    print(json.dumps({"loop": name, "path": path, "W": W, "error": str(e)}), flush=True)
                    continue
                print(json.dumps({"loop": name, "path": path, "W": W, "windows": s["windows"], "ms": ms,
                                  "us_per_window": ms * 1e3 / s["windows"]}), flush=True)
            del wl, L, ws, A0
            torch.cuda.empty_cache()
    for maker, tag in ((synth.config3, "config3"), (synth.config3_waw, "config3_waw")):
        for delta in (1024, 1 << 20):
            for d in (0.01, 0.10):
                wl = maker(d, n=n, delta=delta, device=dev)
                A0 = wl.A.clone()
                L = jp.Loop.from_workload(wl)
                ws = jp.workspace(L)
                prof = jp.jp_profile_density(L, ws)
                for rec in (1, 0):
                    res, ms = timed(lambda: jp.jp_schedule(L, ws, stream=st, tls_recovery=rec), wl.A, A0, st, reps=1)
                    print(json.dumps({"loop": tag, "d": d, "delta": delta, "schedule": rec, "ms": ms,
                                      "G_committed_per_s": n / ms / 1e6, "mode": res["mode_name"],
                                      "path": res["tls_path"], "w_max": res["tls_w_max"],
                                      "recovery": res["tls_recovery"], "windows": res["tls"]["windows"],
                                      "violations": res["tls"]["violations"]}), flush=True)
                if args.schedule_only:
                    continue
                for path, wm in ((1, 256), (1, 1024), (1, 4096), (3, 4096), (3, 16384), (3, 65536), (2, 65536),
                                 (2, 262144)):
                    try:
                        s, ms = timed(lambda: jp.jp_run_tls(L, window=0, w_max=wm, path=path, prof=prof, ws=ws,
                                                            stream=st), wl.A, A0, st, reps=1)
                    except jp.JPError as e:
                        print(json.dumps({"loop": tag, "d": d, "delta": delta, "path": path, "w_max": wm,
                                          "error": str(e)}), flush=True)
                        continue
                    print(json.dumps({"loop": tag, "d": d, "delta": delta, "path": path, "w_max": wm, "ms": ms,
                                      "G_committed_per_s": n / ms / 1e6, "windows": s["windows"],
                                      "violations": s["violations"], "us_per_window": ms * 1e3 / s["windows"]}),
                          flush=True)
                del wl, L, ws, A0
                torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
