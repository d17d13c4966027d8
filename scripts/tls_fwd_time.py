"""Time TLS with on-chip recovery (reading B7) on config 3 (N = 2^24) per density:
jp_run_tls kernel time (CUDA events), guided and unguided, and the whole
jp_schedule call.  Usage: python scripts/tls_fwd_time.py [--n N] [--windows W,...]"""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402


def ev_ms(fn, st, reps=3):
    out = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        fn(pre=True)
        torch.cuda.synchronize()
        a.record(st)
        r = fn(pre=False)
        b.record(st)
        torch.cuda.synchronize()
        out.append((a.elapsed_time(b), r))
    return min(out, key=lambda x: x[0])


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=1 << 24)
    ap.add_argument("--windows", default="0")
    ap.add_argument("--clusters", default="0")
    a = ap.parse_args()
    dev = torch.device("cuda:0")
    st = torch.cuda.current_stream()
    for d in (0.001, 0.01, 0.05, 0.10):
        wl = synth.config3(d, n=a.n, device=dev)
        A0 = wl.A.clone()
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        prof = jp.jp_profile_density(L, ws)
        jp.jp_tls_guide(L, ws)
        row = {"d": d}
        for W in (int(x) for x in a.windows.split(",")):
            for C in (int(x) for x in a.clusters.split(",")):
                for guided in (False, True):
                    def run(pre):
                        wl.A.copy_(A0)
                        if pre:
                            return None
                        return jp.jp_run_tls(L, window=W, cluster=C, prof=prof, ws=ws, guided=guided,
                                             recovery=jp.JP_TLS_ONCHIP, stream=st)
                    ms, s = ev_ms(run, st)
                    row[f"W{W}_C{C}_{'g' if guided else 'u'}"] = {"ms": round(ms, 3), "Miter_s": round(a.n / ms / 1e3, 1),
                                                                   "windows": s["windows"], "viol": s["violations"],
                                                                   "us_per_window": round(ms * 1e3 / s["windows"], 2)}

        def sched(pre):
            wl.A.copy_(A0)
            return None if pre else jp.jp_schedule(L, ws, stream=st)
        ms, r = ev_ms(sched, st)
        row["schedule"] = {"ms": round(ms, 3), "Miter_s": round(a.n / ms / 1e3, 1), "path": r["tls_path"],
                           "guided": r["tls_guided"], "W": r["tls_w_max"]}
        print(json.dumps(row), flush=True)


if __name__ == "__main__":
    main()


def doall_floor():
    """The same body and index shape with no dependence (config 3 at d = 0) run as
    DOALL: the random gather + scatter floor the TLS path is measured against."""
    dev = torch.device("cuda:0")
    st = torch.cuda.current_stream()
    wl = synth.config3(0.0, device=dev)
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    prof = jp.jp_profile_density(L, ws)
    ms, _ = ev_ms(lambda pre: None if pre else jp.jp_run_doall(L, prof, ws, stream=st), st, reps=5)
    print(json.dumps({"doall_indirect_d0": {"ms": round(ms, 3), "Giter_s": round(wl.n / ms / 1e6, 2)}}), flush=True)


if __name__ == "__main__" and os.environ.get("DOALL_FLOOR"):
    doall_floor()
