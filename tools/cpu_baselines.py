#!/usr/bin/env python
"""Bounded CPU baselines of the oracle (test infrastructure: CPU-Seq / CPU-Base,
one thread, fp64) for the BASELINE configs the default bench line does not
cover (SURVEY 8(d) "Oracle timing"):

    python tools/cpu_baselines.py tiny|orkut|twitter [--out FILE.jsonl] [--cap-s 1800]

tiny    : all 50 slides in CPU-Seq mode and in CPU-Base mode (a push after
          every single update), same stream and source as the bench.
orkut   : init (create + static push, timed) and then one slide per batch size
          k = 10^2 .. 10^6 (ceil(k/4) newest insertions + floor(3k/4) oldest
          deletions, undirected), applied one after another on the same oracle.
twitter : create + static push and one 10^5 + 10^5 slide, in a child process
          killed at --cap-s; a run that does not finish reports how far it got.
"""
from __future__ import annotations

import argparse
import json
import multiprocessing as mp
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def cpu_model():
    try:
        for line in open("/proc/cpuinfo"):
            if line.startswith("model name"):
                return line.split(":", 1)[1].strip(), os.cpu_count()
    except Exception:
        pass
    return "", os.cpu_count()


def run_tiny():
    import oracle
    from paper_journals_pvldb_guolst17_b200 import workload as W
    res = {}
    for mode, name in ((oracle.SEQ, "CPU-Seq"), (oracle.BASE, "CPU-Base")):
        st, cfg = W.make_stream("tiny")
        g0s, g0d = st.window()
        srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
        o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, cfg["eps"])
        t0 = time.perf_counter()
        o.push(oracle.SEQ)
        t_static = time.perf_counter() - t0
        per = []
        for _ in range(cfg["slides"]):
            b = st.next_batch()
            t0 = time.perf_counter()
            o.apply(*b, mode=mode)
            per.append(time.perf_counter() - t0)
        upd = cfg["ins"] + cfg["dele"]
        res[name] = {"edge_updates_per_s": upd * len(per) / sum(per), "ms_per_batch": 1e3 * np.mean(per),
                     "slides": len(per), "static_push_s": t_static}
    return {"workload": "tiny", "results": res}


def run_orkut():
    import oracle
    from paper_journals_pvldb_guolst17_b200 import workload as W
    st, cfg = W.make_stream("orkut")
    e0s, e0d = st.src[st.lo:st.hi].copy(), st.dst[st.lo:st.hi].copy()
    arcs = W.expand_undirected(e0s, e0d)
    srcs = W.pick_sources(cfg["n"], arcs[0], arcs[1], cfg["band"], 1)
    t0 = time.perf_counter()
    o = oracle.Oracle(cfg["n"], arcs[0], arcs[1], srcs, 0.15, cfg["eps"])
    t_build = time.perf_counter() - t0
    t0 = time.perf_counter()
    o.push(oracle.SEQ)
    t_static = time.perf_counter() - t0
    static_edges = o.stats(reset=True)["pushed_edges"]
    res = {}
    for k in (100, 1000, 10_000, 100_000, 1_000_000):
        ni, nd = (k + 3) // 4, 3 * k // 4
        i0, d0 = st.hi, st.lo
        ins = W.expand_undirected(st.src[i0:i0 + ni], st.dst[i0:i0 + ni])
        dels = W.expand_undirected(st.src[d0:d0 + nd], st.dst[d0:d0 + nd])
        st.hi, st.lo = i0 + ni, d0 + nd
        t0 = time.perf_counter()
        o.apply(ins[0], ins[1], dels[0], dels[1], mode=oracle.SEQ)
        dt = time.perf_counter() - t0
        s = o.stats(reset=True)
        res[f"k={k}"] = {"edge_updates_per_s": k / dt, "ms_per_batch": 1e3 * dt,
                         "pushed_edges": s["pushed_edges"]}
        print(k, res[f"k={k}"], flush=True)
    return {"workload": "orkut", "build_s": t_build, "static_push_s": t_static,
            "static_push_pushed_edges": static_edges, "results": res,
            "sample": "one oracle: init, then one slide per k in increasing k (the window moves by "
                      "the earlier slides' few thousand edges between k values)"}


def _twitter_child(q):
    import oracle
    from paper_journals_pvldb_guolst17_b200 import workload as W
    t0 = time.perf_counter()
    st, cfg = W.make_stream("twitter")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    q.put(("generated", time.perf_counter() - t0))
    t0 = time.perf_counter()
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, cfg["eps"])
    q.put(("built", time.perf_counter() - t0))
    t0 = time.perf_counter()
    o.push(oracle.SEQ)
    q.put(("static_push", time.perf_counter() - t0, o.stats(reset=True)))
    b = st.next_batch()
    t0 = time.perf_counter()
    o.apply(*b, mode=oracle.SEQ)
    q.put(("slide", time.perf_counter() - t0, o.stats(reset=True)))


def run_twitter(cap_s):
    ctx = mp.get_context("fork")
    q = ctx.Queue()
    p = ctx.Process(target=_twitter_child, args=(q,))
    t_start = time.perf_counter()
    p.start()
    got = {}
    while time.perf_counter() - t_start < cap_s:
        try:
            item = q.get(timeout=5)
        except Exception:
            if not p.is_alive():
                break
            continue
        got[item[0]] = item[1:]
        print(item, flush=True)
        if item[0] == "slide":
            break
    finished = "slide" in got
    if p.is_alive():
        p.kill()
    p.join()
    rec = {"workload": "twitter", "cap_s": cap_s, "finished": finished,
           "stages_s": {k: v[0] for k, v in got.items()}}
    if "static_push" in got:
        rec["static_push_pushed_edges"] = got["static_push"][1]["pushed_edges"]
    if finished:
        rec["results"] = {"edge_updates_per_s": 200_000 / got["slide"][0], "ms_per_batch": 1e3 * got["slide"][0],
                          "pushed_edges": got["slide"][1]["pushed_edges"]}
    else:
        rec["note"] = f"stopped at the {cap_s:.0f} s cap after stages {sorted(got)}"
    return rec


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("workload", choices=["tiny", "orkut", "twitter"])
    ap.add_argument("--out", default=None)
    ap.add_argument("--cap-s", type=float, default=1800.0)
    a = ap.parse_args()
    rec = {"tiny": run_tiny, "orkut": run_orkut}.get(a.workload, lambda: run_twitter(a.cap_s))()
    model, ncpu = cpu_model()
    rec.update({"kind": "oracle", "cores": 1, "host": f"1 thread of {ncpu}-core {model}"})
    print(json.dumps(rec), flush=True)
    if a.out:
        with open(a.out, "a") as f:
            f.write(json.dumps(rec) + "\n")


if __name__ == "__main__":
    main()
