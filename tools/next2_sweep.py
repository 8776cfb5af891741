#!/usr/bin/env python
"""NEXT-2: the epsilon sweep and the source-degree sweep of the
paper's Figs 6-7 on B200, for the LJ and Twitter shapes.

    python tools/next2_sweep.py --workload lj|twitter [--sources 8] [--slides 5]
                                [--eps 1e-4,...,1e-10] [--bands 10,1000,1000000]
                                [--band-eps 1e-9] [--out FILE.jsonl]

One stream per run (generated once).  For every point -- (eps, top-1K band)
for each eps, and (band-eps, band) for each band -- `--sources` sources are
drawn uniformly from the band (seed 7); each gets its own single-source handle
in the bench's launch configuration (Opt mode), the same warm-up slide and the
same `--slides` timed slides (device-resident batches, L2 flushed between
slides, CUDA events on the library's stream).  Per point it prints mean and
spread (min / max over sources) of ms per batch, pushed edges per batch and
edge updates/s.  Output: one JSON line per point.
"""
from __future__ import annotations

import argparse
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def parse():
    p = argparse.ArgumentParser()
    p.add_argument("--workload", default="lj")
    p.add_argument("--sources", type=int, default=8)
    p.add_argument("--slides", type=int, default=5)
    p.add_argument("--warmup", type=int, default=1)
    p.add_argument("--eps", default="1e-4,1e-5,1e-6,1e-7,1e-8,1e-9,1e-10")
    p.add_argument("--bands", default="10,1000,1000000")
    p.add_argument("--band-eps", type=float, default=1e-9)
    p.add_argument("--out", default=None)
    return p.parse_args()


def main():
    args = parse()
    import torch

    from paper_journals_pvldb_guolst17_b200 import dist as D, ppr, workload as W

    dev = torch.device("cuda", 0)
    stream = torch.cuda.Stream(dev)
    torch.cuda.set_stream(stream)
    t0 = time.perf_counter()
    st, cfg = W.make_stream(args.workload)
    g0s, g0d = st.window()
    nsl = args.warmup + args.slides
    batches = [st.next_batch() for _ in range(nsl)]
    counts = (cfg["ins"], cfg["dele"])
    dev_b = [D.pack_batch(*b)[0].to(dev) for b in batches]
    flush_buf = torch.empty(512 * 1024 * 1024 // 4, dtype=torch.int32, device=dev)
    t_gen = time.perf_counter() - t0
    out = open(args.out, "a") if args.out else None

    points = [(float(e), 1000) for e in args.eps.split(",")]
    points += [(args.band_eps, int(b)) for b in args.bands.split(",") if int(b) != 1000]
    for eps, band in points:
        srcs = W.pick_sources(cfg["n"], g0s, g0d, band, args.sources, seed=7)
        per = []
        for s in srcs:
            h = ppr.Ppr(cfg["n"], g0s, g0d, [s], alpha=0.15, eps=eps, mode="opt",
                        stream=stream.cuda_stream)
            cs = h.create_stats
            for b in dev_b[:args.warmup]:
                h.apply_batch(*D.unpack_batch(b, counts), mem=ppr.MEM_DEVICE)
            ms, edges, pushes = [], [], []
            for b in dev_b[args.warmup:]:
                ppr.reset_persisting_l2()
                flush_buf.fill_(1)
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(stream)
                r = h.apply_batch(*D.unpack_batch(b, counts), mem=ppr.MEM_DEVICE)
                e1.record(stream)
                e1.synchronize()
                ms.append(e0.elapsed_time(e1))
                edges.append(r["pushed_edges"])
                pushes.append(r["pushes"])
            P, R = h.query(0)
            assert np.all(np.abs(R) <= eps), "eps-termination violated"
            h.close()
            per.append({"source": int(s), "ms": float(np.mean(ms)), "pushed_edges": float(np.mean(edges)),
                        "pushes": float(np.mean(pushes)), "create_ms": cs["ms_total"],
                        "create_pushed_edges": cs["pushed_edges"]})
        ms = np.array([x["ms"] for x in per])
        ed = np.array([x["pushed_edges"] for x in per])
        upd = (cfg["ins"] + cfg["dele"]) / (ms / 1e3)
        rec = {"workload": args.workload, "eps": eps, "band": f"top-{band}", "sources": len(per),
               "slides": args.slides,
               "ms_per_batch": {"mean": float(ms.mean()), "min": float(ms.min()), "max": float(ms.max())},
               "pushed_edges_per_batch": {"mean": float(ed.mean()), "min": float(ed.min()),
                                          "max": float(ed.max())},
               "edge_updates_per_s": {"mean": float(upd.mean()), "min": float(upd.min()),
                                      "max": float(upd.max())},
               "static_ms": {"mean": float(np.mean([x["create_ms"] for x in per]))},
               "per_source": per, "generate_s": t_gen}
        print(json.dumps({k: rec[k] for k in ("workload", "eps", "band", "ms_per_batch",
                                                "pushed_edges_per_batch")}), flush=True)
        if out:
            out.write(json.dumps(rec) + "\n")
            out.flush()


if __name__ == "__main__":
    main()
