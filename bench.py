#!/usr/bin/env python
"""Benchmark: batch-parallel PPR maintenance on a sliding-window edge stream.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--workload lj]
                    [--impl ours|reference] [--sources S] [--mode opt]

One step = one slide of the window: a batch of 10^4 insertions + 10^4
deletions (configs[1], LiveJournal-shaped R-MAT) applied through the C ABI
(ppr_apply_batch): graph-store apply -> invariant restore -> two-phase push
to eps.  Prints ONE JSON line (rank 0).

value  : edge updates/s with the batch already resident in HBM
         (PPR_MEM_DEVICE), summed over the K timed steps' CUDA-event times.
e2e    : the same metric through the same call with pinned HOST buffers
         (H2D of the batch and D2H of the stats inside the timed region).
N > 1  : one process per GPU; rank r maintains its own source (weak scaling:
         S = N sources); rank 0 owns the stream and broadcasts every batch
         over NCCL (the one exchange step), each rank applies it to its graph
         replica.  Step time = max over ranks.
--sources S : S sources in total (SHARED push with several per rank),
         partitioned over the ranks by G0 out-degree (dist.partition_sources);
         value then counts source-edge-updates/s (each update once per source).
--shard R/G : one process runs only rank R's shard of a G-GPU run of the same
         sources (the per-rank load of a multi-GPU run, measured on one GPU).
--impl reference : the CPU oracle (CPU-Seq, 1 thread) on the same workload,
         bounded by --ref-budget-s; rank 0 only.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

# algorithmic bytes per unit: a pushed edge is
# 24 B = 8 B of walk (v id + d_out(v)) + 16 B of R(v) read+write.  The shared
# multi-source kernel walks an in-arc once per (source group, arc), so its
# bytes are 8 per walked arc + 16 per (source, arc) propagation.
B_EDGE, B_VERTEX, B_ARC = 24, 52, 56
B_WALK, B_PROP = 8, 16


def parse():
    p = argparse.ArgumentParser()
    p.add_argument("--gpus", type=int, default=1)
    p.add_argument("--steps", type=int, default=100)
    p.add_argument("--warmup", type=int, default=5)
    p.add_argument("--workload", default="lj")
    p.add_argument("--impl", default="ours", choices=["ours", "reference"])
    p.add_argument("--sources", type=int, default=0, help="total sources (0: one per rank)")
    p.add_argument("--mode", default="auto",
                   help="push mode; auto: opt with one source per rank, scan (EAGER_SCAN) with several")
    p.add_argument("--eps", type=float, default=None)
    p.add_argument("--ins", type=int, default=None)
    p.add_argument("--dele", type=int, default=None)
    p.add_argument("--seed", type=int, default=42)
    p.add_argument("--band", type=int, default=None,
                   help="sources drawn from the top-BAND out-degree vertices (default: the config's 1000)")
    p.add_argument("--shard", default=None,
                   help="R/G: run only rank R's source shard of a G-GPU run on this one GPU "
                        "(per-rank load of a multi-GPU run; scaling projection)")
    p.add_argument("--no-cpu-baseline", action="store_true")
    p.add_argument("--cpu-budget-s", type=float, default=30.0)
    p.add_argument("--ref-budget-s", type=float, default=150.0)
    p.add_argument("--no-flush", action="store_true")
    p.add_argument("--no-e2e", action="store_true")
    p.add_argument("--backend", default="nccl", choices=["nccl", "gloo"],
                   help="process-group backend (gloo: test the multi-rank path on one GPU)")
    p.add_argument("--relabel", type=int, default=-1,
                   help="1: degree-ordered internal ids, 0: external ids, -1: by size (default)")
    return p.parse_args()


# ---------------------------------------------------------------- helpers

class ClockSampler:
    """nvidia-smi clocks + throttle reasons sampled during the timed region."""
    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.active,clocks_event_reasons.hw_slowdown,"
         "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
         "clocks_event_reasons.sw_power_cap")

    def __init__(self, index):
        self.index = index
        self.rows = []
        self.proc = None

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.Q}",
                 "--format=csv,noheader,nounits", "-lms", "200"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.rows.append([x.strip() for x in line.split(",")])

    def stop(self):
        if not self.proc:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unavailable"]}
        self.proc.terminate()
        try:
            self.proc.wait(timeout=5)
        except Exception:
            self.proc.kill()
        self.t.join(timeout=2)
        sm = [float(r[0]) for r in self.rows if r and r[0].replace(".", "").isdigit()]
        mx = [float(r[1]) for r in self.rows if len(r) > 1 and r[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = set()
        for r in self.rows:
            for i, nm in enumerate(names):
                if len(r) > 3 + i and r[3 + i].lower() == "active":
                    reasons.add(nm)
        busy = [x for x in sm if x > 300] or sm
        return {"sm_mhz": statistics.median(busy) if busy else None,
                "sm_max_mhz": max(mx) if mx else None, "reasons": sorted(reasons),
                "samples": len(self.rows)}


def measured_peak():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            return float(json.load(f)["hbm_gbs"]), "measured"
    except Exception:
        return 6650.0, "fallback"


def profile_traffic(workload):
    """dram bytes per push launch from a committed ncu --set full capture, if any."""
    path = os.path.join(ROOT, "profiles", "push_traffic.json")
    try:
        with open(path) as f:
            d = json.load(f)
        return d.get(workload, {}).get("dram_bytes_per_launch")
    except Exception:
        return None


def cpu_info():
    model = ""
    try:
        with open("/proc/cpuinfo") as f:
            for line in f:
                if line.startswith("model name"):
                    model = line.split(":", 1)[1].strip()
                    break
    except Exception:
        pass
    return model, os.cpu_count()


# ---------------------------------------------------------------- distributed

def dist_env():
    ws = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return ws, rank, local


# ---------------------------------------------------------------- reference arm

def run_reference(args):
    ws, rank, _ = dist_env()
    if rank != 0:
        return
    if args.workload == "twitter":
        print(json.dumps({"impl": "reference", "unavailable": "the sequential oracle cannot build and "
                          "statically push a 1.5e9-arc window within a bounded sample"}), flush=True)
        return
    import oracle
    from paper_journals_pvldb_guolst17_b200 import workload as W
    over = {}
    if args.ins is not None:
        over["ins"] = args.ins
    if args.dele is not None:
        over["dele"] = args.dele
    if args.band is not None:
        over["band"] = args.band
    st, cfg = W.make_stream(args.workload, seed=args.seed, **over)
    eps = args.eps or cfg["eps"]
    g0s, g0d = st.window()
    S = args.sources or ws
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], S)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs[:1], 0.15, eps)
    t0 = time.perf_counter()
    o.push(oracle.SEQ)
    t_static = time.perf_counter() - t0
    per = []
    for _ in range(min(args.warmup, 1)):
        o.apply(*st.next_batch())
    for k in range(args.steps):
        b = st.next_batch()
        t0 = time.perf_counter()
        o.apply(*b, mode=oracle.SEQ)
        per.append(time.perf_counter() - t0)
        if sum(per) > args.ref_budget_s:
            break
    upd = cfg["ins"] + cfg["dele"]
    if cfg["undirected"]:
        upd = upd  # undirected updates counted as given (not doubled)
    T = sum(per)
    value = upd * len(per) / T
    model, ncpu = cpu_info()
    line = {
        "impl": "reference", "metric": "edge updates/s", "value": value, "unit": "edge updates/s",
        "n_gpus": args.gpus, "steps": len(per), "warmup": min(args.warmup, 1),
        "ms_per_step": 1e3 * T / len(per), "higher_is_better": True, "scaling": "weak",
        "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": config_block(args, cfg, eps, S),
        "cpu_baseline": {"value": value, "unit": "edge updates/s", "cores": 1, "kind": "oracle",
                         "sample": f"{len(per)} slides of {cfg['ins']}+{cfg['dele']} after an untimed "
                                   f"static push ({t_static:.1f} s), source rank-band top-{cfg['band']}, "
                                   f"single thread on {ncpu}-core {model}",
                         "sources_maintained": 1},
        "e2e": {"value": value, "unit": "edge updates/s", "h2d_bytes_per_step": 0,
                "d2h_bytes_per_step": 0},
    }
    if S > 1:
        line["note"] = ("oracle maintains 1 of the S sources; multiply ms_per_step by S for the "
                        "sequential cost of all sources")
    print(json.dumps(line), flush=True)


def config_block(args, cfg, eps, S):
    return {"workload": args.workload, "n": cfg["n"], "m_stream": cfg["m"],
            "window": cfg["window"] if cfg["window"] is not None else "resident",
            "batch": f"{cfg['ins']} ins + {cfg['dele']} del per slide",
            "undirected": cfg["undirected"], "alpha": 0.15, "eps": eps,
            "source_band": f"top-{cfg['band']} out-degree", "sources": S,
            "rmat_abc": list(cfg["abc"]), "mode": args.mode,
            "internal_ids": {1: "G0 out-degree order", 0: "external", -1: "auto (degree order iff not SHARED and R+d_out > 48 MB)"}[args.relabel],
            "l2": ("persisting lines reset + flushed between steps (512 MiB write)"
                   if not args.no_flush else "not flushed"),
            **({"shard": f"rank {args.shard} of the sources (one GPU's load of a multi-GPU run)"}
               if getattr(args, "shard", None) else {})}


# ---------------------------------------------------------------- our arm

def run_ours(args):
    import torch
    import torch.distributed as dist

    from paper_journals_pvldb_guolst17_b200 import dist as D, ppr, workload as W

    ws, rank, local = dist_env()
    local = local % max(torch.cuda.device_count(), 1)  # several ranks may share a GPU (gloo tests)
    if ws > 1:
        if args.backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", local))
        else:
            dist.init_process_group("gloo")
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    stream = torch.cuda.Stream(dev)  # the library runs on this stream; events are recorded on it
    torch.cuda.set_stream(stream)

    over = {}
    if args.ins is not None:
        over["ins"] = args.ins
    if args.dele is not None:
        over["dele"] = args.dele
    if args.band is not None:
        over["band"] = args.band
    cfg = dict(W.CONFIGS[args.workload])
    cfg.update(over)
    eps = args.eps or cfg["eps"]
    S = args.sources or ws
    if S < ws:
        raise SystemExit("--sources must be >= the world size")
    steps, warm = args.steps, max(args.warmup, 3)
    nslides = steps * (1 if args.no_e2e else 2) + warm
    und = bool(cfg["undirected"])
    nI, nD = cfg["ins"], cfg["dele"]  # per slide, as given (undirected: edges)

    # rank 0 owns the stream; the window, the sources and every batch reach the
    # other ranks over NCCL (setup untimed; the per-batch broadcast is timed)
    t0 = time.perf_counter()
    if rank == 0:
        st, cfg = W.make_stream(args.workload, seed=args.seed, **over)
        g0s, g0d = (st.src[st.lo:st.hi].copy(), st.dst[st.lo:st.hi].copy()) if und else st.window()
        arcs_s, arcs_d = W.expand_undirected(g0s, g0d) if und else (g0s, g0d)
        srcs = W.pick_sources(cfg["n"], arcs_s, arcs_d, cfg["band"], S)
        batches = []
        for _ in range(nslides):
            i0, i1 = st.hi, st.hi + nI
            d0, d1 = st.lo, st.lo + nD
            if und:  # the library expands undirected edges itself
                b = (st.src[i0:i1], st.dst[i0:i1], st.src[d0:d1], st.dst[d0:d1])
                st.hi, st.lo = i1, d1
            else:
                b = st.next_batch()
            batches.append(tuple(np.ascontiguousarray(x) for x in b))
        meta = torch.tensor([len(g0s)], dtype=torch.int64, device=dev)
    else:
        meta = torch.zeros(1, dtype=torch.int64, device=dev)
    t_gen = time.perf_counter() - t0
    if ws > 1:
        dist.broadcast(meta, 0)
    m0 = int(meta.item())
    if rank == 0:
        win = torch.from_numpy(np.stack([g0s, g0d]).view(np.int32)).to(dev)
        srct = torch.from_numpy(srcs.view(np.int32)).to(dev)
    else:
        win = torch.empty((2, m0), dtype=torch.int32, device=dev)
        srct = torch.empty(S, dtype=torch.int32, device=dev)
    if ws > 1:
        dist.broadcast(win, 0)
        dist.broadcast(srct, 0)
    win_np = win.cpu().numpy().view(np.uint32)
    srcs_all = srct.cpu().numpy().view(np.uint32)
    del win
    deg = np.bincount(win_np[0], minlength=cfg["n"])
    if und:
        deg = deg + np.bincount(win_np[1], minlength=cfg["n"])
    if args.shard:
        sr, sg = (int(x) for x in args.shard.split("/"))
        assert ws == 1 and 0 <= sr < sg, "--shard R/G emulates one rank of G on a single process"
        my_srcs = D.partition_sources(srcs_all, deg, sg, sr)
    else:
        my_srcs = D.partition_sources(srcs_all, deg, ws, rank)
    if args.mode == "auto":  # measured: Opt best single-source, SHARED for several sources per rank
        args.mode = "opt" if len(my_srcs) == 1 else "shared"

    t0 = time.perf_counter()
    h = ppr.Ppr(cfg["n"], win_np[0], win_np[1], my_srcs, alpha=0.15, eps=eps, mode=args.mode,
                device=local, stream=ctypes_stream(stream), undirected=und,
                relabel=args.relabel)
    torch.cuda.synchronize()
    t_create = time.perf_counter() - t0
    create_stats = h.create_stats
    del win_np

    counts = (nI, nD)
    nflat = 2 * (nI + nD)
    if rank == 0:
        dev_batches = [D.pack_batch(*b)[0].to(dev) for b in batches[:warm + steps]]
    else:
        dev_batches = [torch.empty(nflat, dtype=torch.int32, device=dev) for _ in range(warm + steps)]
    flush_buf = torch.empty(512 * 1024 * 1024 // 4, dtype=torch.int32, device=dev)

    def flush():
        if not args.no_flush:
            ppr.reset_persisting_l2()  # the handle pins R/d_out in L2; unpin, then evict
            flush_buf.fill_(1)

    def step_device(flat):
        flat = D.broadcast_batch(flat, counts)
        return h.apply_batch(*D.unpack_batch(flat, counts), mem=ppr.MEM_DEVICE)

    for t in range(warm):
        step_device(dev_batches[t])
    torch.cuda.synchronize()
    if ws > 1:
        dist.barrier()

    # timed: device-resident batches
    clocks = ClockSampler(local)
    clocks.start()
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True))
          for _ in range(steps)]
    stats = []
    torch.cuda.synchronize()
    if ws > 1:
        dist.barrier()
    for k in range(steps):
        flush()
        ev[k][0].record(stream)
        stats.append(step_device(dev_batches[warm + k]))
        ev[k][1].record(stream)
    torch.cuda.synchronize()
    if ws > 1:
        dist.barrier()
    ms = [a.elapsed_time(b) for a, b in ev]

    # timed: end to end from pinned host buffers through the same call
    e2e_ms, e2e_stats = [], []
    if not args.no_e2e:
        host = []
        if rank == 0:
            host = [D.pack_batch(*b)[0].pin_memory() for b in batches[warm + steps:warm + 2 * steps]]
        buf = torch.empty(nflat, dtype=torch.int32, device=dev)
        for k in range(steps):
            flush()
            a_, b_ = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a_.record(stream)
            if ws > 1:
                if rank == 0:
                    buf.copy_(host[k], non_blocking=True)
                s_ = step_device(buf)
                s_["h2d_bytes"] = 4 * nflat if rank == 0 else 0
            else:
                hb = host[k].numpy().view(np.uint32)
                s_ = h.apply_batch(*D.unpack_batch(hb, counts), mem=ppr.MEM_HOST)
            b_.record(stream)
            b_.synchronize()
            e2e_ms.append(a_.elapsed_time(b_))
            e2e_stats.append(s_)
        torch.cuda.synchronize()
    clk = clocks.stop()

    # post-run validity: termination (-eps <= R <= eps) for this rank's first source
    P0, R0 = h.query(0)
    term_ok = bool(np.all(np.abs(R0) <= eps))
    term_ok = D.max_over_ranks(0.0 if term_ok else 1.0, device=dev) == 0.0

    T = D.max_over_ranks(sum(ms), device=dev)
    T_e2e = D.max_over_ranks(sum(e2e_ms), device=dev) if e2e_ms else 0.0
    push_ms = sum(s["ms_push"] for s in stats)
    edges_r0 = sum(s["pushed_edges"] for s in stats)
    verts_r0 = sum(s["pushes"] for s in stats)
    walks_r0 = sum(s["walk_edges"] for s in stats)
    edges, verts, launches = D.sum_over_ranks(
        [edges_r0, verts_r0, sum(s["kernel_launches"] for s in stats)], device=dev)
    dev_bytes = h.device_bytes
    h.close()
    if rank != 0:
        if ws > 1:
            dist.destroy_process_group()
        return

    upd = nI + nD
    value = S * upd * steps / (T / 1e3)
    e2e_value = S * upd * len(e2e_ms) / (T_e2e / 1e3) if e2e_ms else None
    peak, peak_kind = measured_peak()
    # dominant kernel: the persistent push (one launch per step), rank 0's launches
    bytes_per_launch = (B_WALK * walks_r0 + B_PROP * edges_r0 + B_VERTEX * verts_r0) / steps
    push_ms_avg = push_ms / steps
    achieved = bytes_per_launch / (push_ms_avg / 1e3) / 1e9 if push_ms_avg > 0 else 0.0
    traffic = profile_traffic(args.workload) if S == 1 else None

    line = {
        "metric": "edge updates/s", "value": value,
        "unit": "edge updates/s",  # with S sources each update counts once per source
        "n_gpus": ws, "steps": steps, "warmup": warm, "ms_per_step": T / steps,
        "higher_is_better": True, "scaling": "weak" if not args.sources else "strong",
        "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": config_block(args, cfg, eps, S),
        "e2e": ({"value": e2e_value, "unit": "edge updates/s",
                 "h2d_bytes_per_step": int(np.mean([s["h2d_bytes"] for s in e2e_stats])),
                 "d2h_bytes_per_step": int(np.mean([s["d2h_bytes"] for s in e2e_stats])),
                 "ms_per_step": T_e2e / len(e2e_ms)} if e2e_ms else None),
        "gpu_launches": int(launches),
        "roofline": {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                     "frac": achieved / peak, "traffic": traffic,
                     "kernel": f"k_push<{args.mode.upper()}> (persistent, 1 launch/step)",
                     "algorithmic_bytes_per_launch": bytes_per_launch,
                     "peak_kind": peak_kind, "ms_per_launch": push_ms_avg},
        "clocks": clk,
        "checks": {"termination_all_ranks": term_ok},
        "detail": {
            "ms_per_step_p50": statistics.median(ms), "ms_per_step_p95": float(np.percentile(ms, 95)),
            "ms_store": sum(s["ms_store"] for s in stats) / steps,
            "ms_restore": sum(s["ms_restore"] for s in stats) / steps,
            "ms_push": push_ms_avg,
            "pushed_edges_per_s": edges / (T / 1e3),
            "pushes_per_step": verts / steps / S,
            "pushed_edges_per_step": edges / steps / S,
            "walk_edges_per_step_rank0": walks_r0 / steps,
            "iters_per_step": sum(s["iters_pos"] + s["iters_neg"] for s in stats) / steps,
            "rebuilds": sum(s["rebuilt"] for s in stats),
            "atomics_per_s_rank0": (edges_r0 + verts_r0) / (push_ms / 1e3) if push_ms else None,
            "generate_s": t_gen, "create_s": t_create, "create_stats": create_stats,
            "device_bytes_rank0": dev_bytes, "sources_per_rank": len(my_srcs),
        },
    }
    if not args.no_cpu_baseline and ws == 1 and args.workload == "twitter":
        line["cpu_baseline"] = {"value": None, "unit": "edge updates/s", "cores": 1, "kind": "oracle",
                                "unavailable": "the sequential oracle cannot finish the static push of a "
                                               "1.5e9-arc resident window within a bounded sample"}
    elif not args.no_cpu_baseline and ws == 1:
        arcs = (W.expand_undirected(g0s, g0d) if und else (g0s, g0d))
        bl = [(W.expand_undirected(b[0], b[1]) + W.expand_undirected(b[2], b[3])) if und else b
              for b in batches]
        line["cpu_baseline"] = cpu_baseline(args, cfg, eps, my_srcs[:1], arcs[0], arcs[1], bl)
    print(json.dumps(line), flush=True)
    if ws > 1:
        dist.destroy_process_group()


def ctypes_stream(stream):
    return stream.cuda_stream


def cpu_baseline(args, cfg, eps, srcs, g0s, g0d, batches):
    """The oracle (as it stands, CPU-Seq, 1 thread) on a bounded sample of the
    same workload: untimed create + static push on the same window, then the
    same slides, timed until --cpu-budget-s is used."""
    import oracle
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, eps)
    t0 = time.perf_counter()
    o.push(oracle.SEQ)
    t_static = time.perf_counter() - t0
    per = []
    for b in batches:
        t0 = time.perf_counter()
        o.apply(*b, mode=oracle.SEQ)
        per.append(time.perf_counter() - t0)
        if sum(per) > args.cpu_budget_s:
            break
    model, ncpu = cpu_info()
    upd = cfg["ins"] + cfg["dele"]
    return {"value": upd * len(per) / sum(per), "unit": "edge updates/s", "cores": 1,
            "kind": "oracle",
            "sample": f"first {len(per)} slides of the same stream and source (rank 0's), "
                      f"after an untimed static push of {t_static:.1f} s; 1 thread of "
                      f"{ncpu}-core {model}",
            "ms_per_step": 1e3 * sum(per) / len(per)}


def main():
    args = parse()
    if args.impl == "reference":
        run_reference(args)
    else:
        run_ours(args)


if __name__ == "__main__":
    main()
