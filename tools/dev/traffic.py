"""Pairs the ncu --set full capture of one k_push launch with the algorithmic
bytes of the same slide (from the bench JSON printed by the same profiled run)
and records them in profiles/push_traffic.json (read by bench.py's roofline
`traffic`).

    python tools/dev/traffic.py WORKLOAD NCU_REP BENCH_OUT SLIDE_INDEX [--source TEXT]

SLIDE_INDEX: index into detail.per_step_rank0 of the profiled slide (the ncu
-s count selects which launch: create = launch 0, warm-up slides 1..W, timed
slide k = launch W + 1 + k)."""
import csv
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
B_EDGE, B_VERTEX = 24, 52


def ncu_metrics(rep, names):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(out.splitlines()))
    h, units, vals = rows[0], rows[1], rows[2]
    res = {}
    for n, u, v in zip(h, units, vals):
        if n in names:
            x = float(v.replace(",", ""))
            scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12,
                     "ns": 1e-9, "us": 1e-6, "usecond": 1e-6, "ms": 1e-3, "msecond": 1e-3}.get(u, 1)
            res[n] = x * scale
    return res


def main():
    wl, rep, bench_out, idx = sys.argv[1], sys.argv[2], sys.argv[3], int(sys.argv[4])
    src = sys.argv[sys.argv.index("--source") + 1] if "--source" in sys.argv else rep
    line = [l for l in open(bench_out).read().splitlines() if l.startswith("{")][-1]
    step = json.loads(line)["detail"]["per_step_rank0"][idx]
    m = ncu_metrics(rep, {"dram__bytes_read.sum", "dram__bytes_write.sum", "gpu__time_duration.sum",
                          "lts__t_sector_hit_rate.pct"})
    dram = m["dram__bytes_read.sum"] + m["dram__bytes_write.sum"]
    alg = B_EDGE * step["pushed_edges"] + B_VERTEX * step["pushes"]
    path = os.path.join(ROOT, "profiles", "push_traffic.json")
    d = json.load(open(path)) if os.path.exists(path) else {}
    d[wl] = {"slide": step["slide"], "pushed_edges": step["pushed_edges"], "pushes": step["pushes"],
             "algorithmic_bytes": alg, "dram_bytes": dram,
             "dram_read_bytes": m["dram__bytes_read.sum"], "dram_write_bytes": m["dram__bytes_write.sum"],
             "dram_over_algorithmic": dram / alg,
             "dram_bytes_per_pushed_edge": dram / step["pushed_edges"],
             "ncu_duration_ms": m.get("gpu__time_duration.sum", 0) * 1e3,
             "l2_sector_hit_pct": m.get("lts__t_sector_hit_rate.pct"),
             "source": src}
    json.dump(d, open(path, "w"), indent=1)
    print(json.dumps(d[wl], indent=1))


if __name__ == "__main__":
    main()
