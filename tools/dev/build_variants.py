"""Builds libppr variants (extra -D flags) into build/variants/ in parallel (dev A/B helper)."""
import subprocess, sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
from paper_journals_pvldb_guolst17_b200 import build as b

def main(specs):
    os.makedirs("build/variants", exist_ok=True)
    procs = []
    for spec in specs:
        name, _, flags = spec.partition("=")
        out = f"build/variants/libppr_{name}.so"
        cmd = b.nvcc_cmd(out=out, extra=tuple(f for f in flags.split(",") if f))
        procs.append((name, subprocess.Popen(cmd, stdout=subprocess.DEVNULL, stderr=subprocess.PIPE, text=True)))
    for name, p in procs:
        _, err = p.communicate()
        print(name, "ok" if p.returncode == 0 else "FAILED\n" + err[-2000:])

if __name__ == "__main__":
    main(sys.argv[1:])
