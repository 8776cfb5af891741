"""Parser for tests/golden/figures_1_2_3.txt (the paper's worked example).

Pure data plumbing: no PPR arithmetic.  Shared by the oracle pins and the GPU
parity tests, which both compare against the paper's printed values."""
import math
import os

GOLDEN = os.path.join(os.path.dirname(os.path.abspath(__file__)), "golden", "figures_1_2_3.txt")

# G0 of the example, 0-based (v1..v4 -> 0..3); see the golden file header.
N = 4
G0_SRC = [0, 1, 2, 2, 3]
G0_DST = [3, 0, 0, 1, 2]
SOURCE = 0
ALPHA = 0.5
EPS = 0.1


def load():
    blocks = {}
    cur = None
    with open(GOLDEN) as f:
        for line in f:
            line = line.strip()
            if not line or line.startswith("#"):
                continue
            tok = line.split()
            if tok[0] == "block":
                cur = tok[1]
                blocks[cur] = {"cite": tok[2], "R": [None] * N, "P": [None] * N, "typo": set()}
                continue
            v = int(tok[0]) - 1
            blocks[cur]["R"][v] = float(tok[1])
            blocks[cur]["P"][v] = float(tok[2])
            if len(tok) > 3 and tok[3] == "typo":
                blocks[cur]["typo"].add(v)
    return blocks


def trunc4(x):
    """The figures' printing rule: truncate toward zero to 4 decimals."""
    return math.floor(abs(x) * 1e4 + 1e-9) / 1e4 * (1 if x >= 0 else -1)


def matches_printed(x, printed):
    return abs(trunc4(x) - printed) < 1e-12
