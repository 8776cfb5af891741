#!/bin/bash
mkdir -p gpurun_out/sb
for lib in build/variants/libppr_*.so; do echo "== $lib"; PPR_LIB=$PWD/$lib timeout 300 python tools/dev/sb_prof.py 2>&1 | tail -14; done
