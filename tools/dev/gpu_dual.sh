#!/bin/bash
mkdir -p gpurun_out/dual
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > gpurun_out/dual/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/dual/pytest_gpu.log
bash tools/dev/gpu_pooldeg.sh 2>&1 | grep -E "step|failed"
for v in rcp div; do
  PPR_LIB=$PWD/build/msdiv/libppr_$v.so timeout 900 python bench.py --workload ms-lj --steps 5 --no-cpu-baseline --no-e2e > gpurun_out/dual/ms_$v.json 2> gpurun_out/dual/ms_$v.err
  python -c "import json;d=json.load(open('gpurun_out/dual/ms_$v.json'));x=d['detail'];print('ms $v', 'step %.2f push %.2f frac %.3f' % (d['ms_per_step'], x['ms_push'], d['roofline']['frac']))" 2>/dev/null || { echo "ms $v failed"; tail -3 gpurun_out/dual/ms_$v.err; }
done
