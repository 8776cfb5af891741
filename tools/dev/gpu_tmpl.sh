#!/bin/bash
mkdir -p gpurun_out/tmpl
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > gpurun_out/tmpl/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/tmpl/pytest_gpu.log
bash tools/dev/gpu_pooldeg.sh 2>&1 | grep -E "step|failed"
timeout 900 python bench.py --workload ms-lj --steps 5 --no-cpu-baseline --no-e2e > gpurun_out/tmpl/ms.json 2> gpurun_out/tmpl/ms.err
python -c "import json;d=json.load(open('gpurun_out/tmpl/ms.json'));x=d['detail'];print('ms', 'step %.2f push %.2f store %.2f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], d['roofline']['frac']))" 2>/dev/null || { echo "ms failed"; tail -3 gpurun_out/tmpl/ms.err; }
