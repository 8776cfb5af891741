#!/bin/bash
# exactly-once enqueue check: new tests, full GPU suite, default bench (perf unchanged?)
OUT=gpurun_out/chk2; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1 || { echo build failed; tail $OUT/build.log; exit 1; }
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "exactly_once or enqueue_check" > $OUT/pt_new.log 2>&1; echo "new tests rc=$? $(tail -1 $OUT/pt_new.log)"; grep -E "FAIL|assert|Error" $OUT/pt_new.log | head -5
timeout 1800 python -m pytest tests -m gpu -q --timeout 900 > $OUT/pytest_gpu.log 2>&1; echo "pytest rc=$? $(tail -1 $OUT/pytest_gpu.log)"
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo "smoke rc=$? $(tail -1 $OUT/smoke.log)"
timeout 900 python bench.py > $OUT/bench.json 2> $OUT/bench.err; echo "bench rc=$?"; python -c "import json;d=json.load(open('$OUT/bench.json'));print(d['value'], d['ms_per_step'], d['roofline']['frac'], d['clocks'], d['e2e']['value'], d['multi_source']['ms_per_step'])"
