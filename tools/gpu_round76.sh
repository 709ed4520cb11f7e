#!/bin/bash
# inv(L) form by recursive 2x2 block inversion: trsm tests, full-size parity, Cholesky alone, bench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build76.log 2>&1
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x -k "trsm" > gpurun_out/t76_tiles.log 2>&1; echo "exit $?" >> gpurun_out/t76_tiles.log
timeout 600 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_fullsize.py -q -p no:cacheprovider -x > gpurun_out/t76_rt.log 2>&1; echo "exit $?" >> gpurun_out/t76_rt.log
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --only ch --dump-log gpurun_out/b76_ch.json > gpurun_out/b76_ch.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/b76.json > gpurun_out/b76.log 2>&1
