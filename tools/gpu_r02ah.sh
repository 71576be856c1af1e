#!/bin/bash
# staged SpMV march (TEA_SPMV_STG rows of cp.async staging) vs the register-prefetch march
mkdir -p gpurun_out
python tools/dump_u.py /tmp/u_stg3.npz > gpurun_out/dump_ah.log 2>&1
TEA_B200_LIB=build_variants/stg0.so python tools/dump_u.py /tmp/u_stg0.npz >> gpurun_out/dump_ah.log 2>&1
python - <<'PY'
import numpy as np
a = np.load("/tmp/u_stg3.npz"); b = np.load("/tmp/u_stg0.npz")
for k in a.files:
    print(k, "bitwise" if np.array_equal(a[k], b[k]) else f"DIFF max {np.max(np.abs(a[k]-b[k]))}")
PY
tail -1 gpurun_out/dump_ah.log
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_ah.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_ah.log
bash tools/gpu_ab.sh stg "stg0 default stg2 stg4" "--no-variants" 2
bash tools/gpu_ab.sh stg_cg "stg0 default stg4" "--method cg --no-variants" 1
