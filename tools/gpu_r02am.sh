#!/bin/bash
# u += alpha p in the last fused pass (TEA_CPPCG_UPD=1) re-measured with 5-row later-pass staging
mkdir -p gpurun_out
bash tools/gpu_ab.sh upd "default upd1" "--no-variants" 3
