cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag5.log; : > $O
run() { echo "== $*" >> $O; timeout 120 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=90 DIAG_N=2000 python tools/split_diag.py C5 1 1
run CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=90 DIAG_N=5000 python tools/split_diag.py C5 1 1
grep -v "Exception ignored\|culi.py\", line 28\|NoneType" $O | head -60
