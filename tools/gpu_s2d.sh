cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
python tools/one_form.py @carlist:16384 3
timeout 600 ncu --set full --import-source on --clock-control none -k regex:"culi_eval" -s 2 -c 1 -o $OUT/s2d_carlist -f python tools/one_form.py @carlist:16384 3 > $OUT/s2d.log 2>&1
ncu -i $OUT/s2d_carlist.ncu-rep --page source --csv --print-source sass > $OUT/s2d_carlist_sass.csv 2>/dev/null
python tools/ncu_summary.py full $OUT/s2d_carlist.ncu-rep 2>&1 | head -8
